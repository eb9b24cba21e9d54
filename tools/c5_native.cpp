// c5_native.cpp — config C5 (BASELINE.json configs[4]) driven natively: the OLTP
// side, the epoch cutter and the OLAP query loop are C++ threads calling the C ABI, so no
// interpreter lock couples them (the round-1 Python driver's p99 freshness lag was dominated by
// three Python threads sharing one GIL).
//
// Paper anchors: the task-parallel archipelago runs OLTP against a row store (PAPER.md L587-630,
// out of scope — this is a load generator); the data-parallel archipelago runs OLAP on a snapshot
// taken every epoch (L555-572); updates copy-on-write the pages they touch (L573-586); the
// freshness / performance trade-off is the snapshot period (L712-720, L833-870).
//
// Threads:
//   OLTP x K: TPC-C NewOrder (TPC-C 2.4 [EXT]: d uniform, c NURand(1023), ol_cnt U[5,15], items
//             NURand(8191), qty U[1,10], amount = qty x i_price) and Delivery (2.7.4: per district
//             the oldest undelivered order gets a carrier, its lines the delivery time, its
//             new_order row is deleted) at the TPC-C mix ratio 45:4, offered at a fixed rate;
//             thread k owns warehouses w = k mod K (no conflicts); commits append NSM records
//             and log in-place updates under one mutex;
//   cutter:   every E ms takes the committed rows + logged updates (copied under the mutex) and
//             publishes them as a new epoch with h2tap_refresh_rows (column extraction, H2D,
//             copy-on-write of the updated columns), then records the epoch's cut time;
//   queries:  loops h2tap_run_queries(Q1 at 2025-01-01 = lines delivered since the load, Q6, Q1,
//             Q18) on the latest published epoch; freshness lag = query start - cut time of the
//             epoch it read.
// Output: one JSON line. --dump DIR additionally writes the final row store and the final epoch's
// Q6 / Q1 / Q18 results (raw little-endian arrays + manifest.json) for the oracle check in
// tests/test_gpu_c5_native.py (the oracle is test infrastructure: this program never uses it).
//
// Build: tools/c5_native.py (g++ -O2 -pthread, links the in-tree libh2tap.so).
#include <algorithm>
#include <array>
#include <atomic>
#include <chrono>
#include <cinttypes>
#include <cmath>
#include <cstddef>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <deque>
#include <map>
#include <mutex>
#include <random>
#include <string>
#include <thread>
#include <vector>

#include "h2tap.h"

namespace {

using Clock = std::chrono::steady_clock;
constexpr int64_t kNull = INT64_MIN;
constexpr int kDistricts = 10, kOrders = 3000, kCustomers = 3000, kItems = 100000, kDelivered = 2101;
constexpr int64_t kTs1995 = 788918400000000LL, kTs2025 = 1735689600000000LL, kDayUs = 86400000000LL;

// NSM records (the OLTP side's layout); the refresh extracts the hot-path fields by offset
struct OlRec { int32_t w, d, o, number, i_id, supply_w; int64_t delivery; int32_t qty, pad; int64_t amount; };
struct ORec { int32_t w, d, o, c, ol_cnt, carrier, all_local, pad; int64_t entry; };
struct CRec { int32_t w, d, c, last, state_p2; };

struct Args {
    int W = 100, threads = 4, device = 0;
    double seconds = 20, epoch_ms = 100, tps = 400000;
    uint64_t seed = 1;
    std::string dump;
};

uint64_t nurand(std::mt19937_64 &g, uint64_t A, uint64_t x, uint64_t y, uint64_t C) {
    std::uniform_int_distribution<uint64_t> a(0, A), b(x, y);
    return (((a(g) | b(g)) + C) % (y - x + 1)) + x;
}

double now_s(Clock::time_point t0) { return std::chrono::duration<double>(Clock::now() - t0).count(); }

struct Pending {  // an undelivered order: its row positions (orders, first line, new_order)
    int32_t o_id;
    uint64_t o_row, ol_row, no_row;
    int ol_cnt;
};

struct Store {
    std::vector<OlRec> ol;
    std::vector<ORec> o;
    std::vector<CRec> c;
    std::vector<int32_t> no;  // new_order rows as {w, d, o, deleted} quadruples (flat)
    size_t n_ol = 0, n_o = 0, n_no = 0;
    std::vector<int64_t> price;  // i_price by i_id - 1 (cents)
    std::vector<int32_t> next_oid;  // per (w, d)
    std::vector<std::deque<Pending>> fifo;  // per (w, d)
    // in-place updates logged since the last cut
    std::vector<uint32_t> upd_ol_rows, upd_o_rows, upd_no_rows;
    std::vector<int64_t> upd_ol_vals;
    std::vector<int32_t> upd_o_vals;
    uint64_t txns = 0, deliveries = 0;
};

void populate(Store &S, const Args &a) {
    std::mt19937_64 g(a.seed);
    const size_t W = a.W;
    S.price.resize(kItems);
    for (auto &p : S.price) p = 100 + (int64_t)(g() % 9901);
    S.next_oid.assign(W * kDistricts + kDistricts + 1, kOrders + 1);
    S.fifo.resize(W * kDistricts + kDistricts + 1);
    S.c.reserve(W * kDistricts * kCustomers);
    S.o.reserve(W * kDistricts * kOrders);
    S.ol.reserve(W * kDistricts * kOrders * 10);
    for (int w = 1; w <= a.W; ++w)
        for (int d = 1; d <= kDistricts; ++d) {
            for (int c = 1; c <= kCustomers; ++c)
                S.c.push_back({w, d, c, c <= 1000 ? c - 1 : (int32_t)nurand(g, 255, 0, 999, 157),
                               (int32_t)((('A' + (int)(g() % 26)) << 8) | ('A' + (int)(g() % 26)))});
            std::vector<int32_t> perm(kCustomers);
            for (int i = 0; i < kCustomers; ++i) perm[i] = i + 1;
            std::shuffle(perm.begin(), perm.end(), g);
            for (int o = 1; o <= kOrders; ++o) {
                const int cnt = 5 + (int)(g() % 11);
                const int64_t entry = kTs1995 + (int64_t)(g() % (uint64_t)(kTs2025 - kTs1995));
                const bool delivered = o < kDelivered;
                const size_t o_row = S.o.size(), ol_row = S.ol.size();
                S.o.push_back({w, d, o, perm[o - 1], cnt, delivered ? 1 + (int)(g() % 10) : -1, 1, 0, entry});
                for (int n = 1; n <= cnt; ++n)
                    S.ol.push_back({w, d, o, n, 1 + (int32_t)(g() % kItems), w,
                                    delivered ? entry + (int64_t)(g() % (uint64_t)(30 * kDayUs)) : kNull,
                                    1 + (int32_t)(g() % 10), 0, 1 + (int64_t)(g() % 999999)});
                if (!delivered) {
                    S.fifo[w * kDistricts + d].push_back({o, o_row, ol_row, S.n_no, cnt});
                    S.no.insert(S.no.end(), {w, d, o, 0});
                    S.n_no++;
                }
            }
        }
    S.n_o = S.o.size();
    S.n_ol = S.ol.size();
}

h2tap_field F(uint32_t id, uint32_t type, size_t off) { return h2tap_field{id, type, (uint32_t)off}; }

struct Fields {
    std::vector<h2tap_field> ol, o, c, no;
    Fields() {
        ol = {F(H2TAP_OL_W_ID, H2TAP_I32, offsetof(OlRec, w)), F(H2TAP_OL_D_ID, H2TAP_I32, offsetof(OlRec, d)),
              F(H2TAP_OL_O_ID, H2TAP_I32, offsetof(OlRec, o)), F(H2TAP_OL_NUMBER, H2TAP_I32, offsetof(OlRec, number)),
              F(H2TAP_OL_DELIVERY_D, H2TAP_I64, offsetof(OlRec, delivery)),
              F(H2TAP_OL_QUANTITY, H2TAP_I32, offsetof(OlRec, qty)), F(H2TAP_OL_AMOUNT, H2TAP_I64, offsetof(OlRec, amount))};
        o = {F(H2TAP_O_W_ID, H2TAP_I32, offsetof(ORec, w)), F(H2TAP_O_D_ID, H2TAP_I32, offsetof(ORec, d)),
             F(H2TAP_O_ID, H2TAP_I32, offsetof(ORec, o)), F(H2TAP_O_C_ID, H2TAP_I32, offsetof(ORec, c)),
             F(H2TAP_O_OL_CNT, H2TAP_I32, offsetof(ORec, ol_cnt)), F(H2TAP_O_CARRIER_ID, H2TAP_I32, offsetof(ORec, carrier)),
             F(H2TAP_O_ENTRY_D, H2TAP_I64, offsetof(ORec, entry))};
        c = {F(H2TAP_C_W_ID, H2TAP_I32, offsetof(CRec, w)), F(H2TAP_C_D_ID, H2TAP_I32, offsetof(CRec, d)),
             F(H2TAP_C_ID, H2TAP_I32, offsetof(CRec, c)), F(H2TAP_C_LAST, H2TAP_I32, offsetof(CRec, last))};
        no = {F(H2TAP_NO_W_ID, H2TAP_I32, 0), F(H2TAP_NO_D_ID, H2TAP_I32, 4), F(H2TAP_NO_O_ID, H2TAP_I32, 8),
              F(H2TAP_NO_DELETED, H2TAP_I32, 12)};
    }
};

void check(h2tap_status st, const char *what) {
    if (st != H2TAP_OK) {
        std::fprintf(stderr, "%s failed (%d): %s\n", what, (int)st, h2tap_last_error());
        std::exit(2);
    }
}

double pct(std::vector<double> v, double p) {
    if (v.empty()) return NAN;
    std::sort(v.begin(), v.end());
    const size_t i = std::min(v.size() - 1, (size_t)std::llround(p / 100.0 * (double)(v.size() - 1)));
    return v[i];
}

void write_raw(const std::string &path, const void *p, size_t bytes) {
    FILE *f = std::fopen(path.c_str(), "wb");
    if (!f) { std::perror(path.c_str()); std::exit(2); }
    if (bytes) std::fwrite(p, 1, bytes, f);
    std::fclose(f);
}

}  // namespace

int main(int argc, char **argv) {
    Args a;
    for (int i = 1; i < argc; ++i) {
        std::string k = argv[i];
        auto v = [&] { return std::string(i + 1 < argc ? argv[++i] : ""); };
        if (k == "--warehouses") a.W = std::stoi(v());
        else if (k == "--seconds") a.seconds = std::stod(v());
        else if (k == "--epoch-ms") a.epoch_ms = std::stod(v());
        else if (k == "--tps") a.tps = std::stod(v());
        else if (k == "--threads") a.threads = std::stoi(v());
        else if (k == "--seed") a.seed = std::stoull(v());
        else if (k == "--device") a.device = std::stoi(v());
        else if (k == "--dump") a.dump = v();
        else { std::fprintf(stderr, "unknown argument %s\n", k.c_str()); return 2; }
    }
    Store S;
    const auto tp0 = Clock::now();
    populate(S, a);
    const double pop_s = now_s(tp0);
    // capacity for the whole run: the row store never reallocates (refresh reads rows in place)
    const size_t max_txn = (size_t)(a.tps * (a.seconds + 10) * 1.1) + 100000;
    S.o.resize(S.n_o + max_txn);
    S.ol.resize(S.n_ol + 15 * max_txn);
    S.no.resize(4 * (S.n_no + max_txn));

    h2tap_config cfg{a.device, 0, 1, 0};
    h2tap_engine *e = nullptr;
    check(h2tap_open(&cfg, &e), "h2tap_open");
    Fields FL;
    auto rows = [&](uint32_t tid, const std::vector<h2tap_field> &f, const void *rec, size_t rs, uint64_t n,
                    uint64_t first, uint32_t flags) {
        return h2tap_row_table{tid, (uint32_t)f.size(), f.data(), rec, rs, n, first, flags};
    };
    {
        h2tap_row_table t[4] = {rows(H2TAP_T_ORDER_LINE, FL.ol, S.ol.data(), sizeof(OlRec), S.n_ol, 0, H2TAP_FULL_RELOAD),
                                rows(H2TAP_T_ORDERS, FL.o, S.o.data(), sizeof(ORec), S.n_o, 0, H2TAP_FULL_RELOAD),
                                rows(H2TAP_T_CUSTOMER, FL.c, S.c.data(), sizeof(CRec), S.c.size(), 0, H2TAP_FULL_RELOAD),
                                rows(H2TAP_T_NEW_ORDER, FL.no, S.no.data(), 16, S.n_no, 0, H2TAP_FULL_RELOAD)};
        check(h2tap_load_snapshot_rows(e, t, 4, 1, 0), "initial load");
        check(h2tap_reserve(e, H2TAP_T_ORDER_LINE, S.ol.size()), "reserve");
        check(h2tap_reserve(e, H2TAP_T_ORDERS, S.o.size()), "reserve");
        check(h2tap_reserve(e, H2TAP_T_NEW_ORDER, S.no.size() / 4), "reserve");
    }

    std::mutex mu;
    std::atomic<bool> stop{false};
    std::map<uint64_t, double> cut_time;  // epoch -> cut (s since start)
    std::mutex cut_mu;
    uint64_t epoch = 1;
    size_t loaded_ol = S.n_ol, loaded_o = S.n_o, loaded_no = S.n_no;
    const auto t0 = Clock::now();
    cut_time[1] = 0.0;
    std::atomic<int64_t> clock_us{kTs2025 + 30 * kDayUs};  // the OLTP side's logical time
    double refresh_s = 0, refresh_bytes = 0;
    uint64_t refreshes = 0, rows_updated = 0;

    // ---- OLTP threads
    auto oltp = [&](int k) {
        std::mt19937_64 g(a.seed * 1000003ull + (uint64_t)k);
        const double rate = a.tps / a.threads;  // NewOrder per second offered by this thread
        const int batch = 200;
        uint64_t done = 0;
        std::vector<OlRec> lines;
        std::vector<ORec> ords;
        while (!stop.load(std::memory_order_relaxed)) {
            const double ahead = (double)done / rate - now_s(t0);
            if (ahead > 0) std::this_thread::sleep_for(std::chrono::duration<double>(ahead));
            lines.clear();
            ords.clear();
            struct Del { int w, carrier; };
            std::vector<Del> dels;
            for (int t = 0; t < batch; ++t) {
                // warehouses owned by this thread: w = k+1, k+1+K, ...
                const int nw = (a.W - 1 - k) / a.threads + 1;
                const int w = k + 1 + (int)(g() % (uint64_t)nw) * a.threads;
                const int d = 1 + (int)(g() % kDistricts);
                const int c = (int)nurand(g, 1023, 1, kCustomers, 259);
                const int cnt = 5 + (int)(g() % 11);
                ords.push_back({w, d, 0, c, cnt, -1, 1, 0, 0});
                for (int n = 1; n <= cnt; ++n) {
                    const int32_t item = (int32_t)nurand(g, 8191, 1, kItems, 7911);
                    const int32_t qty = 1 + (int32_t)(g() % 10);
                    lines.push_back({w, d, 0, n, item, w, kNull, qty, 0, qty * S.price[item - 1]});
                }
                if (g() % 45 < 4) dels.push_back({k + 1 + (int)(g() % (uint64_t)nw) * a.threads, 1 + (int)(g() % 10)});
            }
            {   // commit: rows and updates become visible to the next cut
                std::lock_guard<std::mutex> lk(mu);
                if (S.n_o + ords.size() > S.o.size() || S.n_ol + lines.size() > S.ol.size() ||
                    4 * (S.n_no + ords.size()) > S.no.size()) {  // row store capacity reached
                    stop.store(true);
                    break;
                }
                size_t li = 0;
                for (auto &o : ords) {
                    const int key = o.w * kDistricts + o.d;
                    o.o = S.next_oid[key]++;
                    o.entry = clock_us.fetch_add(1);
                    const uint64_t o_row = S.n_o++, ol_row = S.n_ol, no_row = S.n_no++;
                    S.o[o_row] = o;
                    for (int n = 0; n < o.ol_cnt; ++n, ++li) {
                        lines[li].o = o.o;
                        S.ol[S.n_ol++] = lines[li];
                    }
                    std::memcpy(&S.no[4 * no_row], std::array<int32_t, 4>{o.w, o.d, o.o, 0}.data(), 16);
                    S.fifo[key].push_back({o.o, o_row, ol_row, no_row, o.ol_cnt});
                }
                for (const auto &dl : dels) {
                    const int64_t ts = clock_us.fetch_add(1);
                    for (int d = 1; d <= kDistricts; ++d) {
                        auto &q = S.fifo[dl.w * kDistricts + d];
                        if (q.empty()) continue;
                        const Pending p = q.front();
                        q.pop_front();
                        S.o[p.o_row].carrier = dl.carrier;
                        S.upd_o_rows.push_back((uint32_t)p.o_row);
                        S.upd_o_vals.push_back(dl.carrier);
                        for (int n = 0; n < p.ol_cnt; ++n) {
                            S.ol[p.ol_row + n].delivery = ts;
                            S.upd_ol_rows.push_back((uint32_t)(p.ol_row + n));
                            S.upd_ol_vals.push_back(ts);
                        }
                        S.no[4 * p.no_row + 3] = 1;
                        S.upd_no_rows.push_back((uint32_t)p.no_row);
                    }
                }
                S.txns += (uint64_t)ords.size();
                S.deliveries += dels.size();
            }
            done += batch;
        }
    };

    // ---- epoch cutter
    std::vector<OlRec> d_ol;
    std::vector<ORec> d_o;
    std::vector<int32_t> d_no;
    std::vector<uint32_t> u_ol, u_o, u_no;
    std::vector<int64_t> v_ol;
    std::vector<int32_t> v_o, v_no;
    auto cut = [&]() {
        size_t n_ol, n_o, n_no;
        double t_cut;
        {
            std::lock_guard<std::mutex> lk(mu);  // a consistent snapshot of committed state
            n_ol = S.n_ol; n_o = S.n_o; n_no = S.n_no;
            t_cut = now_s(t0);
            d_ol.assign(S.ol.begin() + loaded_ol, S.ol.begin() + n_ol);
            d_o.assign(S.o.begin() + loaded_o, S.o.begin() + n_o);
            d_no.assign(S.no.begin() + 4 * loaded_no, S.no.begin() + 4 * n_no);
            u_ol.swap(S.upd_ol_rows); v_ol.swap(S.upd_ol_vals);
            u_o.swap(S.upd_o_rows); v_o.swap(S.upd_o_vals);
            u_no.swap(S.upd_no_rows);
            S.upd_ol_rows.clear(); S.upd_ol_vals.clear(); S.upd_o_rows.clear(); S.upd_o_vals.clear();
            S.upd_no_rows.clear();
        }
        v_no.assign(u_no.size(), 1);
        {   // the new epoch's logical time, visible to the query loop before it can read the epoch
            std::lock_guard<std::mutex> lk(cut_mu);
            cut_time[epoch + 1] = t_cut;
        }
        h2tap_row_table t[3] = {rows(H2TAP_T_ORDER_LINE, FL.ol, d_ol.data(), sizeof(OlRec), n_ol, loaded_ol, 0),
                                rows(H2TAP_T_ORDERS, FL.o, d_o.data(), sizeof(ORec), n_o, loaded_o, 0),
                                rows(H2TAP_T_NEW_ORDER, FL.no, d_no.data(), 16, n_no, loaded_no, 0)};
        h2tap_update u[3] = {{H2TAP_T_ORDER_LINE, H2TAP_OL_DELIVERY_D, H2TAP_I64, u_ol.size(), u_ol.data(), v_ol.data()},
                             {H2TAP_T_ORDERS, H2TAP_O_CARRIER_ID, H2TAP_I32, u_o.size(), u_o.data(), v_o.data()},
                             {H2TAP_T_NEW_ORDER, H2TAP_NO_DELETED, H2TAP_I32, u_no.size(), u_no.data(), v_no.data()}};
        const uint32_t nu = u_ol.empty() ? 0 : 3;
        const auto r0 = Clock::now();
        check(h2tap_refresh_rows(e, t, 3, nu ? u : nullptr, nu, epoch + 1, H2TAP_LOAD_ASYNC), "refresh");
        uint64_t pub = 0;
        check(h2tap_sync(e, &pub), "sync");
        refresh_s += std::chrono::duration<double>(Clock::now() - r0).count();
        refreshes++;
        refresh_bytes += (double)(n_ol - loaded_ol) * 36 + (double)(n_o - loaded_o) * 32 + (double)(n_no - loaded_no) * 16 +
                         (double)u_ol.size() * 12 + (double)u_o.size() * 8 + (double)u_no.size() * 8;
        rows_updated += u_ol.size() + u_o.size() + u_no.size();
        epoch++;
        loaded_ol = n_ol; loaded_o = n_o; loaded_no = n_no;
        u_ol.clear(); v_ol.clear(); u_o.clear(); v_o.clear(); u_no.clear();
    };
    std::thread cutter([&] {
        while (!stop.load()) {
            std::this_thread::sleep_for(std::chrono::duration<double>(a.epoch_ms / 1e3));
            if (!stop.load()) cut();
        }
    });
    std::vector<std::thread> workers;
    for (int k = 0; k < a.threads; ++k) workers.emplace_back(oltp, k);

    // ---- query loop (this thread)
    const int64_t q6p[4] = {915148800000000LL, 1577836800000000LL, 1, 100000};
    const int64_t q1_fresh[1] = {kTs2025};
    const h2tap_query batch[4] = {{H2TAP_Q1, 1, q1_fresh, 0}, {H2TAP_Q6, 4, q6p, H2TAP_RESULT_DEVICE},
                                  {H2TAP_Q1, 0, nullptr, H2TAP_RESULT_DEVICE}, {H2TAP_Q18, 0, nullptr, H2TAP_RESULT_DEVICE}};
    std::vector<double> lags, lat;
    std::vector<uint64_t> eps;
    int64_t delivered_first = -1, delivered_last = -1;
    uint64_t nq = 0;
    while (now_s(t0) < a.seconds) {
        const double tq = now_s(t0);
        h2tap_result *r[4];
        check(h2tap_run_queries(e, batch, 4, r), "queries");
        const double td = now_s(t0);
        int64_t delivered = 0;
        const int64_t *cnt = static_cast<const int64_t *>(r[0]->cols[5]);  // count_order
        for (uint64_t i = 0; i < r[0]->nrows; ++i) delivered += cnt[i];
        if (delivered_first < 0) delivered_first = delivered;
        delivered_last = delivered;
        double tc;
        {
            std::lock_guard<std::mutex> lk(cut_mu);
            tc = cut_time[r[0]->epoch];
        }
        lags.push_back((tq - tc) * 1e3);
        lat.push_back((td - tq) * 1e3);
        eps.push_back(r[0]->epoch);
        for (auto *x : r) h2tap_free(x);
        nq++;
    }
    stop.store(true);
    for (auto &t : workers) t.join();
    cutter.join();
    const double wall = now_s(t0);
    cut();  // the final epoch holds every committed transaction
    h2tap_store_stats ss{};
    check(h2tap_get_store_stats(e, &ss), "stats");
    std::sort(eps.begin(), eps.end());
    const size_t distinct = std::unique(eps.begin(), eps.end()) - eps.begin();
    std::printf("{\"config\": \"C5 mixed HTAP (native C++ driver), W=%d, 1 GPU, epoch period %.0f ms, NewOrder offered at "
                "%.0f tx/s by %d OLTP threads, Delivery at the TPC-C mix 4:45\", \"population_s\": %.1f, "
                "\"seconds\": %.2f, \"neworder_tx_per_s\": %.1f, \"delivery_tx_per_s\": %.1f, "
                "\"epochs_published\": %" PRIu64 ", \"rows_updated\": %" PRIu64 ", \"refresh_ms_per_epoch_mean\": %.3f, "
                "\"refresh_MB_per_s_while_refreshing\": %.1f, \"cow_pages_copied\": %" PRIu64 ", \"cow_full_copies\": %" PRIu64 ", "
                "\"query_batches_per_s\": %.1f, \"batch_latency_ms_p50\": %.3f, \"batch_latency_ms_p99\": %.3f, "
                "\"freshness_lag_ms_p50\": %.2f, \"freshness_lag_ms_p99\": %.2f, \"freshness_lag_ms_max\": %.2f, "
                "\"distinct_epochs_read\": %zu, \"q1_delivered_lines_first_last\": [%" PRId64 ", %" PRId64 "], "
                "\"final_order_line_rows\": %zu}\n",
                a.W, a.epoch_ms, a.tps, a.threads, pop_s, wall, (double)S.txns / wall, (double)S.deliveries / wall,
                refreshes, rows_updated, refresh_s / std::max<uint64_t>(refreshes, 1) * 1e3,
                refresh_bytes / std::max(refresh_s, 1e-9) / 1e6, ss.cow_pages_copied, ss.cow_full_copies,
                (double)nq / wall, pct(lat, 50), pct(lat, 99), pct(lags, 50), pct(lags, 99), pct(lags, 100), distinct,
                delivered_first, delivered_last, S.n_ol);
    if (!a.dump.empty()) {  // final row store + the final epoch's results (host), for the oracle check
        const std::string D = a.dump + "/";
        auto col = [&](const char *name, auto get, size_t n, size_t es) {
            std::vector<char> buf(n * es);
            for (size_t i = 0; i < n; ++i) get(i, buf.data() + i * es);
            write_raw(D + name, buf.data(), buf.size());
        };
        const size_t nol = S.n_ol, no = S.n_o, nc = S.c.size(), nno = S.n_no;
#define COL(NAME, VEC, FIELD, T, N) col(NAME, [&](size_t i, char *p) { T v = (T)VEC[i].FIELD; std::memcpy(p, &v, sizeof v); }, N, sizeof(T))
        COL("ol_w_id", S.ol, w, int32_t, nol); COL("ol_d_id", S.ol, d, int32_t, nol); COL("ol_o_id", S.ol, o, int32_t, nol);
        COL("ol_number", S.ol, number, int32_t, nol); COL("ol_delivery_d", S.ol, delivery, int64_t, nol);
        COL("ol_quantity", S.ol, qty, int32_t, nol); COL("ol_amount", S.ol, amount, int64_t, nol);
        COL("o_w_id", S.o, w, int32_t, no); COL("o_d_id", S.o, d, int32_t, no); COL("o_id", S.o, o, int32_t, no);
        COL("o_c_id", S.o, c, int32_t, no); COL("o_ol_cnt", S.o, ol_cnt, int32_t, no);
        COL("o_carrier_id", S.o, carrier, int32_t, no); COL("o_entry_d", S.o, entry, int64_t, no);
        COL("c_w_id", S.c, w, int32_t, nc); COL("c_d_id", S.c, d, int32_t, nc); COL("c_id", S.c, c, int32_t, nc);
        COL("c_last", S.c, last, int32_t, nc);
#undef COL
        write_raw(D + "new_order", S.no.data(), 16 * nno);
        h2tap_result *r[3];
        const h2tap_query fq[3] = {{H2TAP_Q6, 4, q6p, 0}, {H2TAP_Q1, 0, nullptr, 0}, {H2TAP_Q18, 0, nullptr, 0}};
        check(h2tap_run_queries(e, fq, 3, r), "final queries");
        FILE *m = std::fopen((D + "manifest.json").c_str(), "w");
        std::fprintf(m, "{\"epoch\": %" PRIu64 ", \"n_ol\": %zu, \"n_o\": %zu, \"n_c\": %zu, \"n_no\": %zu, \"results\": {",
                     r[0]->epoch, nol, no, nc, nno);
        const char *qn[3] = {"q6", "q1", "q18"};
        for (int q = 0; q < 3; ++q) {
            std::fprintf(m, "%s\"%s\": {\"nrows\": %" PRIu64 ", \"cols\": [", q ? ", " : "", qn[q], r[q]->nrows);
            for (uint32_t c = 0; c < r[q]->ncols; ++c) {
                const size_t es = r[q]->types[c] == H2TAP_I32 ? 4 : 8;
                const std::string f = std::string(qn[q]) + "." + r[q]->names[c];
                write_raw(D + f, r[q]->cols[c], es * r[q]->nrows);
                std::fprintf(m, "%s[\"%s\", %u, %d]", c ? ", " : "", r[q]->names[c], r[q]->types[c],
                             r[q]->nulls[c] ? (int)r[q]->nulls[c][0] : 0);
            }
            std::fprintf(m, "]}");
        }
        std::fprintf(m, "}}\n");
        std::fclose(m);
        for (auto *x : r) h2tap_free(x);
    }
    h2tap_close(e);
    return 0;
}
