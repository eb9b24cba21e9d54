// engine.cu — the C ABI (include/h2tap.h): snapshot store in HBM with epoch publish (a1),
// plan executors for CH Q1 / Q6 / Q18 (a2-a6, a8), the cross-GPU merge over peer segments (a7).
//
// Paper anchors:
//  - snapshot = shallow copy of the top-level container + epoch++ (L562-567); here a View is
//    an immutable {epoch, row count and device pointer per column}; appended rows go past every
//    published count, so earlier views stay valid (the append-only subset of copy-on-write,
//    L573-586) and views pin their buffers by reference count (the paper's epoch GC, L583-586).
//  - several queries may share one snapshot, or take one each (L555-559): run_query reads the
//    latest published view at entry; load_snapshot publishes a new one.
//  - "the runtime identifies the columns that are necessary for executing the OLAP query and
//    invokes the GPU kernel, passing in pointers" (L568-570): plans read only their columns.
#include <algorithm>
#include <atomic>
#include <chrono>
#include <cstdarg>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <deque>
#include <map>
#include <memory>
#include <mutex>
#include <string>
#include <thread>
#include <vector>

#include <cuda_runtime.h>

#include "../../include/h2tap.h"
#include "kernels.cuh"

// engines open per device in this process (a kernel with a grid barrier needs its grid alone on
// the device: two such grids from two engines could each hold part of the SMs and wait forever)
static std::mutex g_dev_mu;
static std::map<int, int> g_dev_engines;
static void engines_on_device_add(int dev, int d) {
    std::lock_guard<std::mutex> g(g_dev_mu);
    g_dev_engines[dev] += d;
}
static int engines_on_device(int dev) {
    std::lock_guard<std::mutex> g(g_dev_mu);
    auto it = g_dev_engines.find(dev);
    return it == g_dev_engines.end() ? 0 : it->second;
}

namespace h2tap {
static std::atomic<uint64_t> g_launches{0};
void count_launches(int n) { g_launches.fetch_add((uint64_t)n, std::memory_order_relaxed); }
bool pdl_enabled() {
    static const bool on = [] { const char *v = std::getenv("H2TAP_PDL"); return !(v && v[0] == '0'); }();
    return on;
}
uint64_t launches_total() { return g_launches.load(std::memory_order_relaxed); }
}  // namespace h2tap

using namespace h2tap;

// ============================================================== errors ===
namespace {
thread_local std::string g_err;

h2tap_status fail(h2tap_status st, const char *fmt, ...) {
    char buf[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(buf, sizeof buf, fmt, ap);
    va_end(ap);
    g_err = buf;
    return st;
}

struct Fail {  // thrown internally, converted to a status at the ABI boundary
    h2tap_status st;
};
[[noreturn]] void raise(h2tap_status st, const char *fmt, ...) {
    char buf[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(buf, sizeof buf, fmt, ap);
    va_end(ap);
    g_err = buf;
    throw Fail{st};
}
#define CK(call)                                                                           \
    do {                                                                                   \
        cudaError_t e_ = (call);                                                           \
        if (e_ != cudaSuccess)                                                             \
            raise(e_ == cudaErrorMemoryAllocation ? H2TAP_ENOMEM : H2TAP_ECUDA, "%s: %s (%s:%d)", \
                  #call, cudaGetErrorString(e_), __FILE__, __LINE__);                      \
    } while (0)

// ============================================================== schema ===
constexpr int kTables = 6;  // index = table id (1..5)
constexpr int kMaxCols = 9;
const int kNcols[kTables] = {0, 9, 8, 5, 3, 4};
const uint32_t kTypes[kTables][kMaxCols] = {
    {},
    {H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I64, H2TAP_I32, H2TAP_I64},
    {H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I64},
    {H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32},
    {H2TAP_I32, H2TAP_I64, H2TAP_I32},
    {H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I32}};
inline size_t type_size(uint32_t t) { return t == H2TAP_I32 ? 4 : 8; }
constexpr uint64_t kPadRows = 64;  // over-allocation so 128-bit loads of the last tile stay in bounds

// ============================================================ memory ===
// Streams a snapshot buffer's release is ordered after (DevBuf with a stream-ordered free).
struct FreeOrder {
    cudaStream_t compute = nullptr, copy = nullptr, reaper = nullptr;
};

struct DevBuf {  // one device allocation; freed when the last View referencing it dies
    void *ptr = nullptr;
    size_t bytes = 0;
    int device = 0;
    const FreeOrder *order = nullptr;  // null: cudaMalloc / cudaFree (synchronising)
    ~DevBuf() {
        if (!ptr) return;
        int cur;
        cudaGetDevice(&cur);
        cudaSetDevice(device);
        if (order) {
            // stream-ordered: released to the pool once everything already enqueued on the
            // compute and copy streams is done, on a third stream — no device-wide sync (a
            // cudaFree would stall every query and upload in flight) and no false dependency
            cudaEvent_t a, b;
            cudaEventCreateWithFlags(&a, cudaEventDisableTiming);
            cudaEventCreateWithFlags(&b, cudaEventDisableTiming);
            cudaEventRecord(a, order->compute);
            cudaEventRecord(b, order->copy);
            cudaStreamWaitEvent(order->reaper, a, 0);
            cudaStreamWaitEvent(order->reaper, b, 0);
            cudaFreeAsync(ptr, order->reaper);
            cudaEventDestroy(a);
            cudaEventDestroy(b);
        } else {
            cudaFree(ptr);
        }
        cudaSetDevice(cur);
    }
};
using DevBufP = std::shared_ptr<DevBuf>;

DevBufP dev_alloc(size_t bytes, int device) {
    auto b = std::make_shared<DevBuf>();
    b->device = device;
    b->bytes = bytes;
    CK(cudaMalloc(&b->ptr, bytes ? bytes : 16));
    return b;
}

// Snapshot column buffers: from the device's memory pool in copy-stream order (their first
// writer), released stream-ordered (above). The pool keeps freed memory (release threshold =
// max), so a full reload that cannot reuse the spare costs no cudaMalloc either.
DevBufP dev_alloc_ordered(size_t bytes, int device, const FreeOrder *order) {
    static const bool pool = [] { const char *v = std::getenv("H2TAP_POOL"); return !(v && v[0] == '0'); }();
    if (!pool) return dev_alloc(bytes, device);  // A/B: cudaMalloc / synchronising cudaFree
    auto b = std::make_shared<DevBuf>();
    b->device = device;
    b->bytes = bytes;
    CK(cudaMallocAsync(&b->ptr, bytes ? bytes : 16, order->copy));
    b->order = order;
    return b;
}

// Pool of pinned host blocks (result columns) and of device blocks (device-resident results).
struct BlockPool {
    bool pinned;  // true: cudaMallocHost, false: cudaMalloc
    int device;
    std::mutex mu;
    std::multimap<size_t, void *> free_blocks;
    BlockPool(bool p, int d) : pinned(p), device(d) {}
    ~BlockPool() {
        int cur;
        cudaGetDevice(&cur);
        cudaSetDevice(device);
        for (auto &kv : free_blocks) pinned ? cudaFreeHost(kv.second) : cudaFree(kv.second);
        cudaSetDevice(cur);
    }
    static size_t size_class(size_t b) {
        size_t s = 4096;
        while (s < b) s <<= 1;
        return s;
    }
    std::pair<void *, size_t> get(size_t bytes) {
        const size_t sc = size_class(bytes);
        {
            std::lock_guard<std::mutex> g(mu);
            auto it = free_blocks.find(sc);
            if (it != free_blocks.end()) {
                void *p = it->second;
                free_blocks.erase(it);
                return {p, sc};
            }
        }
        void *p = nullptr;
        if (pinned) CK(cudaMallocHost(&p, sc));
        else CK(cudaMalloc(&p, sc));
        return {p, sc};
    }
    void put(void *p, size_t sc) {
        std::lock_guard<std::mutex> g(mu);
        free_blocks.emplace(sc, p);
    }
};

// ============================================================ results ===
struct ResultImpl : h2tap_result {
    std::vector<std::string> name_store;
    std::vector<const char *> name_ptrs;
    std::vector<uint32_t> type_store;
    std::vector<const void *> col_ptrs;
    std::vector<std::vector<uint8_t>> null_store;
    std::vector<const uint8_t *> null_ptrs;
    std::vector<std::string> kname_store;
    std::vector<const char *> kname_ptrs;
    std::vector<double> kms;
    std::vector<std::pair<void *, size_t>> blocks;
    std::shared_ptr<BlockPool> pool;
    ~ResultImpl() {
        if (pool)
            for (auto &b : blocks) pool->put(b.first, b.second);
    }
    void finish() {
        name_ptrs.clear();
        for (auto &s : name_store) name_ptrs.push_back(s.c_str());
        null_ptrs.clear();
        for (auto &v : null_store) null_ptrs.push_back(v.empty() ? nullptr : v.data());
        kname_ptrs.clear();
        for (auto &s : kname_store) kname_ptrs.push_back(s.c_str());
        names = name_ptrs.data();
        types = type_store.data();
        cols = col_ptrs.data();
        nulls = null_ptrs.data();
        ncols = (uint32_t)name_store.size();
        nkernels = (uint32_t)kname_store.size();
        kernel_names = kname_ptrs.data();
        kernel_ms = kms.data();
    }
};

// =========================================================== snapshot ===
constexpr int kStatCols = 4;  // zone-map slots per table: the (w, d, id) key columns 0..2, and
// slot 3 = a payload column of the Q18 result rows (orders: o_ol_cnt; customer: c_last) whose
// range sizes the ORDER BY's carry records; item: i_id only
inline int stat_cols(int table) { return table == H2TAP_T_ITEM ? 1 : kStatCols; }
inline int stat_col(int table, int slot) {  // column id of a zone-map slot, -1 if none
    if (slot < 3) return slot;
    if (table == H2TAP_T_ORDERS) return H2TAP_O_OL_CNT;
    if (table == H2TAP_T_CUSTOMER) return H2TAP_C_LAST;
    return -1;
}
// one 64-bit zone-map column per table: orders.o_entry_d, whose range sizes the ORDER BY's entry
// field (the Q18 plan then reads no o_entry_d column)
inline int stat64_col(int table) { return table == H2TAP_T_ORDERS ? (int)H2TAP_O_ENTRY_D : -1; }
inline int stat_slot(int table, uint32_t column) {  // zone-map slot of a column, -1 if none
    for (int s = 0; s < stat_cols(table); ++s)
        if (stat_col(table, s) == (int)column) return s;
    return -1;
}
struct View {  // immutable snapshot at one epoch (the paper's shallow-copied top container)
    uint64_t epoch = 0;
    uint64_t n[kTables] = {};
    void *col[kTables][kMaxCols] = {};
    DevBufP keep[kTables][kMaxCols];
    // column statistics of the visible rows (zone map): valid once the view is published
    int smin[kTables][kStatCols], smax[kTables][kStatCols];
    bool has_stats[kTables] = {};
    long long smin64[kTables] = {}, smax64[kTables] = {};  // stat64_col(t)
    bool has_stats64[kTables] = {};
    // NEXT-4: columns read zero-copy from the caller's pinned host memory (col[][] is then the
    // mapped device address; nothing is kept alive by the view: the caller owns the memory)
    bool host[kTables][kMaxCols] = {};
    bool any_host(int t, std::initializer_list<int> cs) const {
        for (int c : cs) if (host[t][c]) return true;
        return false;
    }
};
using ViewP = std::shared_ptr<const View>;

struct ColState {
    // cur: the latest accepted version. alt: the shadow (an earlier version, or a spare for full
    // reloads); when alt_valid, alt equals cur on rows [0, alt_synced) except on the pages whose
    // bit is set in `bits` (copy-on-write of in-place updates, store_kernels.cu); bits_next is
    // the map the next update fills
    DevBufP cur, alt, bits, bits_next;
    const char *host_base = nullptr;  // NEXT-4 zero-copy column: mapped address of row 0
    uint64_t cap_rows = 0;
    bool alt_valid = false;
    uint64_t alt_synced = 0;
};
struct TableState {
    bool present = false;
    bool zero_copy = false; // NEXT-4: the table's columns live in the caller's pinned host memory
    uint32_t colmask = 0;   // which column ids this table carries (fixed at first load)
    uint64_t loaded = 0;    // rows copied or in flight
    ColState col[kMaxCols];
};

struct Pending {
    uint64_t epoch;
    std::shared_ptr<View> view;   // becomes visible (const) at publish
    cudaEvent_t done;
    cudaEvent_t t0, t1, t2, t3;   // timing (copy stream): begin, loads done, update arrays
                                  // uploaded, updates applied
    bool loaded[kTables], full[kTables], updated[kTables];
    bool stats64_ok[kTables];     // the 64-bit zone map covers every row this refresh loaded
    int *stats_host;              // pinned [kTables][kStatCols][2] delta min/max, then the u64
                                  // count of pages copied into shadows (kStatBytes offset)
    std::pair<void *, size_t> stats_block;
    uint64_t rows_appended, rows_updated, full_copies;
};
constexpr size_t kStatBytes = sizeof(int) * kTables * kStatCols * 2;  // multiple of 8
constexpr size_t kStat64Off = kStatBytes + 8;                          // after the page count
constexpr size_t kStatTotal = kStat64Off + 16 * kTables;               // + [kTables][2] int64

struct Staging {  // pinned ring for pageable host buffers
    static constexpr size_t kChunk = 32u << 20;
    static constexpr int kSlots = 3;
    void *buf[kSlots] = {};
    cudaEvent_t ev[kSlots] = {};
    int next = 0;
};

// ============================================================ scratch ===
struct Arena {  // grow-only named device buffers, owned by the engine, stream-ordered on `owner`
    struct Buf { void *ptr = nullptr; size_t bytes = 0; };
    std::map<std::string, Buf> bufs;
    int device = 0;
    cudaStream_t owner = nullptr;  // every use of these buffers is on this stream
    void *get(const std::string &name, size_t bytes, bool zero = false, cudaStream_t st = nullptr) {
        Buf &b = bufs[name];
        if (!b.ptr || b.bytes < bytes) {
            // growth without any synchronisation: the old buffer is released after its last use
            // in stream order and the new one comes from the stream-ordered pool. (A cudaFree or
            // cudaDeviceSynchronize here would wait for every stream of the device — with N
            // logical ranks on one GPU, for another rank's kernel that waits for this rank's next
            // launch: a deadlock.)
            if (b.ptr) CK(cudaFreeAsync(b.ptr, owner));
            b = Buf{};
            CK(cudaMallocAsync(&b.ptr, bytes ? bytes : 16, owner));
            b.bytes = bytes;
            if (zero) CK(cudaMemsetAsync(b.ptr, 0, b.bytes, st ? st : owner));
        }
        return b.ptr;
    }
    void release() {
        for (auto &kv : bufs)
            if (kv.second.ptr) cudaFreeAsync(kv.second.ptr, owner);
        bufs.clear();
    }
};

struct Prof {  // per-kernel CUDA events on the compute stream
    bool on = false;
    cudaStream_t st = nullptr;
    std::vector<std::pair<std::string, std::pair<cudaEvent_t, cudaEvent_t>>> marks;
    std::vector<cudaEvent_t> pool;
    size_t used = 0;
    cudaEvent_t ev() {
        if (used == pool.size()) {
            cudaEvent_t e;
            CK(cudaEventCreate(&e));
            pool.push_back(e);
        }
        return pool[used++];
    }
    template <class F> void run(const char *name, F &&f) {
        if (!on) { f(); return; }
        cudaEvent_t a = ev(), b = ev();
        CK(cudaEventRecord(a, st));
        f();
        CK(cudaEventRecord(b, st));
        marks.push_back({name, {a, b}});
    }
    void reset(bool enable, cudaStream_t s) { on = enable; st = s; marks.clear(); used = 0; }
};

}  // namespace

// ============================================================= engine ===
struct h2tap_engine {
    int device = 0, rank = 0, world = 1, num_sms = 148;
    // Q6/Q1 stream their columns with TMA bulk copies (H2TAP_SCAN=ldg: register-prefetch kernels);
    // the Q18 probe keeps register prefetch at high occupancy — its dependent lookups and atomics
    // need more warps than a one-block-per-SM shared-memory ring leaves (H2TAP_PROBE=tma: ring)
    bool scan_tma = true, probe_tma = false;
    // ORDER BY: payload-carrying bucket sort (v2); H2TAP_ORDER=v1 selects the (key, row id) sort
    // with a random gather of the rows at emit (the A/B baseline)
    bool order_v1 = false;
    // zero-copy (host-resident) columns are streamed by the TMA-bulk kernels (cp.async.bulk reads
    // the mapped host memory: 0.92 of the PCIe copy rate vs 0.51 with LDG loads);
    // H2TAP_ZC_TMA=0 selects the LDG kernels
    bool zc_tma = true;
    int having_unroll = 2;  // H2TAP_HAVING_UNROLL (2 or 4): orders rows per thread in the HAVING pass
    bool shared_scan = true;  // H2TAP_SHARED_SCAN=0: separate Q6 and Q1 scans in a batch (A/B)
    bool full_pass = true;    // H2TAP_FULL_PASS=0: Q18's probe not in the batch's shared scan (A/B)
    // in-place updates copy only the dirty pages into the shadow (H2TAP_COW=full: always copy the
    // whole column — the A/B baseline of scripts/cow_bench.py)
    bool cow_full = false;
    // a7: this rank's peer segment and the mapped segments of the others
    struct Peer {
        char *seg = nullptr;            // own segment (cudaMalloc: IPC-exportable)
        size_t seg_bytes = 0;
        std::vector<void *> opened;     // IPC mappings of other processes' segments
        PeerArgs args{};
        unsigned int *err_host = nullptr;  // pinned, mapped: kernels' transport error bits
        bool connected = false, broken = false;
    } peer;
    cudaStream_t compute = nullptr, copy = nullptr;
    // H2TAP_Q18_STREAM=1: a batch's Q18 / Q3 run on this second compute stream, forked from the
    // batch start and joined before the batch's host synchronisation, so their latency-bound
    // kernels can overlap the bandwidth-bound scans of the other queries
    cudaStream_t side = nullptr;
    bool q18_side = false;
    uint64_t q18_runs = 0;  // Q18 / Q3 launches: parity of the clustered-index counters
    bool q1_side = true;   // H2TAP_Q1_SIDE=0: a shared-scan Q1's compact + emit stay on the compute stream
    cudaEvent_t ev_fork = nullptr, ev_join = nullptr;
    cudaStream_t reaper = nullptr;  // stream-ordered frees of snapshot buffers
    FreeOrder free_order;
    cudaEvent_t q_begin = nullptr, q_end = nullptr;
    cudaEvent_t b_begin = nullptr, b_end = nullptr;  // the last h2tap_run_queries batch on the device
    unsigned long long *pages_dev = nullptr;  // copy-on-write pages copied so far (device counter,
                                              // read by h2tap_get_store_stats only)
    float last_batch_ms = -1.f;
    uint64_t ch_runs = 0;  // parity of the Q12 / Q4 clustered-index counters

    std::mutex load_mu, query_mu, view_mu, pend_mu;
    TableState tables[kTables];
    ViewP published;
    ViewP accepted;               // latest accepted (published or pending) view
    std::atomic<uint64_t> last_epoch{0};
    bool any_epoch = false;
    std::deque<Pending> pending;
    Staging staging;

    h2tap_store_stats sstats{};  // under pend_mu
    Arena arena;       // query scratch (compute stream)
    Arena load_arena;  // refresh scratch (copy stream)
    Prof prof;
    std::shared_ptr<BlockPool> host_pool, dev_pool;
    long long *small_host = nullptr;  // pinned scratch for tiny D2H reads
};

namespace {

void publish_ready(h2tap_engine *e, bool wait) {
    std::lock_guard<std::mutex> g(e->pend_mu);
    while (!e->pending.empty()) {
        Pending &p = e->pending.front();
        if (wait) CK(cudaEventSynchronize(p.done));
        else {
            cudaError_t q = cudaEventQuery(p.done);
            if (q == cudaErrorNotReady) break;
            if (q != cudaSuccess) CK(q);
        }
        {  // statistics: delta of this refresh merged onto the previous epoch's (R17)
            View &v = *p.view;
            const View *prev = e->published.get();
            for (int t = 1; t < kTables; ++t) {
                const bool carry = !p.full[t] && prev && prev->has_stats[t];
                for (int c = 0; c < kStatCols; ++c) {
                    int mn = INT32_MAX, mx = INT32_MIN;
                    if (carry) { mn = prev->smin[t][c]; mx = prev->smax[t][c]; }
                    if (p.loaded[t] || p.updated[t]) {
                        mn = std::min(mn, p.stats_host[(t * kStatCols + c) * 2]);
                        mx = std::max(mx, p.stats_host[(t * kStatCols + c) * 2 + 1]);
                    }
                    v.smin[t][c] = mn;
                    v.smax[t][c] = mx;
                }
                v.has_stats[t] = p.loaded[t] || p.updated[t] || carry;
                if (stat64_col(t) >= 0) {
                    const long long *d64 = reinterpret_cast<const long long *>(
                        reinterpret_cast<const char *>(p.stats_host) + kStat64Off) + 2 * t;
                    const bool carry64 = !p.full[t] && prev && prev->has_stats64[t];
                    long long mn = INT64_MAX, mx = INT64_MIN;
                    if (carry64) { mn = prev->smin64[t]; mx = prev->smax64[t]; }
                    if (p.loaded[t] || p.updated[t]) { mn = std::min(mn, d64[0]); mx = std::max(mx, d64[1]); }
                    v.smin64[t] = mn;
                    v.smax64[t] = mx;
                    // a full reload: the delta covers the table; an append: the previous epoch's
                    // zone map plus the appended rows; updates widen it (launched per update)
                    v.has_stats64[t] = v.col[t][stat64_col(t)] && !v.host[t][stat64_col(t)] &&
                                       (p.full[t] ? p.stats64_ok[t] : carry64 && (!p.loaded[t] || p.stats64_ok[t]));
                }
            }
        }
        {
            h2tap_store_stats &S = e->sstats;
            S.published_epoch = p.epoch;
            S.refreshes += 1;
            S.rows_appended += p.rows_appended;
            S.rows_updated += p.rows_updated;
            S.cow_full_copies += p.full_copies;
            float a = 0, b = 0;
            CK(cudaEventElapsedTime(&a, p.t0, p.t1));
            CK(cudaEventElapsedTime(&b, p.t1, p.t2));
            S.last_load_ms = a;
            S.last_update_h2d_ms = b;
            CK(cudaEventElapsedTime(&b, p.t2, p.t3));
            S.last_update_ms = b;
        }
        {
            std::lock_guard<std::mutex> gv(e->view_mu);
            e->published = p.view;
        }
        for (cudaEvent_t ev : {p.done, p.t0, p.t1, p.t2, p.t3}) cudaEventDestroy(ev);
        e->host_pool->put(p.stats_block.first, p.stats_block.second);
        e->pending.pop_front();
    }
}

inline size_t round_up16(size_t b) { return (b + 15) & ~size_t(15); }

bool host_is_pinned(const void *p) {
    cudaPointerAttributes a;
    if (cudaPointerGetAttributes(&a, p) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    return a.type == cudaMemoryTypeHost;
}

// The next slot of the pinned staging ring, once its previous DMA has drained; staging_dma
// sends its first `bytes` to `dst` on the copy stream (the engine owns the bytes: no wait).
void *staging_slot(h2tap_engine *e) {
    Staging &S = e->staging;
    const int k = S.next;
    if (!S.buf[k]) {
        CK(cudaMallocHost(&S.buf[k], Staging::kChunk));
        CK(cudaEventCreateWithFlags(&S.ev[k], cudaEventDisableTiming));
    } else {
        CK(cudaEventSynchronize(S.ev[k]));
    }
    return S.buf[k];
}
void staging_dma(h2tap_engine *e, void *dst, size_t bytes) {
    Staging &S = e->staging;
    const int k = S.next;
    S.next = (S.next + 1) % Staging::kSlots;
    CK(cudaMemcpyAsync(dst, S.buf[k], bytes, cudaMemcpyHostToDevice, e->copy));
    CK(cudaEventRecord(S.ev[k], e->copy));
}
constexpr size_t kPackUpdateBytes = 256u << 10;

// Copy `bytes` from host `src` to device `dst` on the copy stream. Pinned sources are DMA'd
// directly (returns true: the caller must wait before returning); pageable ones go through the
// pinned staging ring (the engine owns those bytes once memcpy'd, so no wait is needed).
bool h2d(h2tap_engine *e, void *dst, const void *src, size_t bytes) {
    if (!bytes) return false;
    if (host_is_pinned(src)) {
        CK(cudaMemcpyAsync(dst, src, bytes, cudaMemcpyHostToDevice, e->copy));
        return true;
    }
    Staging &S = e->staging;
    for (size_t off = 0; off < bytes; off += Staging::kChunk) {
        const size_t len = std::min(Staging::kChunk, bytes - off);
        const int k = S.next;
        S.next = (S.next + 1) % Staging::kSlots;
        if (!S.buf[k]) {
            CK(cudaMallocHost(&S.buf[k], Staging::kChunk));
            CK(cudaEventCreateWithFlags(&S.ev[k], cudaEventDisableTiming));
        } else {
            CK(cudaEventSynchronize(S.ev[k]));  // previous DMA out of this slot has drained
        }
        std::memcpy(S.buf[k], static_cast<const char *>(src) + off, len);
        CK(cudaMemcpyAsync(static_cast<char *>(dst) + off, S.buf[k], len, cudaMemcpyHostToDevice,
                           e->copy));
        CK(cudaEventRecord(S.ev[k], e->copy));
    }
    return false;
}

// Zone-map deltas of a small refresh on the host, over the caller's own buffers (appended rows,
// update values): no device kernel and no device-to-host copy on the refresh's critical path — a
// kernel there waits for an SM slot under a saturating query loop, a DMA behind any large
// read-back of the caller's. Large deltas (full reloads) keep the device kernels.
constexpr uint64_t kHostStatsValues = 8u << 20;  // values scanned on the host at most per refresh
__attribute__((target_clones("avx2", "default")))
void host_minmax_i32(const int32_t *p, uint64_t n, int &mn, int &mx) {
    int a = INT32_MAX, b = INT32_MIN;
    for (uint64_t i = 0; i < n; ++i) { a = p[i] < a ? p[i] : a; b = p[i] > b ? p[i] : b; }
    mn = std::min(mn, a);
    mx = std::max(mx, b);
}
__attribute__((target_clones("avx2", "default")))
void host_minmax_i64(const int64_t *p, uint64_t n, long long &mn, long long &mx) {
    long long a = INT64_MAX, b = INT64_MIN;
    for (uint64_t i = 0; i < n; ++i) { a = p[i] < a ? p[i] : a; b = p[i] > b ? p[i] : b; }
    mn = std::min(mn, a);
    mx = std::max(mx, b);
}

h2tap_status load_impl(h2tap_engine *e, const h2tap_table *tables, uint32_t ntables,
                       const h2tap_update *updates, uint32_t nupdates, uint64_t epoch,
                       uint32_t flags) {
    std::lock_guard<std::mutex> g(e->load_mu);
    CK(cudaSetDevice(e->device));
    publish_ready(e, false);
    // back-pressure: at most 3 refreshes in flight (each may hold a snapshot copy), so a stream
    // of async loads reaches a steady state the memory pool can serve without growing
    // (polled: a query thread may publish — and release — the oldest refresh concurrently)
    for (;;) {
        size_t inflight;
        {
            std::lock_guard<std::mutex> gp(e->pend_mu);
            inflight = e->pending.size();
        }
        if (inflight < 3) break;
        std::this_thread::sleep_for(std::chrono::microseconds(50));
        publish_ready(e, false);
    }
    if (e->any_epoch && epoch <= e->last_epoch.load())
        return fail(H2TAP_ESTALE, "epoch %llu is not greater than the last accepted epoch %llu",
                    (unsigned long long)epoch, (unsigned long long)e->last_epoch.load());
    if (ntables && !tables) return fail(H2TAP_EINVAL, "tables is NULL");
    if (nupdates && !updates) return fail(H2TAP_EINVAL, "updates is NULL");
    // ---- validate everything before touching state
    bool seen[kTables] = {};
    for (uint32_t i = 0; i < ntables; ++i) {
        const h2tap_table &t = tables[i];
        if (t.table_id < 1 || t.table_id >= (uint32_t)kTables) return fail(H2TAP_EINVAL, "unknown table id %u", t.table_id);
        if (seen[t.table_id]) return fail(H2TAP_EINVAL, "table %u listed twice", t.table_id);
        seen[t.table_id] = true;
        if (t.ncols == 0 || !t.cols) return fail(H2TAP_EINVAL, "table %u has no columns", t.table_id);
        if (t.row_count < t.first_row) return fail(H2TAP_EINVAL, "table %u: row_count < first_row", t.table_id);
        if (t.row_count >= (1ull << 31)) return fail(H2TAP_EINVAL, "table %u: more than 2^31-1 rows", t.table_id);
        uint32_t mask = 0;
        for (uint32_t c = 0; c < t.ncols; ++c) {
            const h2tap_column &col = t.cols[c];
            if (col.column_id >= (uint32_t)kNcols[t.table_id])
                return fail(H2TAP_EINVAL, "table %u: unknown column id %u", t.table_id, col.column_id);
            if (col.type != kTypes[t.table_id][col.column_id])
                return fail(H2TAP_EINVAL, "table %u column %u: type %u, schema type %u", t.table_id,
                            col.column_id, col.type, kTypes[t.table_id][col.column_id]);
            if (mask & (1u << col.column_id))
                return fail(H2TAP_EINVAL, "table %u: column %u listed twice", t.table_id, col.column_id);
            if (!col.host_data && t.row_count > t.first_row)
                return fail(H2TAP_EINVAL, "table %u column %u: host_data is NULL", t.table_id, col.column_id);
            mask |= 1u << col.column_id;
        }
        const TableState &ts = e->tables[t.table_id];
        const bool zc = flags & H2TAP_LOAD_ZERO_COPY;
        if (!(t.flags & H2TAP_FULL_RELOAD) && ts.present && ts.zero_copy != zc)
            return fail(H2TAP_ESHAPE, "table %u: switching between HBM and zero-copy needs a full reload", t.table_id);
        if (zc) {
            for (uint32_t c = 0; c < t.ncols; ++c) {
                const h2tap_column &col = t.cols[c];
                const size_t es = type_size(col.type);
                const char *base = static_cast<const char *>(col.host_data) - t.first_row * es;
                if (!col.host_data || (reinterpret_cast<uintptr_t>(base) & 15))
                    return fail(H2TAP_EINVAL, "table %u column %u: zero-copy data must be 16-byte aligned", t.table_id, col.column_id);
                cudaPointerAttributes a{};
                if (cudaPointerGetAttributes(&a, base) != cudaSuccess || a.type != cudaMemoryTypeHost || !a.devicePointer) {
                    cudaGetLastError();
                    return fail(H2TAP_EINVAL, "table %u column %u: zero-copy data must be pinned, mapped host memory",
                                t.table_id, col.column_id);
                }
                const ColState &cs = ts.col[col.column_id];
                if (!(t.flags & H2TAP_FULL_RELOAD) && ts.present && cs.host_base != static_cast<const char *>(a.devicePointer))
                    return fail(H2TAP_ESHAPE, "table %u column %u: a zero-copy append must extend the same host buffer",
                                t.table_id, col.column_id);
            }
        }
        if (t.flags & H2TAP_FULL_RELOAD) {
            if (t.first_row != 0) return fail(H2TAP_EINVAL, "table %u: full reload must start at row 0", t.table_id);
        } else {
            if (ts.present && mask != ts.colmask)
                return fail(H2TAP_ESHAPE, "table %u: append column set differs from the loaded set", t.table_id);
            if (t.first_row != ts.loaded)
                return fail(H2TAP_ESHAPE, "table %u: append starts at row %llu but %llu rows are loaded",
                            t.table_id, (unsigned long long)t.first_row, (unsigned long long)ts.loaded);
        }
    }
    {  // updates: target columns loaded at the new epoch, row ids inside its row count
        uint32_t listed[kTables] = {};
        for (uint32_t i = 0; i < nupdates; ++i) {
            const h2tap_update &u = updates[i];
            if (u.table_id < 1 || u.table_id >= (uint32_t)kTables) return fail(H2TAP_EINVAL, "update %u: unknown table id %u", i, u.table_id);
            if (u.column_id >= (uint32_t)kNcols[u.table_id])
                return fail(H2TAP_EINVAL, "update %u: unknown column id %u", i, u.column_id);
            if (u.type != kTypes[u.table_id][u.column_id])
                return fail(H2TAP_EINVAL, "update %u: type %u, schema type %u", i, u.type,
                            kTypes[u.table_id][u.column_id]);
            if (listed[u.table_id] & (1u << u.column_id))
                return fail(H2TAP_EINVAL, "update %u: table %u column %u listed twice", i, u.table_id, u.column_id);
            listed[u.table_id] |= 1u << u.column_id;
            if (u.n && (!u.row_ids || !u.values)) return fail(H2TAP_EINVAL, "update %u: NULL row_ids/values", i);
            uint32_t mask = 0;
            uint64_t rows = 0;
            if (seen[u.table_id]) {
                for (uint32_t k = 0; k < ntables; ++k)
                    if (tables[k].table_id == u.table_id) {
                        for (uint32_t c = 0; c < tables[k].ncols; ++c) mask |= 1u << tables[k].cols[c].column_id;
                        rows = tables[k].row_count;
                    }
            } else if (e->tables[u.table_id].present) {
                mask = e->tables[u.table_id].colmask;
                rows = e->accepted ? e->accepted->n[u.table_id] : 0;
            }
            if (!(mask & (1u << u.column_id)))
                return fail(H2TAP_EPLAN, "update %u: table %u column %u was never loaded", i, u.table_id, u.column_id);
            if ((seen[u.table_id] && (flags & H2TAP_LOAD_ZERO_COPY)) || (!seen[u.table_id] && e->tables[u.table_id].zero_copy))
                return fail(H2TAP_EPLAN, "update %u: table %u is zero-copy (host-resident): update the host rows instead", i, u.table_id);
            uint32_t mx = 0;
            for (uint64_t k = 0; k < u.n; ++k) mx = std::max(mx, u.row_ids[k]);
            if (u.n && mx >= rows)
                return fail(H2TAP_EINVAL, "update %u: row id %u outside the table's %llu rows", i, mx,
                            (unsigned long long)rows);
        }
    }
    // ---- copy and build the new view
    auto v = std::make_shared<View>();
    if (e->accepted) *v = *e->accepted;
    v->epoch = epoch;
    bool must_wait = false;
    Pending pend{};
    pend.epoch = epoch;
    pend.stats_block = e->host_pool->get(kStatTotal);
    pend.stats_host = static_cast<int *>(pend.stats_block.first);
    int *stats_dev = static_cast<int *>(e->load_arena.get("load.stats", kStatTotal));
    auto *stats64_dev = reinterpret_cast<long long *>(reinterpret_cast<char *>(stats_dev) + kStat64Off);
    unsigned long long *pages_dev = e->pages_dev;
    // zone maps on the host when the delta is small (see host_minmax_i32)
    bool host_stats;
    {
        uint64_t vals = 0;
        for (uint32_t i = 0; i < ntables; ++i) {
            const h2tap_table &t = tables[i];
            vals += (t.row_count - t.first_row) * (uint64_t)(stat_cols(t.table_id) + 1);
        }
        for (uint32_t i = 0; i < nupdates; ++i) vals += updates[i].n;
        host_stats = vals <= kHostStatsValues || (flags & H2TAP_LOAD_ZERO_COPY);
    }
    int *stats_h = pend.stats_host;
    long long *stats64_h = reinterpret_cast<long long *>(reinterpret_cast<char *>(stats_h) + kStat64Off);
    for (cudaEvent_t *ev : {&pend.t0, &pend.t1, &pend.t2, &pend.t3}) CK(cudaEventCreate(ev));
    CK(cudaEventRecord(pend.t0, e->copy));
    if (host_stats) {
        for (int i = 0; i < kTables * kStatCols; ++i) { stats_h[2 * i] = INT32_MAX; stats_h[2 * i + 1] = INT32_MIN; }
        for (int i = 0; i < kTables; ++i) { stats64_h[2 * i] = INT64_MAX; stats64_h[2 * i + 1] = INT64_MIN; }
    } else {
        launch_stats_init(stats_dev, kTables * kStatCols, e->copy);
        launch_stats_init64(stats64_dev, kTables, e->copy);
    }
    for (uint32_t i = 0; i < ntables; ++i) {
        const h2tap_table &t = tables[i];
        TableState &ts = e->tables[t.table_id];
        const bool full = t.flags & H2TAP_FULL_RELOAD;
        if (full) {  // a full reload may change the column set
            uint32_t mask = 0;
            for (uint32_t c = 0; c < t.ncols; ++c) mask |= 1u << t.cols[c].column_id;
            for (int c = 0; c < kNcols[t.table_id]; ++c)
                if (!(mask & (1u << c))) {
                    v->col[t.table_id][c] = nullptr;
                    v->host[t.table_id][c] = false;
                    v->keep[t.table_id][c].reset();
                    ts.col[c] = ColState{};
                }
            ts.colmask = mask;
        }
        const bool zc = flags & H2TAP_LOAD_ZERO_COPY;
        ts.zero_copy = zc;
        for (uint32_t c = 0; c < t.ncols; ++c) {
            const h2tap_column &col = t.cols[c];
            ColState &cs = ts.col[col.column_id];
            const size_t es = type_size(col.type);
            const uint64_t need = t.row_count + kPadRows;
            if (zc) {
                // NEXT-4: publish the caller's pinned rows [0, row_count) as they are — no copy;
                // kernels read them over PCIe through the mapped address
                cudaPointerAttributes a{};
                CK(cudaPointerGetAttributes(&a, static_cast<const char *>(col.host_data) - t.first_row * es));
                cs = ColState{};
                cs.host_base = static_cast<const char *>(a.devicePointer);
                v->col[t.table_id][col.column_id] = const_cast<char *>(cs.host_base);
                v->keep[t.table_id][col.column_id].reset();
                v->host[t.table_id][col.column_id] = true;
                continue;
            }
            v->host[t.table_id][col.column_id] = false;
            cs.host_base = nullptr;
            if (full) {
                // never overwrite a buffer a live view may read: reuse the spare only when no
                // view references it any more, else allocate
                DevBufP target;
                if (cs.alt && cs.alt.use_count() == 1 && cs.alt->bytes >= need * es) target = cs.alt;
                else target = dev_alloc_ordered(need * es + need * es / 8, e->device, &e->free_order);
                cs.alt = cs.cur;
                cs.alt_valid = false;
                cs.cur = target;
                cs.cap_rows = target->bytes / es;
            } else if (!cs.cur || need > cs.cap_rows) {
                // grow: new buffer, device-to-device copy of the visible prefix; the old buffer
                // stays alive for views that still reference it
                const uint64_t cap = std::max<uint64_t>(need, (cs.cap_rows * 3) / 2);
                DevBufP nb = dev_alloc_ordered(cap * es, e->device, &e->free_order);
                if (cs.cur && t.first_row)
                    CK(cudaMemcpyAsync(nb->ptr, cs.cur->ptr, t.first_row * es, cudaMemcpyDeviceToDevice, e->copy));
                cs.alt.reset();
                cs.alt_valid = false;
                cs.cur = nb;
                cs.cap_rows = cap;
            }
            must_wait |= h2d(e, static_cast<char *>(cs.cur->ptr) + t.first_row * es, col.host_data,
                             (t.row_count - t.first_row) * es);
            v->col[t.table_id][col.column_id] = cs.cur->ptr;
            v->keep[t.table_id][col.column_id] = cs.cur;
        }
        ts.present = true;
        if (!full) {
            uint32_t mask = 0;
            for (uint32_t c = 0; c < t.ncols; ++c) mask |= 1u << t.cols[c].column_id;
            ts.colmask = mask;
        }
        pend.rows_appended += t.row_count - t.first_row;
        ts.loaded = t.row_count;
        v->n[t.table_id] = t.row_count;
        pend.loaded[t.table_id] = true;
        pend.full[t.table_id] = full;
        // zone map of the appended rows' key columns: on the host from the caller's buffers (small
        // deltas), else on the copy stream after their H2D
        auto host_col = [&](int cid) -> const void * {
            for (uint32_t c = 0; c < t.ncols; ++c)
                if ((int)t.cols[c].column_id == cid) return t.cols[c].host_data;
            return nullptr;
        };
        const uint64_t nrows_delta = t.row_count - t.first_row;
        if (const int c64 = stat64_col(t.table_id); c64 >= 0 && v->col[t.table_id][c64] && !v->host[t.table_id][c64]) {
            if (host_stats) {
                if (const void *hp = host_col(c64))
                    host_minmax_i64(static_cast<const int64_t *>(hp), nrows_delta, stats64_h[2 * t.table_id],
                                    stats64_h[2 * t.table_id + 1]);
            } else {
                launch_minmax_i64(static_cast<const int64_t *>(v->col[t.table_id][c64]) + t.first_row,
                                  nrows_delta, stats64_dev + 2 * t.table_id, e->num_sms, e->copy);
            }
            pend.stats64_ok[t.table_id] = true;
        }
        for (int c = 0; c < stat_cols(t.table_id); ++c) {
            const int cid = stat_col(t.table_id, c);
            if (cid < 0 || !v->col[t.table_id][cid]) continue;
            if (host_stats) {
                if (const void *hp = host_col(cid))
                    host_minmax_i32(static_cast<const int32_t *>(hp), nrows_delta,
                                    stats_h[(t.table_id * kStatCols + c) * 2],
                                    stats_h[(t.table_id * kStatCols + c) * 2 + 1]);
            } else {
                launch_minmax_i32(static_cast<const int32_t *>(v->col[t.table_id][cid]) + t.first_row, nrows_delta,
                                  stats_dev + (t.table_id * kStatCols + c) * 2, e->num_sms, e->copy);
            }
        }
    }
    CK(cudaEventRecord(pend.t1, e->copy));
    // ---- in-place updates: upload every update's row ids and values first (one arena region;
    // the device-side phase below then runs without waiting on the host), then rebuild each
    // updated column in its shadow buffer (copy-on-write)
    std::vector<size_t> upd_off(nupdates + 1, 0);
    for (uint32_t i = 0; i < nupdates; ++i)
        upd_off[i + 1] = upd_off[i] + round_up16(updates[i].n * 4) + round_up16(updates[i].n * type_size(updates[i].type));
    char *upd_dev = nupdates ? static_cast<char *>(e->load_arena.get("upd.arrays", upd_off[nupdates] + 16)) : nullptr;
    if (nupdates && upd_off[nupdates] <= kPackUpdateBytes) {
        // small update sets are latency-bound: pack them into one staging slot, one DMA
        char *stage = static_cast<char *>(staging_slot(e));
        for (uint32_t i = 0; i < nupdates; ++i) {
            const h2tap_update &u = updates[i];
            if (u.n) std::memcpy(stage + upd_off[i], u.row_ids, u.n * 4);
            if (u.n) std::memcpy(stage + upd_off[i] + round_up16(u.n * 4), u.values, u.n * type_size(u.type));
        }
        staging_dma(e, upd_dev, upd_off[nupdates]);
    } else {
        for (uint32_t i = 0; i < nupdates; ++i) {
            const h2tap_update &u = updates[i];
            must_wait |= h2d(e, upd_dev + upd_off[i], u.row_ids, u.n * 4);
            must_wait |= h2d(e, upd_dev + upd_off[i] + round_up16(u.n * 4), u.values, u.n * type_size(u.type));
        }
    }
    CK(cudaEventRecord(pend.t2, e->copy));
    for (uint32_t i = 0; i < nupdates; ++i) {
        const h2tap_update &u = updates[i];
        ColState &cs = e->tables[u.table_id].col[u.column_id];
        const size_t es = type_size(u.type);
        const uint64_t n_rows = v->n[u.table_id];
        const uint64_t words = (cs.cap_rows + kCowPageRows * 32 - 1) / (kCowPageRows * 32);
        if (!cs.bits || cs.bits->bytes < words * 4) {
            cs.bits = dev_alloc_ordered(words * 4, e->device, &e->free_order);
            cs.bits_next = dev_alloc_ordered(words * 4, e->device, &e->free_order);
            cs.alt_valid = false;  // no record of where alt differs
        }
        uint32_t *next_bits = static_cast<uint32_t *>(cs.bits_next->ptr);
        const bool reuse = cs.alt && cs.alt.use_count() == 1 && cs.alt->bytes >= cs.cap_rows * es;
        if (reuse && cs.alt_valid && !e->cow_full) {
            launch_cow_catchup(cs.alt->ptr, cs.cur->ptr, (uint32_t)es, static_cast<const uint32_t *>(cs.bits->ptr),
                               next_bits, words, cs.alt_synced, n_rows, pages_dev, e->num_sms, e->copy);
        } else {
            if (!reuse) cs.alt = dev_alloc_ordered(cs.cap_rows * es, e->device, &e->free_order);
            if (n_rows) CK(cudaMemcpyAsync(cs.alt->ptr, cs.cur->ptr, n_rows * es, cudaMemcpyDeviceToDevice, e->copy));
            CK(cudaMemsetAsync(next_bits, 0, words * 4, e->copy));
            pend.full_copies += 1;
        }
        if (u.n) {
            const auto *rows_d = reinterpret_cast<const uint32_t *>(upd_dev + upd_off[i]);
            const void *vals_d = upd_dev + upd_off[i] + round_up16(u.n * 4);
            launch_apply_updates(cs.alt->ptr, (uint32_t)es, next_bits, rows_d, vals_d, u.n, e->num_sms, e->copy);
            if ((int)u.column_id == stat64_col(u.table_id)) {  // 64-bit zone map: widen
                if (host_stats)
                    host_minmax_i64(static_cast<const int64_t *>(u.values), u.n, stats64_h[2 * u.table_id],
                                    stats64_h[2 * u.table_id + 1]);
                else
                    launch_minmax_i64(static_cast<const int64_t *>(vals_d), u.n, stats64_dev + 2 * u.table_id,
                                      e->num_sms, e->copy);
            }
            if (const int sl = stat_slot(u.table_id, u.column_id); sl >= 0) {  // zone map: widen
                if (host_stats)
                    host_minmax_i32(static_cast<const int32_t *>(u.values), u.n,
                                    stats_h[(u.table_id * kStatCols + sl) * 2],
                                    stats_h[(u.table_id * kStatCols + sl) * 2 + 1]);
                else
                    launch_minmax_i32(static_cast<const int32_t *>(vals_d), u.n,
                                      stats_dev + (u.table_id * kStatCols + sl) * 2, e->num_sms, e->copy);
            }
        }
        std::swap(cs.cur, cs.alt);
        std::swap(cs.bits, cs.bits_next);
        cs.alt_valid = true;
        cs.alt_synced = n_rows;
        v->col[u.table_id][u.column_id] = cs.cur->ptr;
        v->keep[u.table_id][u.column_id] = cs.cur;
        pend.updated[u.table_id] = true;
        pend.rows_updated += u.n;
    }
    CK(cudaEventRecord(pend.t3, e->copy));
    CK(cudaGetLastError());
    // device statistics (large deltas): one DMA, not a kernel's stores to the mapped block (under a
    // saturating query loop a kernel waits for an SM slot — config C5: refresh 4.8 vs 8.1 ms, lag
    // p99 138 vs 622 ms)
    if (!host_stats) CK(cudaMemcpyAsync(pend.stats_host, stats_dev, kStatTotal, cudaMemcpyDeviceToHost, e->copy));
    CK(cudaEventCreateWithFlags(&pend.done, cudaEventDisableTiming));
    CK(cudaEventRecord(pend.done, e->copy));
    pend.view = v;
    e->accepted = v;
    e->last_epoch = epoch;
    e->any_epoch = true;
    {
        std::lock_guard<std::mutex> gp(e->pend_mu);
        e->pending.push_back(pend);
    }
    // pinned caller buffers are read by the DMA after we return: wait, unless they are lent
    if ((must_wait && !(flags & H2TAP_LOAD_BORROW)) || !(flags & H2TAP_LOAD_ASYNC)) publish_ready(e, true);
    return H2TAP_OK;
}

// ------------------------------------------------------------ plans --
struct Col { const void *p; };
template <class T> const T *colp(const View &v, int t, int c) {
    return static_cast<const T *>(v.col[t][c]);
}

void need_cols(const View &v, int t, std::initializer_list<int> cs, const char *plan) {
    for (int c : cs)
        if (!v.col[t][c] && v.n[t])
            raise(H2TAP_EPLAN, "%s needs column %d of table %d, which was never loaded", plan, c, t);
}

ResultImpl *new_result(h2tap_engine *e, const View &v, bool dev) {
    auto *r = new ResultImpl();
    std::memset(static_cast<h2tap_result *>(r), 0, sizeof(h2tap_result));
    r->epoch = v.epoch;
    r->rows_scanned = v.n[H2TAP_T_ORDER_LINE];
    r->on_device = dev ? 1 : 0;
    r->pool = dev ? e->dev_pool : e->host_pool;
    return r;
}

// Allocate result column storage (pinned host or device) of `bytes`.
void *result_block(ResultImpl *r, size_t bytes) {
    auto b = r->pool->get(bytes ? bytes : 8);
    r->blocks.push_back(b);
    return b.first;
}

void add_col(ResultImpl *r, const char *name, uint32_t type, const void *p) {
    r->name_store.emplace_back(name);
    r->type_store.push_back(type);
    r->col_ptrs.push_back(p);
    r->null_store.emplace_back();
}

void sync_compute(h2tap_engine *e) { CK(cudaStreamSynchronize(e->compute)); }

// ---- query execution: launch (asynchronous) + finish (after one stream synchronisation) ------
// A query's kernels are enqueued by launch(); finish() runs after the host has synchronised
// with the compute stream, reads the few scalars it needs (counts, flags), and completes the
// result (host copies when requested). h2tap_run_queries launches a whole batch, synchronises
// once and finishes every query, so the GPU runs the batch back to back (the paper's "several
// OLAP queries share a snapshot", L555-559). With world > 1 a plan synchronises inside launch
// where a collective needs host-side sizes.
struct QueryCtx {
    uint32_t plan = 0, flags = 0;
    int64_t p[4] = {};
    std::unique_ptr<ResultImpl> r;
    cudaEvent_t begin = nullptr, end = nullptr;
    uint64_t launches0 = 0, launches = 0;
    std::pair<void *, size_t> small{};     // pinned scalars read back at finish
    void *small_dev = nullptr;             // its mapped device address: kernels write it directly
    std::chrono::steady_clock::time_point t0;
    size_t mark0 = 0, mark1 = 0;           // this query's profile marks [mark0, mark1)
    // Q1
    Q1Scratch q1{};
    std::vector<std::pair<void *, size_t>> dev_blocks;  // per-query device output blocks
    // Q18
    Q18Scratch q18{};
    Q18Plan *plan_dev = nullptr;
    Q18Zone zone{};                         // ORDER BY field bounds from the zone maps
    int64_t shared_cutoff = 0;              // the paired Q1's cutoff (shared_scan == 1)
    int shared_scan = 0;                    // 1: this Q6 runs the batch's shared Q6+Q1 scan;
                                            // 2: this Q1's scan was done by it
    QueryCtx *full18 = nullptr;             // (Q6, shared_scan == 1) the batch's Q18 whose probe
                                            // runs in the same pass (the full pass, §4.5)
    bool probe_done = false;                // (Q18) init, build and probe ran in the full pass
    const Q18Row *rows = nullptr;
    const long long *amt = nullptr;
    const unsigned int *perm = nullptr;
    const unsigned long long *perm_keys = nullptr;
    SortPairs sp{};
    Q18Cols out{};                          // device output columns (sorted)
    uint64_t n_max = 0;
    unsigned int *tie_dev = nullptr;
    // Q18 v3 (HAVING builds the carry records) and the batch's snapshot
    bool v3 = false;
    const View *view = nullptr;
    // world > 1: distributed ORDER BY
    bool dist = false;
    uint64_t dist_out_cap = 0;              // rows the output columns hold
    unsigned int *recv_off = nullptr;       // this rank's bucket offsets in its heap
    BucketSort bs{};
    long long *q6_out = nullptr;           // Q6 result {revenue, count} on the device
    // NEXT-2: Q14 / Q12 / Q4
    Q14Scratch q14{};
    SmallGroups sg{};
    unsigned int *err = nullptr;
};

void *dev_block(h2tap_engine *e, QueryCtx &q, size_t bytes) {
    auto b = e->dev_pool->get(bytes ? bytes : 8);
    q.dev_blocks.push_back(b);
    return b.first;
}
void release_dev_blocks(h2tap_engine *e, QueryCtx &q) {
    for (auto &b : q.dev_blocks) e->dev_pool->put(b.first, b.second);
    q.dev_blocks.clear();
}
// Device output blocks become the result's columns (ownership moves to the result).
void give_blocks_to_result(QueryCtx &q) {
    for (auto &b : q.dev_blocks) q.r->blocks.push_back(b);
    q.dev_blocks.clear();
}

// ---- Q6 (a2 + a7)
void q1_tables(h2tap_engine *e, Q1Scratch &s);

void q18_pre_probe(h2tap_engine *e, const View &v, QueryCtx &q);

void launch_q6_plan(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int T = H2TAP_T_ORDER_LINE;
    need_cols(v, T, {H2TAP_OL_DELIVERY_D, H2TAP_OL_QUANTITY, H2TAP_OL_AMOUNT}, "Q6");
    Q6Scratch s;
    const int mb = q6_max_blocks(e->num_sms);
    s.block_part = static_cast<long long *>(e->arena.get("q6.part", sizeof(long long) * 2 * mb));
    s.done_counter = static_cast<unsigned int *>(e->arena.get("q6.counter", 64, true, e->compute));
    // world == 1: the kernel writes {revenue, count} straight into the result's device block and
    // into the mapped pinned scalars (no copies); world > 1: the rank's partial, then the peer
    // allreduce writes both (a7)
    s.out = e->world > 1 ? static_cast<long long *>(e->arena.get("q6.out", 64))
                         : static_cast<long long *>(dev_block(e, q, 16));
    s.host_out = e->world > 1 ? nullptr : static_cast<long long *>(q.small_dev);
    q.q6_out = s.out;
    if (q.shared_scan == 1 && q.full18) {  // one pass for this Q6, the batch's Q1 and Q18's probe
        Q1Scratch t{};
        q1_tables(e, t);
        QueryCtx &q18 = *q.full18;
        q18_pre_probe(e, v, q18);  // the join indexes (and zeroed accumulators) the probe needs
        e->prof.run("q6118_full_pass", [&] {
            launch_q6118_tma(colp<int32_t>(v, T, H2TAP_OL_NUMBER), colp<int64_t>(v, T, H2TAP_OL_DELIVERY_D),
                             colp<int32_t>(v, T, H2TAP_OL_QUANTITY), colp<int64_t>(v, T, H2TAP_OL_AMOUNT),
                             colp<int32_t>(v, T, H2TAP_OL_W_ID), colp<int32_t>(v, T, H2TAP_OL_D_ID),
                             colp<int32_t>(v, T, H2TAP_OL_O_ID), v.n[T], q.shared_cutoff, t, q.p[0], q.p[1],
                             q.p[2], q.p[3], s, q18.q18, e->num_sms, e->compute);
            CK(cudaGetLastError());
        });
        q18.probe_done = true;
    } else if (q.shared_scan == 1) {  // one pass for this Q6 and the batch's Q1 (its tables filled here)
        Q1Scratch t{};
        q1_tables(e, t);
        e->prof.run("q61_shared_scan", [&] {
            launch_q61_tma(colp<int32_t>(v, T, H2TAP_OL_NUMBER), colp<int64_t>(v, T, H2TAP_OL_DELIVERY_D),
                           colp<int32_t>(v, T, H2TAP_OL_QUANTITY), colp<int64_t>(v, T, H2TAP_OL_AMOUNT), v.n[T],
                           q.shared_cutoff, t, q.p[0], q.p[1], q.p[2], q.p[3], s, e->num_sms, e->compute);
            CK(cudaGetLastError());
        });
    } else
    e->prof.run("q6_scan_filter_sum", [&] {
        (e->scan_tma && (e->zc_tma || !v.any_host(T, {H2TAP_OL_DELIVERY_D, H2TAP_OL_QUANTITY, H2TAP_OL_AMOUNT})) ? launch_q6_tma : launch_q6)(
            colp<int64_t>(v, T, H2TAP_OL_DELIVERY_D), colp<int32_t>(v, T, H2TAP_OL_QUANTITY),
            colp<int64_t>(v, T, H2TAP_OL_AMOUNT), v.n[T], q.p[0], q.p[1], q.p[2], q.p[3], s,
            e->num_sms, e->compute);
        CK(cudaGetLastError());
    });
    if (e->world > 1) {
        auto *dst = static_cast<long long *>(dev_block(e, q, 16));
        e->prof.run("q6_peer_allreduce", [&] {
            launch_peer_allreduce_i64(e->peer.args, s.out, 2, dst, static_cast<long long *>(q.small_dev),
                                      e->compute);
        });
        q.q6_out = dst;
    }
}

void finish_q6(h2tap_engine *e, QueryCtx &q) {
    ResultImpl *r = q.r.get();
    const long long *sm = static_cast<const long long *>(q.small.first);
    const long long rev = sm[0], cnt = sm[1];
    r->nrows = 1;
    long long *blk;
    if (r->on_device) {  // the scan (one GPU) or the allreduce wrote the result column already
        blk = q.q6_out;
        give_blocks_to_result(q);
    } else {
        blk = static_cast<long long *>(result_block(r, 16));
        if (r->on_device) {
            CK(cudaMemcpyAsync(blk, sm, 16, cudaMemcpyHostToDevice, e->compute));
            sync_compute(e);
        }
        else { blk[0] = rev; blk[1] = cnt; }
        release_dev_blocks(e, q);
    }
    add_col(r, "revenue", H2TAP_I64, blk);
    r->null_store.back().assign(1, cnt == 0 ? 1 : 0);  // SUM over no rows IS NULL (R8)
    add_col(r, "count_rows", H2TAP_I64, blk + 1);
}

// ---- Q1 (a3 + a7 + a8)
constexpr size_t kQ1MaxGroups = kQ1GlobalSlots + kQ1Dense;

// Q1's aggregation tables (named arena buffers; they self-clean in q1_compact after each use).
void q1_tables(h2tap_engine *e, Q1Scratch &s) {
    const bool fresh = !e->arena.bufs.count("q1.gtag");
    s.dense = static_cast<unsigned long long *>(e->arena.get("q1.dense", 8 * kQ1Dense * 3));
    s.gtag = static_cast<unsigned long long *>(e->arena.get("q1.gtag", 8ull * kQ1GlobalSlots));
    s.gacc = static_cast<unsigned long long *>(e->arena.get("q1.gacc", 24ull * kQ1GlobalSlots));
    s.flags = static_cast<unsigned int *>(e->arena.get("q1.flags", 64));
    s.groups = static_cast<Q1Group *>(e->arena.get("q1.groups", sizeof(Q1Group) * kQ1MaxGroups));
    s.ngroups = static_cast<unsigned long long *>(e->arena.get("q1.ngroups", 64));
    if (fresh) launch_q1_reset(s, e->compute);
}

// The columns a Q6 / Q1 scan reads are all in HBM (or the zero-copy TMA path is enabled).
bool scan_tma_ok(h2tap_engine *e, const View &v, std::initializer_list<int> cols) {
    return e->scan_tma && (e->zc_tma || !v.any_host(H2TAP_T_ORDER_LINE, cols));
}

void launch_q1_plan(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int T = H2TAP_T_ORDER_LINE;
    need_cols(v, T, {H2TAP_OL_NUMBER, H2TAP_OL_DELIVERY_D, H2TAP_OL_QUANTITY, H2TAP_OL_AMOUNT}, "Q1");
    Q1Scratch &s = q.q1;
    q1_tables(e, s);
    // outputs go straight into per-query device blocks (they become the result's columns)
    s.o_key = static_cast<int32_t *>(dev_block(e, q, 4 * kQ1MaxGroups));
    s.o_qty = static_cast<long long *>(dev_block(e, q, 8 * kQ1MaxGroups));
    s.o_amt = static_cast<long long *>(dev_block(e, q, 8 * kQ1MaxGroups));
    s.o_avg_qty = static_cast<double *>(dev_block(e, q, 8 * kQ1MaxGroups));
    s.o_avg_amt = static_cast<double *>(dev_block(e, q, 8 * kQ1MaxGroups));
    s.o_cnt = static_cast<long long *>(dev_block(e, q, 8 * kQ1MaxGroups));
    if (q.shared_scan != 2)
    e->prof.run("q1_scan_filter_groupby", [&] {
        (e->scan_tma && (e->zc_tma || !v.any_host(T, {H2TAP_OL_NUMBER, H2TAP_OL_DELIVERY_D, H2TAP_OL_QUANTITY, H2TAP_OL_AMOUNT})) ? launch_q1_tma : launch_q1)(colp<int32_t>(v, T, H2TAP_OL_NUMBER), colp<int64_t>(v, T, H2TAP_OL_DELIVERY_D),
                  colp<int32_t>(v, T, H2TAP_OL_QUANTITY), colp<int64_t>(v, T, H2TAP_OL_AMOUNT), v.n[T],
                  q.p[0], s, e->num_sms, e->compute);
        CK(cudaGetLastError());
    });
    e->prof.run("q1_compact", [&] { launch_q1_compact(s, e->compute); });
    if (e->world > 1) {  // a7: every rank's group list into every rank's mailbox, folded, re-compacted
        e->prof.run("q1_peer_push", [&] {
            launch_peer_push(e->peer.args, s.groups, s.ngroups, 0, sizeof(Q1Group), e->num_sms, e->compute);
        });
        e->prof.run("q1_peer_merge", [&] {
            launch_peer_wait(e->peer.args, e->compute);
            launch_q1_peer_merge(e->peer.args, s, e->num_sms, e->compute);
            launch_q1_compact(s, e->compute);
        });
    }
    s.host_small = static_cast<unsigned long long *>(q.small_dev);  // emit writes {ngroups, flags}
    e->prof.run("q1_emit", [&] { launch_q1_emit(s, kQ1MaxGroups, e->compute); });
}

void finish_q1(h2tap_engine *e, QueryCtx &q) {
    ResultImpl *r = q.r.get();
    const auto *sm = static_cast<const unsigned long long *>(q.small.first);
    const uint64_t ng = sm[0];
    if (static_cast<const unsigned int *>(q.small.first)[2] & 1) {
        CK(cudaMemsetAsync(q.q1.flags, 0, 4, e->compute));
        raise(H2TAP_ENOMEM, "Q1: more than %d distinct ol_number groups", kQ1GlobalSlots);
    }
    r->nrows = ng;
    const Q1Scratch &s = q.q1;
    struct { const char *name; uint32_t type; const void *src; size_t es; } cols[] = {
        {"ol_number", H2TAP_I32, s.o_key, 4}, {"sum_qty", H2TAP_I64, s.o_qty, 8},
        {"sum_amount", H2TAP_I64, s.o_amt, 8}, {"avg_qty", H2TAP_F64, s.o_avg_qty, 8},
        {"avg_amount", H2TAP_F64, s.o_avg_amt, 8}, {"count_order", H2TAP_I64, s.o_cnt, 8}};
    if (r->on_device) {
        for (auto &c : cols) add_col(r, c.name, c.type, c.src);
        give_blocks_to_result(q);
        return;
    }
    for (auto &c : cols) {
        void *dst = result_block(r, ng * c.es);
        if (ng) CK(cudaMemcpyAsync(dst, c.src, ng * c.es, cudaMemcpyDeviceToHost, e->compute));
        add_col(r, c.name, c.type, dst);
    }
    sync_compute(e);
    release_dev_blocks(e, q);
}

// ---- Q18 (a4 + a5 + a6 + a7 + a8)
int bitwidth(unsigned long long x) { return x ? 64 - __builtin_clzll(x) : 0; }

uint64_t pow2_at_least(uint64_t x) {
    uint64_t c = 16;
    while (c < x) c <<= 1;
    return c;
}

// Planner for a join index on (w, d, id) = columns 0..2 of `table`: a perfect
// hash over the key box of the build side when the box holds <= 4 slots per row, else an
// open-addressing hash table. Statistics come from the published snapshot (zone maps).
JoinIndex plan_index(h2tap_engine *e, const View &v, int table, bool force_hash, const char *name) {
    JoinIndex j{};
    const uint64_t n = v.n[table];
    if (!force_hash && n && v.has_stats[table]) {
        const long long nw = (long long)v.smax[table][0] - v.smin[table][0] + 1;
        const long long nd = (long long)v.smax[table][1] - v.smin[table][1] + 1;
        const long long nk = (long long)v.smax[table][2] - v.smin[table][2] + 1;
        if (nw > 0 && nd > 0 && nk > 0) {
            const double range = (double)nw * (double)nd * (double)nk;
            if (range <= 4.0 * (double)n + 4096.0 && range < 4.0e9) {
                j.dense = 1;
                j.w0 = v.smin[table][0]; j.d0 = v.smin[table][1]; j.k0 = v.smin[table][2];
                j.nw = (unsigned)nw; j.nd = (unsigned)nd; j.nk = (unsigned)nk;
                j.range = (unsigned long long)nw * (unsigned long long)nd * (unsigned long long)nk;
                j.slots = static_cast<unsigned int *>(
                    e->arena.get(std::string(name) + ".dense", 4 * (j.range + 4)));
                return j;
            }
        }
    }
    const uint64_t cap = pow2_at_least(2 * n);
    j.dense = 0;
    j.mask = cap - 1;
    j.ht = static_cast<HtSlot *>(e->arena.get(std::string(name) + ".ht", sizeof(HtSlot) * cap));
    return j;
}

// {nout, err, tie} written by q18_publish (one GPU) or {n_mine, err, tie, -, row0, n_total} by the
// distributed publish (world > 1), into mapped pinned memory
struct Q18Small { unsigned long long nout; unsigned int err, tie; Q18Stats st; unsigned long long row0, n_total;
                  unsigned int clustered; };
const char *const kQ18Names[8] = {"c_last", "c_id", "o_id", "o_entry_d", "o_ol_cnt", "amount_sum", "o_w_id", "o_d_id"};
const uint32_t kQ18Types[8] = {H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I64, H2TAP_I32, H2TAP_I64, H2TAP_I32, H2TAP_I32};
const char *const kQ3Names[5] = {"ol_o_id", "ol_w_id", "ol_d_id", "revenue", "o_entry_d"};
const uint32_t kQ3Types[5] = {H2TAP_I32, H2TAP_I32, H2TAP_I32, H2TAP_I64, H2TAP_I64};

struct ProfMarks : PhaseMarks {  // one profile mark per phase kernel (H2TAP_QUERY_PROFILE)
    Prof &p;
    cudaEvent_t a = nullptr;
    std::string name;
    explicit ProfMarks(Prof &pr) : p(pr) {}
    void begin(const char *nm) override {
        if (!p.on) return;
        name = nm;
        a = p.ev();
        CK(cudaEventRecord(a, p.st));
    }
    void end() override {
        if (!p.on) return;
        cudaEvent_t b = p.ev();
        CK(cudaEventRecord(b, p.st));
        p.marks.push_back({name, {a, b}});
    }
};

void q18_alloc_out(h2tap_engine *e, QueryCtx &q, uint64_t rows) {
    Q18Cols &d = q.out;
    d.c_last = static_cast<int32_t *>(dev_block(e, q, 4 * rows));
    d.c_id = static_cast<int32_t *>(dev_block(e, q, 4 * rows));
    d.o_id = static_cast<int32_t *>(dev_block(e, q, 4 * rows));
    d.o_entry_d = static_cast<int64_t *>(dev_block(e, q, 8 * rows));
    d.o_ol_cnt = static_cast<int32_t *>(dev_block(e, q, 4 * rows));
    d.amount_sum = static_cast<int64_t *>(dev_block(e, q, 8 * rows));
    d.o_w_id = static_cast<int32_t *>(dev_block(e, q, 4 * rows));
    d.o_d_id = static_cast<int32_t *>(dev_block(e, q, 4 * rows));
}

void q18_sort_and_emit(h2tap_engine *e, QueryCtx &q) {
    // a8: ORDER BY amount_sum DESC, o_entry_d, o_w_id, o_d_id, o_id, entirely on the device:
    // plan (field widths from the stats) -> 64-bit prefix keys + bucket histogram -> bucket
    // scatter -> per-bucket sort + tie-fix + emit into the output columns. Grids are sized for
    // n_max (the orders rows); the actual row count is read on the device.
    const uint64_t n_max = std::max<uint64_t>(q.n_max, 1);
    int bb = 1;
    while (bb < kBucketMaxBits && (n_max >> (bb + 9)) > 0) ++bb;   // ~256-512 rows per bucket
    if (!e->order_v1) bb = ob_bucket_bits(n_max);
    if (const char *d = std::getenv("H2TAP_BUCKET_BITS_DELTA"))      // tuning knob
        bb = std::max(1, std::min(kBucketMaxBits, bb + std::atoi(d)));
    q.plan_dev = static_cast<Q18Plan *>(e->arena.get("q18.plan", sizeof(Q18Plan)));
    // carry records unless disabled for A/B (H2TAP_ORDER_CARRY=0) or on v1
    const char *cv = std::getenv("H2TAP_ORDER_CARRY");
    const bool carry = !e->order_v1 && !(cv && cv[0] == '0');
    if (e->order_v1)  // (the v2 histogram kernel derives the plan itself)
        e->prof.run("q18_plan", [&] {
            launch_q18_plan(q.q18.stats, q.zone, q.q18.nout, bb, carry, q.plan_dev, q.q18.tie, e->compute);
        });
    for (int b = 0; b < 2; ++b) {
        q.sp.k[b] = static_cast<unsigned long long *>(e->arena.get("q18.sk" + std::to_string(b), 8 * n_max));
        q.sp.v[b] = static_cast<unsigned int *>(e->arena.get("q18.sv" + std::to_string(b), 4 * n_max));
    }
    q.sp.counts = static_cast<unsigned int *>(e->arena.get("q18.counts", 4ull * 256 * sort_tiles(n_max)));
    q.sp.totals = static_cast<unsigned int *>(e->arena.get("q18.totals", 4 * 256));
    BucketSort bs;
    bs.k[0] = q.sp.k[0]; bs.k[1] = q.sp.k[1]; bs.v[0] = q.sp.v[0]; bs.v[1] = q.sp.v[1];
    bs.count = static_cast<unsigned int *>(e->arena.get("q18.bcount", 4 * ((1 << kBucketMaxBits) + 1)));
    bs.cursor = static_cast<unsigned int *>(e->arena.get("q18.bcursor", 4 * (1 << kBucketMaxBits)));
    bs.offset = static_cast<unsigned int *>(e->arena.get("q18.boffset", 4 * ((1 << kBucketMaxBits) + 1)));
    bs.big = static_cast<unsigned int *>(e->arena.get("q18.bbig", 4 * ((1 << kBucketMaxBits) + 1)));
    bs.ticket = static_cast<unsigned int *>(e->arena.get("q18.bticket", 64, true, e->compute));
    q.tie_dev = q.q18.tie;  // zeroed by q18_init / q3_init
    q18_alloc_out(e, q, n_max);
    Q18Cols &d = q.out;
    ProfMarks marks(e->prof);
    if (e->order_v1) {
        q18_bucket_order(q.rows, q.amt, q.plan_dev, n_max, bb, bs, d, q.tie_dev, e->num_sms, e->compute,
                         &marks);
    } else {
        bs.mat = static_cast<unsigned int *>(e->arena.get("q18.bmat", 4ull * ob_grid(e->num_sms) << kBucketMaxBits));
        bs.kv = static_cast<unsigned long long *>(e->arena.get("q18.kv", 16 * n_max));
        const Q18PlanArgs pa{q.q18.stats, q.zone, q.q18.nout, carry ? 1 : 0};
        q18_bucket_order_v2(q.rows, q.amt, q.plan_dev, n_max, bb, bs, d, q.tie_dev, e->num_sms, e->compute,
                            &marks, &pa);
    }
}

// Scratch of the orders/customer group-join (Q18, and Q3 which reuses it): join indexes,
// per-orders-row accumulators, counters, statistics and the unsorted result rows (`rows_cap`).
void q18_scratch(h2tap_engine *e, const View &v, QueryCtx &q, uint64_t rows_cap) {
    const int O = H2TAP_T_ORDERS, C = H2TAP_T_CUSTOMER;
    const uint64_t n_o = v.n[O];
    const bool force_hash = q.flags & H2TAP_QUERY_HASH_JOIN;
    Q18Scratch &s = q.q18;
    s.jo = plan_index(e, v, O, force_hash, "q18.jo");
    s.jc = plan_index(e, v, C, force_hash, "q18.jc");
    {   // clustered build sides (row == dense slot), verified on the device by the init kernel;
        // counters per query parity (the init of query k clears those of query k+1)
        auto *viol = static_cast<unsigned int *>(e->arena.get("q18.viol", 64, true, e->compute));
        const int par = (int)(e->q18_runs++ & 1);
        static const bool on = [] { const char *x = std::getenv("H2TAP_CLUSTERED"); return !(x && x[0] == '0'); }();
        s.jo.may_ident = on && s.jo.dense && s.jo.range == v.n[O];
        s.jc.may_ident = on && s.jc.dense && s.jc.range == v.n[C];
        s.jo.viol = viol + 2 * par; s.jo.viol_next = viol + 2 * (par ^ 1);
        s.jc.viol = viol + 2 * par + 1; s.jc.viol_next = viol + 2 * (par ^ 1) + 1;
    }
    s.acc = static_cast<Q18Acc *>(e->arena.get("q18.acc", sizeof(Q18Acc) * std::max<uint64_t>(n_o, 1)));
    s.err = static_cast<unsigned int *>(e->arena.get("q18.err", 64));
    s.nout = static_cast<unsigned long long *>(e->arena.get("q18.nout", 64));
    s.stats = static_cast<Q18Stats *>(e->arena.get("q18.stats", sizeof(Q18Stats)));
    s.stat_part = static_cast<Q18Stats *>(e->arena.get("q18.statpart", sizeof(Q18Stats) * 8 * e->num_sms));
    s.ticket = static_cast<unsigned int *>(e->arena.get("q18.ticket", 64, true, e->compute));
    s.rows = static_cast<Q18Row *>(e->arena.get("q18.rows", sizeof(Q18Row) * std::max<uint64_t>(rows_cap, 1)));
    s.amt = static_cast<long long *>(e->arena.get("q18.amt", 8 * std::max<uint64_t>(rows_cap, 1)));
    s.cand = nullptr;
    s.ncand = nullptr;
    s.qbits = nullptr;
    s.qwords = 0;
    s.tie = static_cast<unsigned int *>(e->arena.get("q18.tie", 64));  // zeroed by the init kernel
    q.r->plan_flags = (s.jo.dense ? 1u : 0u) | (s.jc.dense ? 2u : 0u);
}

void q18_gather_and_order(h2tap_engine *e, QueryCtx &q, uint64_t n_rows_max);

// Bounds of the result rows' (w, d, o) and payload fields from the published zone maps: every
// result row is an orders row matched to a customer row of this snapshot. Q3 returns no
// customer / o_ol_cnt fields (its rows carry zeros there).
Q18Zone q18_zone(const View &v, bool q3) {
    const int O = H2TAP_T_ORDERS, C = H2TAP_T_CUSTOMER;
    Q18Zone z{};
    z.w_min = v.smin[O][0]; z.w_max = v.smax[O][0];
    z.d_min = v.smin[O][1]; z.d_max = v.smax[O][1];
    z.o_min = v.smin[O][2]; z.o_max = v.smax[O][2];
    if (!q3) {
        z.cl_min = v.smin[C][3]; z.cl_max = v.smax[C][3];
        z.ci_min = v.smin[C][2]; z.ci_max = v.smax[C][2];
        z.n_min = v.smin[O][3]; z.n_max = v.smax[O][3];
    }
    z.has_e = v.has_stats64[O] ? 1 : 0;
    z.e_min = v.smin64[O];
    z.e_max = v.smax64[O];
    return z;
}

// HAVING of the v2 path: the 32-byte result rows + amounts (compacted) and their statistics.
void q18_having_v2(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int O = H2TAP_T_ORDERS, C = H2TAP_T_CUSTOMER;
    const uint64_t n_o = v.n[O];
    e->prof.run("q18_having_compact", [&] {
        if (n_o)
            launch_q18_having(colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID),
                              colp<int32_t>(v, O, H2TAP_O_ID), colp<int32_t>(v, O, H2TAP_O_C_ID),
                              colp<int32_t>(v, O, H2TAP_O_OL_CNT), colp<int64_t>(v, O, H2TAP_O_ENTRY_D),
                              n_o, colp<int32_t>(v, C, H2TAP_C_LAST), q.p[0], q.q18, e->num_sms, e->compute,
                              e->having_unroll);
    });
    CK(cudaGetLastError());
}

void q18_order_dist(h2tap_engine *e, QueryCtx &q, const Q18HavingArgs *hv = nullptr,
                    const unsigned long long *nout_for_meta = nullptr);

// Q18 v3: statistics of the accumulators -> plan -> HAVING writes the carry records
// and the bucket counts -> scan -> scatter -> per-bucket sort + emit (world > 1: the distributed
// ORDER BY of §6.3 on the same records).
void q18_launch_v3(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int O = H2TAP_T_ORDERS, C = H2TAP_T_CUSTOMER;
    const uint64_t n_o = v.n[O];
    const uint64_t n_max = std::max<uint64_t>(n_o, 1);
    Q18Scratch &s = q.q18;
    q.v3 = true;
    q.n_max = n_o;
    q.tie_dev = s.tie;
    const int G = ob_grid(e->num_sms);
    auto *cpart = static_cast<unsigned long long *>(e->arena.get("q18.cpart", 8ull * 8 * e->num_sms));
    auto *scount = static_cast<unsigned long long *>(e->arena.get("q18.scount", 64));
    auto *cnt_part = static_cast<unsigned int *>(e->arena.get("q18.cntpart", 4ull * G));
    q.plan_dev = static_cast<Q18Plan *>(e->arena.get("q18.plan", sizeof(Q18Plan)));
    const size_t nbm = size_t(1) << kBucketMaxBits;
    BucketSort &bs = q.bs;
    bs = BucketSort{};
    bs.k[0] = static_cast<unsigned long long *>(e->arena.get("q18.rec", 16 * n_max));  // HAVING's records
    bs.kv = static_cast<unsigned long long *>(e->arena.get("q18.kv", 16 * n_max));
    bs.count = static_cast<unsigned int *>(e->arena.get("q18.bcount", 4 * (nbm + 1)));
    bs.offset = static_cast<unsigned int *>(e->arena.get("q18.boffset", 4 * (nbm + 1)));
    bs.big = static_cast<unsigned int *>(e->arena.get("q18.bbig", 4 * (nbm + 1)));
    bs.ticket = static_cast<unsigned int *>(e->arena.get("q18.bticket", 64, true, e->compute));
    bs.mat = static_cast<unsigned int *>(e->arena.get("q18.bmat", 4ull * G * nbm));
    const int64_t *o_ent = colp<int64_t>(v, O, H2TAP_O_ENTRY_D);
    ProfMarks marks(e->prof);
    if (e->world > 1) {
        e->prof.run("q18_acc_stats", [&] {
            launch_q18_acc_stats(s, o_ent, n_o, q.p[0], cpart, scount, nullptr, 0, nullptr, q.tie_dev,
                                 e->num_sms, e->compute);
        });
        const Q18HavingArgs hv{colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID),
                               colp<int32_t>(v, O, H2TAP_O_ID), colp<int32_t>(v, O, H2TAP_O_C_ID),
                               colp<int32_t>(v, O, H2TAP_O_OL_CNT), o_ent, n_o,
                               colp<int32_t>(v, C, H2TAP_C_LAST), q.p[0], s, cnt_part};
        q18_order_dist(e, q, &hv, scount);
        return;
    }
    int bb = ob_bucket_bits(n_max);
    if (const char *d = std::getenv("H2TAP_BUCKET_BITS_DELTA"))
        bb = std::max(1, std::min(kBucketMaxBits, bb + std::atoi(d)));
    q18_alloc_out(e, q, n_max);
    const Q18PlanArgs pa{s.stats, q.zone, nullptr, 1};
    // the plan and the bucket counts in one kernel (grid barrier): direct ORDER BY, o_entry_d's bounds
    // from the zone map, the grid resident at once, no other engine on the device (§4.4)
    const char *dx = std::getenv("H2TAP_ORDER_DIRECT"), *fx = std::getenv("H2TAP_PLAN_HIST");
    const bool fused = !(dx && dx[0] == '0') && !(fx && fx[0] == '0') && q.zone.has_e &&
                       engines_on_device(e->device) == 1 && q18_plan_hist_ok(e->num_sms, bb);
    if (fused)
        e->prof.run("q18_plan_count", [&] {
            launch_q18_plan_hist(s, n_o, q.p[0], cpart,
                                 static_cast<unsigned long long *>(e->arena.get("q18.gbar", 64, true, e->compute)),
                                 scount, q.zone, bb, q.plan_dev, q.tie_dev, bs, e->num_sms, e->compute);
        });
    else
    e->prof.run("q18_acc_stats", [&] {
        launch_q18_acc_stats(s, o_ent, n_o, q.p[0], cpart, scount, &pa, bb, q.plan_dev, q.tie_dev, e->num_sms,
                             e->compute);
    });
    q18_order_v3(colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID), colp<int32_t>(v, O, H2TAP_O_ID),
                 colp<int32_t>(v, O, H2TAP_O_C_ID), colp<int32_t>(v, O, H2TAP_O_OL_CNT), o_ent, n_o,
                 colp<int32_t>(v, C, H2TAP_C_LAST), q.p[0], s, q.plan_dev, bb, bs, cnt_part, q.out, q.tie_dev,
                 e->num_sms, e->compute, &marks, fused);
    CK(cudaGetLastError());
    launch_q18_publish(s.nout, s.err, q.tie_dev, q.small_dev, s.jo, s.jc, e->compute);  // -> small (mapped)
}

// The v3 records did not fit 128 bits (or a bucket overflowed): redo HAVING + ORDER BY on the v2
// path from the accumulators, which are intact (host-synchronous; rare on realistic data).
void q18_rerun_v2(h2tap_engine *e, QueryCtx &q) {
    Q18Scratch &s = q.q18;
    const Q18Stats init{INT64_MAX, INT64_MIN, INT64_MAX, INT64_MIN};
    CK(cudaMemsetAsync(s.nout, 0, 8, e->compute));
    CK(cudaMemsetAsync(s.tie, 0, 4, e->compute));
    CK(cudaMemcpyAsync(s.stats, &init, sizeof init, cudaMemcpyHostToDevice, e->compute));
    release_dev_blocks(e, q);
    q.v3 = false;
    q18_having_v2(e, *q.view, q);
    q18_gather_and_order(e, q, q.view->n[H2TAP_T_ORDERS]);
    sync_compute(e);
}

// Q18's steps before its probe: join-index plan, init (+ clustered-side verify, zeroed
// accumulators) and build. Run by the batch's full pass ahead of it, or by launch_q18_plan.
void q18_pre_probe(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int O = H2TAP_T_ORDERS, C = H2TAP_T_CUSTOMER;
    need_cols(v, O, {H2TAP_O_W_ID, H2TAP_O_D_ID, H2TAP_O_ID, H2TAP_O_C_ID, H2TAP_O_OL_CNT, H2TAP_O_ENTRY_D}, "Q18");
    need_cols(v, C, {H2TAP_C_W_ID, H2TAP_C_D_ID, H2TAP_C_ID, H2TAP_C_LAST}, "Q18");
    const uint64_t n_o = v.n[O], n_c = v.n[C];
    q18_scratch(e, v, q, n_o);
    Q18Scratch &s = q.q18;
    e->prof.run("q18_init", [&] {
        launch_q18_init(s, colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID),
                        colp<int32_t>(v, O, H2TAP_O_ID), n_o, colp<int32_t>(v, C, H2TAP_C_W_ID),
                        colp<int32_t>(v, C, H2TAP_C_D_ID), colp<int32_t>(v, C, H2TAP_C_ID), n_c, e->num_sms,
                        e->compute);
    });
    e->prof.run("q18_build", [&] {
        launch_q18_build(colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID),
                         colp<int32_t>(v, O, H2TAP_O_ID), n_o, colp<int32_t>(v, C, H2TAP_C_W_ID),
                         colp<int32_t>(v, C, H2TAP_C_D_ID), colp<int32_t>(v, C, H2TAP_C_ID), n_c, s,
                         e->num_sms, e->compute);
    });
}

void launch_q18_plan(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int OL = H2TAP_T_ORDER_LINE, O = H2TAP_T_ORDERS, C = H2TAP_T_CUSTOMER;
    need_cols(v, OL, {H2TAP_OL_W_ID, H2TAP_OL_D_ID, H2TAP_OL_O_ID, H2TAP_OL_AMOUNT}, "Q18");
    need_cols(v, O, {H2TAP_O_W_ID, H2TAP_O_D_ID, H2TAP_O_ID, H2TAP_O_C_ID, H2TAP_O_OL_CNT, H2TAP_O_ENTRY_D}, "Q18");
    need_cols(v, C, {H2TAP_C_W_ID, H2TAP_C_D_ID, H2TAP_C_ID, H2TAP_C_LAST}, "Q18");
    const uint64_t n_ol = v.n[OL], n_o = v.n[O];
    Q18Scratch &s = q.q18;
    if (!q.probe_done) {  // else the batch's full pass ran them (launch_q6_plan)
        q18_pre_probe(e, v, q);
        e->prof.run("q18_probe_groupjoin", [&] {
            if (n_ol)
                ((e->probe_tma || e->zc_tma) && (e->probe_tma || v.any_host(OL, {H2TAP_OL_W_ID, H2TAP_OL_D_ID, H2TAP_OL_O_ID, H2TAP_OL_AMOUNT}))
                     ? launch_q18_probe_tma : launch_q18_probe)(colp<int32_t>(v, OL, H2TAP_OL_W_ID), colp<int32_t>(v, OL, H2TAP_OL_D_ID),
                                 colp<int32_t>(v, OL, H2TAP_OL_O_ID), colp<int64_t>(v, OL, H2TAP_OL_AMOUNT),
                                 n_ol, s, e->num_sms, e->compute);
        });
    }
    CK(cudaGetLastError());
    q.zone = q18_zone(v, false);
    q.view = &v;
    const char *cv = std::getenv("H2TAP_ORDER_CARRY");
    if (!e->order_v1 && !(cv && cv[0] == '0')) {  // v3: HAVING builds the carry records
        q18_launch_v3(e, v, q);
        return;
    }
    q18_having_v2(e, v, q);
    q18_gather_and_order(e, q, n_o);
}

// a7 + a8 of Q18 (and Q3) with world > 1: the distributed ORDER BY. Every rank
// ends up with its range of the global order; nothing is gathered, nothing waits for the host.
void q18_order_dist(h2tap_engine *e, QueryCtx &q, const Q18HavingArgs *hv, const unsigned long long *nout_for_meta) {
    Q18Scratch &s = q.q18;
    const uint64_t n_max = std::max<uint64_t>(q.n_max, 1);
    const size_t nbm = size_t(1) << kBucketMaxBits;
    q.plan_dev = static_cast<Q18Plan *>(e->arena.get("q18.plan", sizeof(Q18Plan)));
    BucketSort &bs = q.bs;
    bs = BucketSort{};
    bs.count = static_cast<unsigned int *>(e->arena.get("q18.bcount", 4 * (nbm + 1)));
    bs.offset = static_cast<unsigned int *>(e->arena.get("q18.boffset", 4 * (nbm + 1)));
    bs.big = static_cast<unsigned int *>(e->arena.get("q18.bbig", 4 * (nbm + 1)));
    bs.ticket = static_cast<unsigned int *>(e->arena.get("q18.bticket", 64, true, e->compute));
    bs.mat = static_cast<unsigned int *>(e->arena.get("q18.bmat", 4ull * ob_grid(e->num_sms) * nbm));
    bs.kv = static_cast<unsigned long long *>(e->arena.get("q18.kv", 16 * n_max));
    if (hv) bs.k[0] = static_cast<unsigned long long *>(e->arena.get("q18.rec", 16 * n_max));
    auto *send = static_cast<unsigned long long *>(e->arena.get("q18.dsend", 8 * nbm));
    q.recv_off = static_cast<unsigned int *>(e->arena.get("q18.drecv", 4 * (nbm + 1)));
    // output capacity: ~1/world of the global result lands here; twice the local orders rows
    // covers any balanced sharding (more: kPeerErrOutCap, re-emitted into exact columns at finish)
    uint64_t cap = 2 * n_max + 4096;
    if (const char *c = std::getenv("H2TAP_DIST_OUT_CAP")) cap = std::strtoull(c, nullptr, 10);
    q.dist_out_cap = cap;
    q18_alloc_out(e, q, std::max<uint64_t>(cap, 1));
    const char *cv = std::getenv("H2TAP_ORDER_CARRY");
    const bool carry = !(cv && cv[0] == '0');
    q.tie_dev = s.tie;
    const Q18PlanArgs meta{s.stats, q.zone, nout_for_meta ? nout_for_meta : s.nout, carry ? 1 : 0};
    ProfMarks marks(e->prof);
    q18_bucket_order_dist(e->peer.args, q.rows, q.amt, q.plan_dev, meta, s.err, bs, send, q.recv_off, cap, q.out,
                          q.tie_dev, q.small_dev, e->num_sms, e->compute, &marks, hv);
    q.dist = true;
}

// a8 of Q18 (and Q3): the ORDER BY on the device and the scalar read-backs (mapped pinned).
// `n_rows_max` bounds the local row count.
void q18_gather_and_order(h2tap_engine *e, QueryCtx &q, uint64_t n_rows_max) {
    Q18Scratch &s = q.q18;
    q.rows = s.rows;
    q.amt = s.amt;
    q.n_max = n_rows_max;
    if (e->world > 1) {
        q18_order_dist(e, q);
        return;
    }
    q18_sort_and_emit(e, q);
    launch_q18_publish(s.nout, s.err, q.tie_dev, q.small_dev, s.jo, s.jc, e->compute);  // -> small (mapped)
}

// ---- NEXT-2: CH Q3 (customer ⋈ new_order ⋈ orders ⋈ order_line) on the Q18 machinery
void launch_q3_plan(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int OL = H2TAP_T_ORDER_LINE, O = H2TAP_T_ORDERS, C = H2TAP_T_CUSTOMER, NO = H2TAP_T_NEW_ORDER;
    need_cols(v, OL, {H2TAP_OL_W_ID, H2TAP_OL_D_ID, H2TAP_OL_O_ID, H2TAP_OL_AMOUNT}, "Q3");
    need_cols(v, O, {H2TAP_O_W_ID, H2TAP_O_D_ID, H2TAP_O_ID, H2TAP_O_C_ID, H2TAP_O_OL_CNT, H2TAP_O_ENTRY_D}, "Q3");
    need_cols(v, C, {H2TAP_C_W_ID, H2TAP_C_D_ID, H2TAP_C_ID, H2TAP_C_STATE_P2}, "Q3");
    need_cols(v, NO, {H2TAP_NO_W_ID, H2TAP_NO_D_ID, H2TAP_NO_O_ID}, "Q3");
    const uint64_t n_ol = v.n[OL], n_o = v.n[O], n_c = v.n[C], n_no = v.n[NO];
    const uint64_t cap = std::min<uint64_t>(n_o, n_no);  // result rows <= distinct marked orders
    q18_scratch(e, v, q, cap);
    Q18Scratch &s = q.q18;
    s.cand = static_cast<unsigned int *>(e->arena.get("q3.cand", 4 * std::max<uint64_t>(cap, 1)));
    s.ncand = static_cast<unsigned long long *>(e->arena.get("q3.ncand", 64));
    s.qwords = (n_o + 31) / 32;
    s.qbits = static_cast<unsigned int *>(e->arena.get("q3.bits", 4 * std::max<uint64_t>(s.qwords, 1)));
    e->prof.run("q3_init", [&] {
        launch_q18_init(s, colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID),
                        colp<int32_t>(v, O, H2TAP_O_ID), n_o, colp<int32_t>(v, C, H2TAP_C_W_ID),
                        colp<int32_t>(v, C, H2TAP_C_D_ID), colp<int32_t>(v, C, H2TAP_C_ID), n_c, e->num_sms,
                        e->compute);
    });
    e->prof.run("q3_build", [&] {
        launch_q18_build(colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID),
                         colp<int32_t>(v, O, H2TAP_O_ID), n_o, colp<int32_t>(v, C, H2TAP_C_W_ID),
                         colp<int32_t>(v, C, H2TAP_C_D_ID), colp<int32_t>(v, C, H2TAP_C_ID), n_c, s,
                         e->num_sms, e->compute);
    });
    e->prof.run("q3_mark", [&] {
        if (n_no)
            launch_q3_mark(colp<int32_t>(v, NO, H2TAP_NO_W_ID), colp<int32_t>(v, NO, H2TAP_NO_D_ID),
                           colp<int32_t>(v, NO, H2TAP_NO_O_ID), colp<int32_t>(v, NO, H2TAP_NO_DELETED), n_no, colp<int32_t>(v, O, H2TAP_O_W_ID),
                           colp<int32_t>(v, O, H2TAP_O_D_ID), colp<int32_t>(v, O, H2TAP_O_C_ID),
                           colp<int64_t>(v, O, H2TAP_O_ENTRY_D), colp<int32_t>(v, C, H2TAP_C_STATE_P2),
                           q.p[0], (int)q.p[1], s, e->num_sms, e->compute);
    });
    e->prof.run("q3_probe_groupjoin", [&] {
        if (n_ol && n_no)
            launch_q3_probe(colp<int32_t>(v, OL, H2TAP_OL_W_ID), colp<int32_t>(v, OL, H2TAP_OL_D_ID),
                            colp<int32_t>(v, OL, H2TAP_OL_O_ID), colp<int64_t>(v, OL, H2TAP_OL_AMOUNT),
                            n_ol, s, e->num_sms, e->compute);
    });
    e->prof.run("q3_emit", [&] {
        if (cap)
            launch_q3_emit(colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID),
                           colp<int32_t>(v, O, H2TAP_O_ID), colp<int32_t>(v, O, H2TAP_O_C_ID),
                           colp<int32_t>(v, O, H2TAP_O_OL_CNT), colp<int64_t>(v, O, H2TAP_O_ENTRY_D), cap, s,
                           e->num_sms, e->compute);
    });
    CK(cudaGetLastError());
    q.zone = q18_zone(v, true);
    q18_gather_and_order(e, q, cap);
}

void finish_q18(h2tap_engine *e, QueryCtx &q) {
    ResultImpl *r = q.r.get();
    Q18Small *sm = static_cast<Q18Small *>(q.small.first);
    const bool q3 = q.plan == H2TAP_Q3;  // Q3 returns 5 of the sorted columns (R33)
    const char *const *names = q3 ? kQ3Names : kQ18Names;
    const uint32_t *types = q3 ? kQ3Types : kQ18Types;
    const int ncols = q3 ? 5 : 8;
    // (carry did not fit, a bucket overflowed, or the direct ORDER BY counted a row with no customer)
    if (q.v3 && !q.dist && (sm->tie & (1u | 2u | 4u | 8u | 16u))) q18_rerun_v2(e, q);
    const unsigned int err = sm->err;  // world > 1: every rank's join errors and the exchange's
    const unsigned pl = q.plan;
    if (err & kPeerErrTimeout) {
        e->peer.broken = true;
        raise(H2TAP_EPEER, "Q%u: a peer did not deliver its ORDER BY exchange in time", pl);
    }
    if (err & kErrDupOrders) raise(H2TAP_EDUPKEY, "Q%u: duplicate orders primary key (w, d, o_id)", pl);
    if (err & kErrDupCustomer) raise(H2TAP_EDUPKEY, "Q%u: duplicate customer primary key (w, d, c_id)", pl);
    if (err & kErrDomain) raise(H2TAP_EPLAN, "Q%u: join key outside the supported domain", pl);
    if (err & kPeerErrHeap)
        raise(H2TAP_ENOMEM, "Q%u: a rank's share of the distributed ORDER BY exceeds its peer heap "
              "(h2tap_config.peer_heap_bytes)", pl);
    if (err & kPeerErrNoCarry)
        raise(H2TAP_EPLAN, "Q%u: the distributed ORDER BY needs 128-bit carry records; the result "
              "fields are too wide", pl);
    const uint64_t nout = sm->nout;
    if (!q.dist) r->plan_flags |= (sm->clustered & 3u) << 3;  // bit3 / bit4: positional indexes
    r->total_rows = q.dist ? sm->n_total : nout;
    r->row_offset = q.dist ? sm->row0 : 0;
    if (q.dist && (err & kPeerErrOutCap)) {
        // this rank's slice exceeded the output columns: re-emit from the heap into exact ones
        // (the exchanged records stay there until the next exchange of the same parity)
        release_dev_blocks(e, q);
        q18_alloc_out(e, q, std::max<uint64_t>(nout, 1));
        const unsigned int cleared = err & ~kPeerErrOutCap;
        CK(cudaMemcpyAsync(reinterpret_cast<char *>(q.plan_dev) + offsetof(Q18Plan, err), &cleared, 4,
                           cudaMemcpyHostToDevice, e->compute));
        q18_dist_emit(e->peer.args, q.plan_dev, q.recv_off, q.out, q.tie_dev, q.bs, e->num_sms, e->compute);
        sync_compute(e);
    }
    if (!q.dist && sm->tie && nout > 1) {
        // a run of > 32 equal 64-bit prefixes, or a bucket larger than shared memory: redo
        // exactly, one stable LSD radix sort per field (r, then e, then a)
        SortPairs w = q.sp;
        Q18Plan hp;
        CK(cudaMemcpy(&hp, q.plan_dev, sizeof hp, cudaMemcpyDeviceToHost));
        launch_iota(w.v[0], nout, e->num_sms, e->compute);
        // (r = the concatenated (w, d, o) fields; wider than 62 bits: o, d, w sorted one by one)
        const bool wide = hp.spec.wide_r != 0;
        const int fid[5] = {3, 4, 5, 1, 2};
        const int nf = wide ? 5 : 3;
        for (int k = 0; k < nf; ++k) {
            const int f = wide ? fid[k] : k;
            const int bits = f == 0 ? hp.spec.bits_r : f == 1 ? hp.spec.bits_e : f == 2 ? hp.spec.bits_a
                           : f == 3 ? hp.spec.bits_o : f == 4 ? hp.spec.bits_d : hp.spec.bits_w;
            launch_q18_field_keys(q.rows, q.amt, w.v[0], nout, f, q.plan_dev, w.k[0], e->num_sms, e->compute);
            const int cur = radix_sort_pairs(nout, bits, w, e->num_sms, e->compute);
            if (cur) { std::swap(w.k[0], w.k[1]); std::swap(w.v[0], w.v[1]); }
        }
        // keys are field keys, not the prefix: amounts are read from amt[]
        launch_q18_permute(q.rows, q.amt, w.v[0], nullptr, q.plan_dev, nout, q.out, e->num_sms, e->compute);
        CK(cudaGetLastError());
    }
    r->nrows = nout;
    const void *src18[8] = {q.out.c_last, q.out.c_id, q.out.o_id, q.out.o_entry_d, q.out.o_ol_cnt,
                            q.out.amount_sum, q.out.o_w_id, q.out.o_d_id};
    const void *src3[5] = {q.out.o_id, q.out.o_w_id, q.out.o_d_id, q.out.amount_sum, q.out.o_entry_d};
    const void *const *src = q3 ? src3 : src18;
    const size_t es18[8] = {4, 4, 4, 8, 4, 8, 4, 4}, es3[5] = {4, 4, 4, 8, 8};
    const size_t *es = q3 ? es3 : es18;
    if (r->on_device) {
        for (int i = 0; i < ncols; ++i) add_col(r, names[i], types[i], src[i]);
        give_blocks_to_result(q);
        if (sm->tie) sync_compute(e);
        return;
    }
    for (int i = 0; i < ncols; ++i) {
        void *h = result_block(r, nout * es[i]);
        if (nout) CK(cudaMemcpyAsync(h, src[i], nout * es[i], cudaMemcpyDeviceToHost, e->compute));
        add_col(r, names[i], types[i], h);
    }
    sync_compute(e);
    release_dev_blocks(e, q);
}

// ---- NEXT-2: CH Q14 (order_line ⋈ item), Q12 (orders ⋈ order_line), Q4 (orders ⋉ order_line)
struct SgSmall { unsigned long long ngroups; unsigned int flags, err; };
struct Q14Small { long long out[3]; double promo; unsigned int err; };

void raise_join_err(unsigned int err, const char *plan) {
    if (err & kErrDupOrders) raise(H2TAP_EDUPKEY, "%s: duplicate orders primary key (w, d, o_id)", plan);
    if (err & kErrDupItem) raise(H2TAP_EDUPKEY, "%s: duplicate item primary key i_id", plan);
    if (err & kErrDomain) raise(H2TAP_EPLAN, "%s: join key outside the supported domain", plan);
}

void launch_q14_plan(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int OL = H2TAP_T_ORDER_LINE, I = H2TAP_T_ITEM;
    need_cols(v, OL, {H2TAP_OL_DELIVERY_D, H2TAP_OL_I_ID, H2TAP_OL_AMOUNT}, "Q14");
    need_cols(v, I, {H2TAP_I_ID, H2TAP_I_DATA_P2}, "Q14");
    const uint64_t n_i = v.n[I];
    ItemMap m{};
    if (n_i) {  // i_id box from the item zone map (R31)
        if (!v.has_stats[I]) raise(H2TAP_EPLAN, "Q14: no statistics for item");
        m.i0 = v.smin[I][0];
        m.range = (unsigned long long)((long long)v.smax[I][0] - v.smin[I][0] + 1);
        if (m.range > (1ull << 28)) raise(H2TAP_EPLAN, "Q14: item ids span %llu values (> 2^28)", m.range);
        m.words = (m.range + 15) / 16;
    }
    m.bits = static_cast<unsigned int *>(e->arena.get("q14.map", 4 * (m.words + 1)));
    Q14Scratch &s = q.q14;
    s.block_part = static_cast<long long *>(e->arena.get("q14.part", 24ull * q14_max_blocks(e->num_sms)));
    s.done_counter = static_cast<unsigned int *>(e->arena.get("q14.counter", 64, true, e->compute));
    s.out = static_cast<long long *>(e->arena.get("q14.out", 32));
    s.promo = static_cast<double *>(dev_block(e, q, 8));
    q.err = static_cast<unsigned int *>(e->arena.get("q14.err", 64));
    CK(cudaMemsetAsync(q.err, 0, 4, e->compute));
    q.r->plan_flags = m.words <= 16384 ? 4u : 0u;  // bit2: item map held in shared memory
    e->prof.run("q14_item_map", [&] {
        launch_item_map(colp<int32_t>(v, I, H2TAP_I_ID), colp<int32_t>(v, I, H2TAP_I_DATA_P2), n_i,
                        (int32_t)q.p[2], m, q.err, e->num_sms, e->compute);
    });
    e->prof.run("q14_scan_join_sum", [&] {
        launch_q14(colp<int64_t>(v, OL, H2TAP_OL_DELIVERY_D), colp<int32_t>(v, OL, H2TAP_OL_I_ID),
                   colp<int64_t>(v, OL, H2TAP_OL_AMOUNT), v.n[OL], q.p[0], q.p[1], m, s, e->num_sms,
                   e->compute);
        CK(cudaGetLastError());
    });
    if (e->world > 1)
        e->prof.run("q14_peer_allreduce", [&] {
            launch_peer_allreduce_i64(e->peer.args, s.out, 3, s.out, nullptr, e->compute);
        });
    e->prof.run("q14_finalize", [&] { launch_q14_finalize(s, e->compute); });
    auto *sm = static_cast<Q14Small *>(q.small.first);
    CK(cudaMemcpyAsync(sm->out, s.out, 24, cudaMemcpyDeviceToHost, e->compute));
    CK(cudaMemcpyAsync(&sm->promo, s.promo, 8, cudaMemcpyDeviceToHost, e->compute));
    CK(cudaMemcpyAsync(&sm->err, q.err, 4, cudaMemcpyDeviceToHost, e->compute));
}

void finish_q14(h2tap_engine *e, QueryCtx &q) {
    ResultImpl *r = q.r.get();
    const auto *sm = static_cast<const Q14Small *>(q.small.first);
    raise_join_err(sm->err, "Q14");
    r->nrows = 1;
    const bool null = sm->out[2] == 0;  // SUM over no joined row IS NULL -> NULL ratio (R30)
    auto *blk = static_cast<long long *>(result_block(r, 32));
    if (r->on_device) {
        CK(cudaMemcpyAsync(blk, sm->out, 24, cudaMemcpyHostToDevice, e->compute));
        sync_compute(e);
        add_col(r, "promo_revenue", H2TAP_F64, q.q14.promo);
        give_blocks_to_result(q);
    } else {
        std::memcpy(blk, sm->out, 24);
        std::memcpy(blk + 3, &sm->promo, 8);
        add_col(r, "promo_revenue", H2TAP_F64, blk + 3);
        release_dev_blocks(e, q);
    }
    r->null_store.back().assign(1, null ? 1 : 0);
    add_col(r, "sum_promo", H2TAP_I64, blk);
    r->null_store.back().assign(1, null ? 1 : 0);
    add_col(r, "sum_amount", H2TAP_I64, blk + 1);
    r->null_store.back().assign(1, null ? 1 : 0);
    add_col(r, "count_rows", H2TAP_I64, blk + 2);
}

// small-group tables (dense | gtag | gacc contiguous, so one allgather moves them) + outputs
void sg_setup(h2tap_engine *e, QueryCtx &q) {
    SmallGroups &g = q.sg;
    const bool fresh = !e->arena.bufs.count("sg.tables");
    auto *t = static_cast<unsigned long long *>(e->arena.get("sg.tables", 8ull * (3 * kSgDense + 4 * kSgSlots)));
    g.dense = t;
    g.gtag = t + 3 * kSgDense;
    g.gacc = g.gtag + kSgSlots;
    g.flags = static_cast<unsigned int *>(e->arena.get("sg.flags", 64));
    g.ngroups = static_cast<unsigned long long *>(e->arena.get("sg.ngroups", 64));
    const size_t maxg = kSgSlots + kSgDense;
    g.o_key = static_cast<int32_t *>(dev_block(e, q, 4 * maxg));
    g.o_a = static_cast<long long *>(dev_block(e, q, 8 * maxg));
    g.o_b = static_cast<long long *>(dev_block(e, q, 8 * maxg));
    if (fresh) launch_sg_reset(g, e->compute);  // the emit kernel re-clears after every query
    q.err = static_cast<unsigned int *>(e->arena.get("sg.err", 64));
    CK(cudaMemsetAsync(q.err, 0, 4, e->compute));
}

void sg_merge_and_emit(h2tap_engine *e, QueryCtx &q, const char *name) {
    SmallGroups &g = q.sg;
    if (e->world > 1) {  // a7: every rank's tables to every rank's mailbox, folded into the local one
        const size_t words = 3 * kSgDense + 4 * kSgSlots;
        e->prof.run((std::string(name) + "_peer_merge").c_str(), [&] {
            launch_peer_push(e->peer.args, g.dense, nullptr, words, 8u, e->num_sms, e->compute);
            launch_peer_wait(e->peer.args, e->compute);
            launch_sg_peer_merge(e->peer.args, g, e->compute);
        });
    }
    e->prof.run((std::string(name) + "_emit").c_str(), [&] { launch_sg_emit(g, e->compute); });
    auto *sm = static_cast<SgSmall *>(q.small.first);
    CK(cudaMemcpyAsync(&sm->ngroups, g.ngroups, 8, cudaMemcpyDeviceToHost, e->compute));
    CK(cudaMemcpyAsync(&sm->flags, g.flags, 4, cudaMemcpyDeviceToHost, e->compute));
    CK(cudaMemcpyAsync(&sm->err, q.err, 4, cudaMemcpyDeviceToHost, e->compute));
}

JoinIndex plan_orders_index(h2tap_engine *e, const View &v, QueryCtx &q, const char *plan) {
    const int O = H2TAP_T_ORDERS;
    JoinIndex jo = plan_index(e, v, O, q.flags & H2TAP_QUERY_HASH_JOIN, "ch.jo");
    q.r->plan_flags = jo.dense ? 1u : 0u;
    {   // clustered orders (row == dense slot), verified on the device before the build: the
        // index is then positional and nothing is cleared or inserted
        auto *viol = static_cast<unsigned int *>(e->arena.get("ch.viol", 64, true, e->compute));
        const int par = (int)(e->ch_runs++ & 1);
        static const bool on = [] { const char *x = std::getenv("H2TAP_CLUSTERED"); return !(x && x[0] == '0'); }();
        jo.may_ident = on && jo.dense && jo.range == v.n[O];
        jo.viol = viol + par;
        jo.viol_next = viol + (par ^ 1);
    }
    (void)plan;
    return jo;
}

void launch_q12_plan(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int OL = H2TAP_T_ORDER_LINE, O = H2TAP_T_ORDERS;
    need_cols(v, OL, {H2TAP_OL_W_ID, H2TAP_OL_D_ID, H2TAP_OL_O_ID, H2TAP_OL_DELIVERY_D}, "Q12");
    need_cols(v, O, {H2TAP_O_W_ID, H2TAP_O_D_ID, H2TAP_O_ID, H2TAP_O_OL_CNT, H2TAP_O_CARRIER_ID, H2TAP_O_ENTRY_D}, "Q12");
    sg_setup(e, q);
    const JoinIndex jo = plan_orders_index(e, v, q, "Q12");
    e->prof.run("q12_build", [&] {
        launch_jx_build_orders(colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID),
                               colp<int32_t>(v, O, H2TAP_O_ID), v.n[O], jo, q.err, nullptr, e->num_sms, e->compute);
    });
    e->prof.run("q12_probe_groupby", [&] {
        if (v.n[OL])
            launch_q12_probe(colp<int32_t>(v, OL, H2TAP_OL_W_ID), colp<int32_t>(v, OL, H2TAP_OL_D_ID),
                             colp<int32_t>(v, OL, H2TAP_OL_O_ID), colp<int64_t>(v, OL, H2TAP_OL_DELIVERY_D),
                             v.n[OL], jo, colp<int64_t>(v, O, H2TAP_O_ENTRY_D), colp<int32_t>(v, O, H2TAP_O_CARRIER_ID),
                             colp<int32_t>(v, O, H2TAP_O_OL_CNT), q.p[0], q.sg, e->num_sms, e->compute);
        CK(cudaGetLastError());
    });
    sg_merge_and_emit(e, q, "q12");
}

void launch_q4_plan(h2tap_engine *e, const View &v, QueryCtx &q) {
    const int OL = H2TAP_T_ORDER_LINE, O = H2TAP_T_ORDERS;
    need_cols(v, OL, {H2TAP_OL_W_ID, H2TAP_OL_D_ID, H2TAP_OL_O_ID, H2TAP_OL_DELIVERY_D}, "Q4");
    need_cols(v, O, {H2TAP_O_W_ID, H2TAP_O_D_ID, H2TAP_O_ID, H2TAP_O_OL_CNT, H2TAP_O_ENTRY_D}, "Q4");
    sg_setup(e, q);
    const JoinIndex jo = plan_orders_index(e, v, q, "Q4");
    auto *mark = static_cast<uint8_t *>(e->arena.get("q4.mark", std::max<uint64_t>(v.n[O], 1) + 16));
    e->prof.run("q4_build", [&] {
        launch_jx_build_orders(colp<int32_t>(v, O, H2TAP_O_W_ID), colp<int32_t>(v, O, H2TAP_O_D_ID),
                               colp<int32_t>(v, O, H2TAP_O_ID), v.n[O], jo, q.err, mark, e->num_sms, e->compute);
    });
    struct Marks : PhaseMarks {
        Prof &p;
        cudaEvent_t a = nullptr;
        std::string name;
        explicit Marks(Prof &pr) : p(pr) {}
        void begin(const char *nm) override {
            if (!p.on) return;
            name = nm;
            a = p.ev();
            CK(cudaEventRecord(a, p.st));
        }
        void end() override {
            if (!p.on) return;
            cudaEvent_t b = p.ev();
            CK(cudaEventRecord(b, p.st));
            p.marks.push_back({name, {a, b}});
        }
    } marks(e->prof);
    launch_q4(colp<int32_t>(v, OL, H2TAP_OL_W_ID), colp<int32_t>(v, OL, H2TAP_OL_D_ID),
              colp<int32_t>(v, OL, H2TAP_OL_O_ID), colp<int64_t>(v, OL, H2TAP_OL_DELIVERY_D), v.n[OL], jo,
              colp<int64_t>(v, O, H2TAP_O_ENTRY_D), colp<int32_t>(v, O, H2TAP_O_OL_CNT), v.n[O], q.p[0], q.p[1],
              mark, q.sg, e->num_sms, e->compute, &marks);
    CK(cudaGetLastError());
    sg_merge_and_emit(e, q, "q4");
}

void finish_groups(h2tap_engine *e, QueryCtx &q, const char *plan, const char *a_name, const char *b_name) {
    ResultImpl *r = q.r.get();
    const auto *sm = static_cast<const SgSmall *>(q.small.first);
    raise_join_err(sm->err, plan);
    if (sm->flags & 1) {
        CK(cudaMemsetAsync(q.sg.flags, 0, 4, e->compute));
        raise(H2TAP_ENOMEM, "%s: more than %d distinct o_ol_cnt groups", plan, kSgSlots + kSgDense);
    }
    const uint64_t ng = sm->ngroups;
    r->nrows = ng;
    struct { const char *name; uint32_t type; const void *src; size_t es; } cols[] = {
        {"o_ol_cnt", H2TAP_I32, q.sg.o_key, 4}, {a_name, H2TAP_I64, q.sg.o_a, 8}, {b_name, H2TAP_I64, q.sg.o_b, 8}};
    const int ncols = b_name ? 3 : 2;
    if (r->on_device) {
        for (int i = 0; i < ncols; ++i) add_col(r, cols[i].name, cols[i].type, cols[i].src);
        give_blocks_to_result(q);
        return;
    }
    for (int i = 0; i < ncols; ++i) {
        void *dst = result_block(r, ng * cols[i].es);
        if (ng) CK(cudaMemcpyAsync(dst, cols[i].src, ng * cols[i].es, cudaMemcpyDeviceToHost, e->compute));
        add_col(r, cols[i].name, cols[i].type, dst);
    }
    sync_compute(e);
    release_dev_blocks(e, q);
}

// CH-benCHmark constants as int64 µs UTC / cents (R4, R6).
constexpr int64_t kQ1Cutoff = 1167696000000000LL;   // 2007-01-02 00:00:00
constexpr int64_t kQ6DLo = 915148800000000LL;       // 1999-01-01 00:00:00
constexpr int64_t kQ6DHi = 1577836800000000LL;      // 2020-01-01 00:00:00
constexpr int64_t kQ18Having = 20000;               // 200.00
constexpr int64_t kQ14DLo = 1167696000000000LL;     // 2007-01-02 00:00:00
constexpr int64_t kQ14DHi = 1577923200000000LL;     // 2020-01-02 00:00:00
constexpr int64_t kQ14Prefix = 0x5052;              // 'P' << 8 | 'R'  (LIKE 'PR%')
constexpr int64_t kQ12DHi = 1577836800000000LL;     // 2020-01-01 00:00:00
constexpr int64_t kQ4ELo = 1167696000000000LL;      // 2007-01-02 00:00:00
constexpr int64_t kQ4EHi = 1325462400000000LL;      // 2012-01-02 00:00:00
constexpr int64_t kQ3ELo = 1167696000000000LL;      // 2007-01-02 00:00:00
constexpr int64_t kQ3Prefix = 0x4100;               // 'A' << 8  (LIKE 'A%')

h2tap_status parse_query(const h2tap_query &in, QueryCtx &q) {
    uint32_t want;
    switch (in.plan_id) {
        case H2TAP_Q1: want = 1; q.p[0] = kQ1Cutoff; break;
        case H2TAP_Q6: want = 4; q.p[0] = kQ6DLo; q.p[1] = kQ6DHi; q.p[2] = 1; q.p[3] = 100000; break;
        case H2TAP_Q18: want = 1; q.p[0] = kQ18Having; break;
        case H2TAP_Q14: want = 3; q.p[0] = kQ14DLo; q.p[1] = kQ14DHi; q.p[2] = kQ14Prefix; break;
        case H2TAP_Q12: want = 1; q.p[0] = kQ12DHi; break;
        case H2TAP_Q4: want = 2; q.p[0] = kQ4ELo; q.p[1] = kQ4EHi; break;
        case H2TAP_Q3: want = 2; q.p[0] = kQ3ELo; q.p[1] = kQ3Prefix; break;
        default: return fail(H2TAP_EINVAL, "unknown plan id %u", in.plan_id);
    }
    if (in.nparams) {
        if (in.nparams != want || !in.params)
            return fail(H2TAP_EINVAL, "plan %u takes %u params, got %u", in.plan_id, want, in.nparams);
        std::memcpy(q.p, in.params, sizeof(int64_t) * want);
    }
    if (in.plan_id == H2TAP_Q3 && (q.p[1] < 0 || q.p[1] > 0xffff || ((q.p[1] & 0xff) && !(q.p[1] & 0xff00))))
        return fail(H2TAP_EINVAL, "Q3: prefix must be (c0 << 8) | c1 with c0 != 0 when c1 != 0");
    q.plan = in.plan_id;
    q.flags = in.flags;
    return H2TAP_OK;
}

// Plans sharing scratch: Q3 runs on Q18's join scratch and ORDER BY buffers.
uint32_t scratch_group(uint32_t plan) { return plan == H2TAP_Q3 ? (uint32_t)H2TAP_Q18 : plan; }

h2tap_status queries_impl(h2tap_engine *e, const h2tap_query *qs, uint32_t n, h2tap_result **out) {
    const auto t0 = std::chrono::steady_clock::now();
    if (!out || (n && !qs)) return fail(H2TAP_EINVAL, "queries/out is NULL");
    for (uint32_t i = 0; i < n; ++i) out[i] = nullptr;
    std::vector<QueryCtx> ctx(n);
    for (uint32_t i = 0; i < n; ++i) {
        const h2tap_status st = parse_query(qs[i], ctx[i]);
        if (st != H2TAP_OK) return st;
    }
    std::lock_guard<std::mutex> g(e->query_mu);
    CK(cudaSetDevice(e->device));
    if (e->world > 1 && (!e->peer.connected || e->peer.broken))
        return fail(H2TAP_EPEER, e->peer.broken ? "the peer group failed earlier (close and re-open the engines)"
                                                : "world > 1: call h2tap_peer_connect / h2tap_peer_connect_local first");
    publish_ready(e, false);
    ViewP v;
    {
        std::lock_guard<std::mutex> gv(e->view_mu);
        v = e->published;
    }
    if (!v) return fail(H2TAP_EPLAN, "no snapshot has been published yet");
    {   // shared scan: one Q6 followed by one Q1 in the batch, both on the TMA
        // path: the Q6 launch runs one pass over Q1's columns that serves both queries
        int i6 = -1, i1 = -1, n6 = 0, n1 = 0;
        for (uint32_t i = 0; i < n; ++i) {
            if (ctx[i].plan == H2TAP_Q6) { i6 = (int)i; ++n6; }
            if (ctx[i].plan == H2TAP_Q1) { i1 = (int)i; ++n1; }
        }
        const int OL = H2TAP_T_ORDER_LINE;
        const bool cols = v->n[OL] && v->col[OL][H2TAP_OL_NUMBER] && v->col[OL][H2TAP_OL_DELIVERY_D] &&
                          v->col[OL][H2TAP_OL_QUANTITY] && v->col[OL][H2TAP_OL_AMOUNT];
        if (e->shared_scan && n6 == 1 && n1 == 1 && i6 < i1 && cols &&
            scan_tma_ok(e, *v, {H2TAP_OL_NUMBER, H2TAP_OL_DELIVERY_D, H2TAP_OL_QUANTITY, H2TAP_OL_AMOUNT})) {
            ctx[i6].shared_scan = 1;
            ctx[i6].shared_cutoff = ctx[i1].p[0];
            ctx[i1].shared_scan = 2;
            // the full pass: one Q18 after them, and no Q3 (it shares Q18's
            // scratch, which the pass fills ahead of Q18's own launch) — Q18's probe joins the pass
            int i18 = -1, n18 = 0, n3 = 0;
            for (uint32_t i = 0; i < n; ++i) {
                if (ctx[i].plan == H2TAP_Q18) { i18 = (int)i; ++n18; }
                if (ctx[i].plan == H2TAP_Q3) ++n3;
            }
            if (e->full_pass && n18 == 1 && n3 == 0 && i18 > i1 && v->col[OL][H2TAP_OL_W_ID] &&
                v->col[OL][H2TAP_OL_D_ID] && v->col[OL][H2TAP_OL_O_ID] &&
                scan_tma_ok(e, *v, {H2TAP_OL_W_ID, H2TAP_OL_D_ID, H2TAP_OL_O_ID}))
                ctx[i6].full18 = &ctx[i18];
        }
    }
    bool profile = false;
    for (auto &q : ctx) profile |= (q.flags & H2TAP_QUERY_PROFILE) != 0;
    e->prof.reset(profile, e->compute);
    // with per-kernel profiling, a short gate lets the whole batch be enqueued before the GPU
    // starts it, so no kernel's event window contains host launch latency
    static const unsigned long long gate_ns = [] {  // H2TAP_PROFILE_GATE_US (default 30)
        const char *v = std::getenv("H2TAP_PROFILE_GATE_US");
        return (unsigned long long)((v ? std::atof(v) : 30.0) * 1000.0);
    }();
    if (profile) launch_gate(gate_ns, e->compute);
    // with world > 1, profiling also aligns the ranks first (a data-less collective): the per-kernel
    // windows then hold each merge's own cost, not the host-side skew between the ranks' launches
    if (profile && e->world > 1)
        launch_peer_allreduce_i64(e->peer.args, nullptr, 0, nullptr, nullptr, e->compute);
    struct Cleanup {  // return pooled blocks of queries that did not complete
        h2tap_engine *e; std::vector<QueryCtx> &c;
        ~Cleanup() {
            bool pending = false;
            for (auto &q : c) pending |= !q.dev_blocks.empty() || q.small.first;
            if (pending) {  // kernels may still use the blocks
                cudaStreamSynchronize(e->side);
                cudaStreamSynchronize(e->compute);
            }
            for (auto &q : c) {
                release_dev_blocks(e, q);
                if (q.small.first) e->host_pool->put(q.small.first, q.small.second);
            }
        }
    } cleanup{e, ctx};
    // launch phase: a plan's scratch is reused by a later query of the same plan, so a repeated
    // plan first completes the queries launched before it
    size_t done = 0;
    bool forked = false;
    auto join_side = [&] {
        if (!forked) return;
        CK(cudaEventRecord(e->ev_join, e->side));
        CK(cudaStreamWaitEvent(e->compute, e->ev_join, 0));
        forked = false;
    };
    auto finish_upto = [&](size_t upto) {
        if (done >= upto) return;
        join_side();
        sync_compute(e);
        if (e->world > 1 && *reinterpret_cast<volatile unsigned int *>(e->peer.err_host)) {
            e->peer.broken = true;
            const volatile unsigned int *d = e->peer.err_host;
            raise(H2TAP_EPEER, "rank %d: rank %u did not deliver cross-GPU merge #%u within %.0f ms (its "
                  "flag here: %u)", e->rank, d[2], d[1], e->peer.args.timeout_ns / 1e6, d[3]);
        }
        for (; done < upto; ++done) {
            QueryCtx &q = ctx[done];
            switch (q.plan) {
                case H2TAP_Q1: finish_q1(e, q); break;
                case H2TAP_Q6: finish_q6(e, q); break;
                case H2TAP_Q18: case H2TAP_Q3: finish_q18(e, q); break;
                case H2TAP_Q14: finish_q14(e, q); break;
                case H2TAP_Q12: finish_groups(e, q, "Q12", "high_line_count", "low_line_count"); break;
                case H2TAP_Q4: finish_groups(e, q, "Q4", "order_count", nullptr); break;
            }
        }
    };
    CK(cudaEventRecord(e->b_begin, e->compute));
    CK(cudaEventRecord(e->ev_fork, e->compute));  // the batch start (fork point of the side stream)
    for (size_t i = 0; i < ctx.size(); ++i) {
        QueryCtx &q = ctx[i];
        for (size_t j = done; j < i; ++j)
            if (scratch_group(ctx[j].plan) == scratch_group(q.plan)) { finish_upto(i); break; }
        if (!q.r) q.r.reset(new_result(e, *v, q.flags & H2TAP_RESULT_DEVICE));
        if (q.full18 && !q.full18->r)  // the full pass plans Q18's join indexes (plan_flags)
            q.full18->r.reset(new_result(e, *v, q.full18->flags & H2TAP_RESULT_DEVICE));
        q.small = e->host_pool->get(256);
        CK(cudaHostGetDevicePointer(&q.small_dev, q.small.first, 0));
        if (!q.begin) {
            q.begin = e->prof.ev();
            q.end = e->prof.ev();
        }
        q.mark0 = e->prof.marks.size();
        q.launches0 = launches_total();
        // Q18 / Q3 on the side stream (only when something else in the batch could overlap)
        // The tail of a Q1 whose scan ran in the batch's shared pass (compact + emit, two small
        // latency-bound kernels) goes to the side stream, forked right after that pass, when more
        // queries follow: it overlaps the next query's first kernels instead of delaying them
        // (one GPU only: with world > 1 every collective must stay in one stream order, the same
        // on every rank, because their sequence numbers come from one device counter)
        const bool q1_tail = e->q1_side && e->world == 1 && q.plan == H2TAP_Q1 && q.shared_scan == 2 &&
                             i + 1 < ctx.size() && !forked;
        const bool on_side = q1_tail || (e->q18_side && n > 1 && (q.plan == H2TAP_Q18 || q.plan == H2TAP_Q3));
        if (q1_tail) {  // fork point: now (the compute stream's last work is the shared scan)
            CK(cudaEventRecord(e->ev_fork, e->compute));
            CK(cudaStreamWaitEvent(e->side, e->ev_fork, 0));
            forked = true;
        } else if (on_side && !forked) {  // fork from the batch start: the side work need not
                                          // wait for the queries enqueued before it
            CK(cudaStreamWaitEvent(e->side, e->ev_fork, 0));
            forked = true;
        }
        struct SideSwap {  // launch this query's work on the side stream (scratch ordered there)
            h2tap_engine *e; bool on;
            SideSwap(h2tap_engine *x, bool o) : e(x), on(o) { if (on) swap(); }
            ~SideSwap() { if (on) swap(); }
            void swap() {
                std::swap(e->compute, e->side);
                e->arena.owner = e->compute;
                e->prof.st = e->compute;
            }
        } side_swap(e, on_side);
        CK(cudaEventRecord(q.begin, e->compute));
        switch (q.plan) {
            case H2TAP_Q1: launch_q1_plan(e, *v, q); break;
            case H2TAP_Q6: launch_q6_plan(e, *v, q); break;
            case H2TAP_Q18: launch_q18_plan(e, *v, q); break;
            case H2TAP_Q3: launch_q3_plan(e, *v, q); break;
            case H2TAP_Q14: launch_q14_plan(e, *v, q); break;
            case H2TAP_Q12: launch_q12_plan(e, *v, q); break;
            case H2TAP_Q4: launch_q4_plan(e, *v, q); break;
        }
        CK(cudaEventRecord(q.end, e->compute));
        q.launches = launches_total() - q.launches0;
        q.mark1 = e->prof.marks.size();
    }
    join_side();
    CK(cudaEventRecord(e->b_end, e->compute));  // every kernel of the batch, side stream included
    finish_upto(ctx.size());
    CK(cudaEventElapsedTime(&e->last_batch_ms, e->b_begin, e->b_end));
    const double wall = std::chrono::duration<double, std::milli>(std::chrono::steady_clock::now() - t0).count();
    for (uint32_t i = 0; i < n; ++i) {
        QueryCtx &q = ctx[i];
        ResultImpl *r = q.r.get();
        float ms = 0;
        CK(cudaEventElapsedTime(&ms, q.begin, q.end));
        r->device_ms = ms;
        r->kernel_launches = q.launches;
        for (size_t m = q.mark0; m < q.mark1; ++m) {
            float k = 0;
            CK(cudaEventElapsedTime(&k, e->prof.marks[m].second.first, e->prof.marks[m].second.second));
            r->kname_store.push_back(e->prof.marks[m].first);
            r->kms.push_back(k);
        }
        r->e2e_ms = wall;
        if (!q.dist) r->total_rows = r->nrows;
        e->host_pool->put(q.small.first, q.small.second);
        q.small = {};
    }
    for (uint32_t i = 0; i < n; ++i) {
        ctx[i].r->finish();
        out[i] = ctx[i].r.release();
    }
    return H2TAP_OK;
}

h2tap_status query_impl(h2tap_engine *e, uint32_t plan, const int64_t *params, uint32_t nparams,
                        uint32_t flags, h2tap_result **out) {
    if (!out) return fail(H2TAP_EINVAL, "out is NULL");
    h2tap_query q{plan, nparams, params, flags};
    return queries_impl(e, &q, 1, out);
}

template <class F> h2tap_status guarded(F &&f) {
    try {
        return f();
    } catch (const Fail &x) {
        return x.st;
    } catch (const std::bad_alloc &) {
        return fail(H2TAP_ENOMEM, "host allocation failed");
    } catch (...) {
        return fail(H2TAP_EINVAL, "unexpected internal error");
    }
}

}  // namespace

// ================================================================ ABI ===
extern "C" {

h2tap_status h2tap_open(const h2tap_config *cfg, h2tap_engine **out) {
    return guarded([&]() -> h2tap_status {
        if (!cfg || !out) return fail(H2TAP_EINVAL, "cfg/out is NULL");
        *out = nullptr;
        if (cfg->world < 1 || cfg->rank < 0 || cfg->rank >= cfg->world)
            return fail(H2TAP_EINVAL, "bad rank %d / world %d", cfg->rank, cfg->world);
        if (cfg->world > kMaxRanks)
            return fail(H2TAP_EINVAL, "world %d > %d ranks (one node)", cfg->world, kMaxRanks);
        int ndev = 0;
        CK(cudaGetDeviceCount(&ndev));
        if (cfg->device < 0 || cfg->device >= ndev)
            return fail(H2TAP_EINVAL, "device %d not present (%d devices)", cfg->device, ndev);
        std::unique_ptr<h2tap_engine> e(new h2tap_engine());
        e->device = cfg->device;
        e->rank = cfg->rank;
        e->world = cfg->world;
        CK(cudaSetDevice(e->device));
        cudaDeviceProp prop;
        CK(cudaGetDeviceProperties(&prop, e->device));
        if (prop.major != 10)
            return fail(H2TAP_ECUDA, "built for sm_100a (B200); device %d is sm_%d%d", e->device,
                        prop.major, prop.minor);
        e->num_sms = prop.multiProcessorCount;
        CK(set_attributes_scan(e->num_sms));  // per device: shared-memory limits of the kernels
        CK(set_attributes_join(e->num_sms));
        CK(set_attributes_sort(e->num_sms));
        CK(set_attributes_ch(e->num_sms));
        CK(set_attributes_layout(e->num_sms));
        CK(set_attributes_store(e->num_sms));
        CK(set_attributes_peer(e->num_sms));
        if (const char *impl = std::getenv("H2TAP_SCAN")) e->scan_tma = std::strcmp(impl, "ldg") != 0;
        if (const char *ob = std::getenv("H2TAP_ORDER")) e->order_v1 = std::strcmp(ob, "v1") == 0;
        if (const char *z = std::getenv("H2TAP_ZC_TMA")) e->zc_tma = std::atoi(z) != 0;
        if (const char *hu = std::getenv("H2TAP_HAVING_UNROLL")) e->having_unroll = std::atoi(hu) == 4 ? 4 : 2;
        if (const char *ss = std::getenv("H2TAP_SHARED_SCAN")) e->shared_scan = std::atoi(ss) != 0;
        if (const char *fp = std::getenv("H2TAP_FULL_PASS")) e->full_pass = std::atoi(fp) != 0;
        if (const char *impl = std::getenv("H2TAP_PROBE")) e->probe_tma = std::strcmp(impl, "tma") == 0;
        if (const char *impl = std::getenv("H2TAP_COW")) e->cow_full = std::strcmp(impl, "full") == 0;

        CK(cudaStreamCreateWithFlags(&e->compute, cudaStreamNonBlocking));
        {   // the refresh stream at the highest priority: its kernels (zone maps, copy-on-write) are
            // scheduled ahead of queued query blocks as SM slots free up, so a refresh under a
            // saturating query loop (config C5) does not wait behind whole query kernels
            // (H2TAP_COPY_PRIORITY=0: default priority, A/B)
            int lo = 0, hi = 0;
            CK(cudaDeviceGetStreamPriorityRange(&lo, &hi));
            const char *cp = std::getenv("H2TAP_COPY_PRIORITY");
            CK(cudaStreamCreateWithPriority(&e->copy, cudaStreamNonBlocking, (cp && cp[0] == '0') ? lo : hi));
        }
        CK(cudaStreamCreateWithFlags(&e->side, cudaStreamNonBlocking));
        CK(cudaEventCreateWithFlags(&e->ev_fork, cudaEventDisableTiming));
        CK(cudaEventCreateWithFlags(&e->ev_join, cudaEventDisableTiming));
        if (const char *q = std::getenv("H2TAP_Q18_STREAM")) e->q18_side = std::atoi(q) != 0;
        if (const char *q = std::getenv("H2TAP_Q1_SIDE")) e->q1_side = std::atoi(q) != 0;
        CK(cudaStreamCreateWithFlags(&e->reaper, cudaStreamNonBlocking));
        CK(cudaMalloc(&e->pages_dev, 8));
        CK(cudaMemset(e->pages_dev, 0, 8));
        e->free_order = FreeOrder{e->compute, e->copy, e->reaper};
        {   // keep freed pool memory cached (no release to the OS at stream syncs)
            cudaMemPool_t pool;
            CK(cudaDeviceGetDefaultMemPool(&pool, e->device));
            uint64_t thr = UINT64_MAX;
            CK(cudaMemPoolSetAttribute(pool, cudaMemPoolAttrReleaseThreshold, &thr));
            // never let an allocation on the copy stream wait for a pending free (that free waits
            // for queries on the compute stream: refreshes would serialise behind queries, C5
            // measured 8 -> 101 ms per refresh); reuse only memory whose free has completed
            int no = 0;
            CK(cudaMemPoolSetAttribute(pool, cudaMemPoolReuseAllowInternalDependencies, &no));
        }
        CK(cudaEventCreate(&e->q_begin));
        CK(cudaEventCreate(&e->q_end));
        CK(cudaEventCreate(&e->b_begin));
        CK(cudaEventCreate(&e->b_end));
        CK(cudaMallocHost(&e->small_host, 256));
        e->arena.device = e->device;
        e->load_arena.device = e->device;
        e->arena.owner = e->compute;
        e->load_arena.owner = e->copy;
        e->host_pool = std::make_shared<BlockPool>(true, e->device);
        e->dev_pool = std::make_shared<BlockPool>(false, e->device);
        if (e->world > 1) {  // a7: this rank's peer segment, zeroed before any peer maps it
            auto &P = e->peer;
            uint64_t heap = cfg->peer_heap_bytes ? cfg->peer_heap_bytes : (1ull << 30);
            const uint64_t half = ((heap / 2) + 255) & ~uint64_t(255);
            P.seg_bytes = kPeerCtlBytes + 2 * kMaxRanks * kPeerSlotBytes + 2 * half;
            CK(cudaMalloc(&P.seg, P.seg_bytes));
            CK(cudaMemset(P.seg, 0, kPeerCtlBytes));
            CK(cudaHostAlloc(&P.err_host, 64, cudaHostAllocMapped));
            *P.err_host = 0;
            CK(cudaDeviceSynchronize());
            P.args = PeerArgs{};
            P.args.rank = e->rank;
            P.args.world = e->world;
            P.args.slot_bytes = kPeerSlotBytes;
            P.args.heap_half = half;
            double ms = 20000.0;
            if (const char *t = std::getenv("H2TAP_PEER_TIMEOUT_MS")) ms = std::atof(t);
            P.args.timeout_ns = (unsigned long long)(ms * 1e6);
            void *dp = nullptr;
            CK(cudaHostGetDevicePointer(&dp, P.err_host, 0));
            P.args.err_host = static_cast<unsigned int *>(dp);
        }
        engines_on_device_add(e->device, 1);
        *out = e.release();
        return H2TAP_OK;
    });
}

h2tap_status h2tap_load_snapshot_ex(h2tap_engine *e, const h2tap_table *tables, uint32_t ntables,
                                    uint64_t epoch, uint32_t flags) {
    if (!e) return fail(H2TAP_EINVAL, "engine is NULL");
    return guarded([&] { return load_impl(e, tables, ntables, nullptr, 0, epoch, flags); });
}

h2tap_status h2tap_reserve(h2tap_engine *e, uint32_t table_id, uint64_t rows) {
    if (!e) return fail(H2TAP_EINVAL, "engine is NULL");
    if (table_id < 1 || table_id >= (uint32_t)kTables) return fail(H2TAP_EINVAL, "unknown table id %u", table_id);
    return guarded([&]() -> h2tap_status {
        std::lock_guard<std::mutex> g(e->load_mu);
        CK(cudaSetDevice(e->device));
        TableState &ts = e->tables[table_id];
        const uint64_t need = rows + kPadRows;
        for (int c = 0; c < kNcols[table_id]; ++c) {
            ColState &cs = ts.col[c];
            if (!cs.cur || cs.cap_rows >= need) continue;
            const size_t es = type_size(kTypes[table_id][c]);
            DevBufP nb = dev_alloc_ordered(need * es, e->device, &e->free_order);
            if (ts.loaded)
                CK(cudaMemcpyAsync(nb->ptr, cs.cur->ptr, ts.loaded * es, cudaMemcpyDeviceToDevice, e->copy));
            cs.alt.reset();
            cs.alt_valid = false;
            cs.cur = nb;  // published views keep the old buffer alive until they retire
            cs.cap_rows = need;
        }
        CK(cudaStreamSynchronize(e->copy));
        return H2TAP_OK;
    });
}

h2tap_status h2tap_refresh(h2tap_engine *e, const h2tap_table *tables, uint32_t ntables,
                           const h2tap_update *updates, uint32_t nupdates, uint64_t epoch,
                           uint32_t flags) {
    if (!e) return fail(H2TAP_EINVAL, "engine is NULL");
    return guarded([&] { return load_impl(e, tables, ntables, updates, nupdates, epoch, flags); });
}

h2tap_status h2tap_get_store_stats(h2tap_engine *e, h2tap_store_stats *out) {
    if (!e || !out) return fail(H2TAP_EINVAL, "NULL argument");
    return guarded([&]() -> h2tap_status {
        std::lock_guard<std::mutex> g(e->load_mu);
        CK(cudaSetDevice(e->device));
        publish_ready(e, false);
        {
            std::lock_guard<std::mutex> gp(e->pend_mu);
            *out = e->sstats;
        }
        {   // the copy-on-write page counter lives on the device (no copy per refresh); the copies of
            // the refreshes published so far are complete (publish waited for their events)
            unsigned long long pages = 0;
            CK(cudaMemcpy(&pages, e->pages_dev, 8, cudaMemcpyDeviceToHost));
            out->cow_pages_copied = pages;
        }
        uint64_t bytes = 0;
        for (auto &t : e->tables)
            for (auto &c : t.col)
                for (const DevBufP *b : {&c.cur, &c.alt, &c.bits, &c.bits_next})
                    if (*b) bytes += (*b)->bytes;
        out->device_bytes = bytes;
        return H2TAP_OK;
    });
}

// ---- NEXT-3 / NEXT-4: SUM(col_1 + ... + col_N) over a DSM / PAX / NSM table (§5.3)
namespace {
int log2_exact(uint64_t x) {
    if (!x || (x & (x - 1))) return -1;
    return 63 - __builtin_clzll(x);
}
}  // namespace

h2tap_status h2tap_layout_sum(h2tap_engine *e, const h2tap_layout_table *t, uint64_t col_mask,
                              int64_t *sum, int32_t *is_null, double *device_ms) {
    if (!e || !t || !sum || !is_null) return fail(H2TAP_EINVAL, "NULL argument");
    if (t->layout < H2TAP_DSM || t->layout > H2TAP_NSM) return fail(H2TAP_EINVAL, "unknown layout %u", t->layout);
    if (t->ncols < 1 || t->ncols > 64) return fail(H2TAP_EINVAL, "ncols must be in [1, 64]");
    const uint64_t all = t->ncols == 64 ? ~0ull : ((1ull << t->ncols) - 1);
    if (!col_mask || (col_mask & ~all)) return fail(H2TAP_EINVAL, "column mask selects no column or one >= ncols");
    const int log_ncols = log2_exact(t->ncols), log_mp = log2_exact(t->pax_rows);
    uint64_t stride = t->col_stride ? t->col_stride : t->nrows;
    if (t->layout != H2TAP_DSM && (log_ncols < 2)) return fail(H2TAP_EINVAL, "PAX/NSM need ncols a power of two >= 4");
    if (t->layout == H2TAP_PAX && log_mp < 2) return fail(H2TAP_EINVAL, "PAX needs pax_rows a power of two >= 4");
    if (t->layout == H2TAP_DSM && stride < t->nrows) return fail(H2TAP_EINVAL, "DSM col_stride must be >= nrows");
    if (t->layout == H2TAP_PAX && log_mp >= 2 &&
        ((t->nrows + t->pax_rows - 1) >> log_mp) * (uint64_t)__builtin_popcountll(col_mask) >= (1ull << 32))
        return fail(H2TAP_EINVAL, "PAX: pages x selected columns must be < 2^32");
    if (t->nrows && (!t->data || (reinterpret_cast<uintptr_t>(t->data) & (t->layout == H2TAP_DSM ? 3 : 15))))
        return fail(H2TAP_EINVAL, "data must be non-NULL and 16-byte aligned (4-byte for DSM)");
    return guarded([&]() -> h2tap_status {
        std::lock_guard<std::mutex> g(e->query_mu);
        CK(cudaSetDevice(e->device));
        const int32_t *dptr = static_cast<const int32_t *>(t->data);
        if (t->nrows) {
            // device memory, or pinned host memory reached through its mapped (UVA) address: the
            // paper's zero-copy GPU access to host data (L568-572); pageable memory is refused
            cudaPointerAttributes a{};
            CK(cudaPointerGetAttributes(&a, t->data));
            if (a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged) {
                if (a.device != e->device) raise(H2TAP_EINVAL, "data lives on device %d, engine on %d", a.device, e->device);
            } else if (a.type == cudaMemoryTypeHost) {
                if (!a.devicePointer) raise(H2TAP_EINVAL, "pinned host data is not mapped into the device address space");
                dptr = static_cast<const int32_t *>(a.devicePointer);
            } else {
                raise(H2TAP_EINVAL, "data is pageable host memory: pin it (cudaHostAlloc / cudaHostRegister)");
            }
        }
        LayoutSel sel{};
        for (int c = 0; c < 64; ++c)
            if (col_mask >> c & 1) sel.col[sel.n++] = c;
        auto *acc = static_cast<unsigned long long *>(e->arena.get("layout.acc", 64));
        CK(cudaMemsetAsync(acc, 0, 8, e->compute));
        CK(cudaEventRecord(e->q_begin, e->compute));
        if (t->nrows)
            launch_layout_sum(dptr, (int)t->layout, t->nrows, log_ncols, log_mp, stride, col_mask, sel, acc,
                              e->num_sms, e->compute);
        CK(cudaGetLastError());
        CK(cudaEventRecord(e->q_end, e->compute));
        unsigned long long host = 0;
        CK(cudaMemcpyAsync(e->small_host, acc, 8, cudaMemcpyDeviceToHost, e->compute));
        sync_compute(e);
        std::memcpy(&host, e->small_host, 8);
        float ms = 0;
        CK(cudaEventElapsedTime(&ms, e->q_begin, e->q_end));
        *sum = (int64_t)host;
        *is_null = t->nrows == 0;  // SUM over no rows is NULL
        if (device_ms) *device_ms = ms;
        return H2TAP_OK;
    });
}

h2tap_status h2tap_refresh_rows(h2tap_engine *e, const h2tap_row_table *tables, uint32_t ntables,
                                const h2tap_update *updates, uint32_t nupdates, uint64_t epoch,
                                uint32_t flags) {
    if (!e) return fail(H2TAP_EINVAL, "engine is NULL");
    if (ntables && !tables) return fail(H2TAP_EINVAL, "tables is NULL");
    if (flags & H2TAP_LOAD_ZERO_COPY)
        return fail(H2TAP_EINVAL, "zero-copy needs columns (DSM) in caller-owned pinned memory, not NSM records");
    return guarded([&]() -> h2tap_status {
        // column extraction NSM -> DSM into pinned buffers (the library's pinned block pool)
        std::vector<std::vector<h2tap_column>> cols(ntables);
        std::vector<h2tap_table> tabs(ntables);
        std::vector<std::pair<void *, size_t>> blocks;
        struct Job { const char *src; size_t stride; size_t es; char *dst; uint64_t n; };
        std::vector<Job> jobs;
        struct Release {
            h2tap_engine *e; std::vector<std::pair<void *, size_t>> &b;
            ~Release() { for (auto &x : b) e->host_pool->put(x.first, x.second); }
        } release{e, blocks};
        for (uint32_t t = 0; t < ntables; ++t) {
            const h2tap_row_table &rt = tables[t];
            if (rt.row_count < rt.first_row) return fail(H2TAP_EINVAL, "row_count < first_row");
            const uint64_t n = rt.row_count - rt.first_row;
            if (n && (!rt.records || !rt.fields)) return fail(H2TAP_EINVAL, "records/fields is NULL");
            for (uint32_t f = 0; f < rt.nfields; ++f) {
                const h2tap_field &fd = rt.fields[f];
                const size_t es = fd.type == H2TAP_I32 ? 4 : 8;
                if (fd.offset + es > rt.record_size) return fail(H2TAP_EINVAL, "field outside the record");
                auto b = e->host_pool->get(n * es + 8);
                blocks.push_back(b);
                jobs.push_back(Job{static_cast<const char *>(rt.records) + fd.offset, rt.record_size, es,
                                   static_cast<char *>(b.first), n});
                cols[t].push_back(h2tap_column{fd.column_id, fd.type, b.first});
            }
            tabs[t] = h2tap_table{rt.table_id, rt.nfields, cols[t].data(), rt.row_count, rt.first_row, rt.flags};
        }
        // strided gathers, split over host threads by row ranges
        uint64_t total = 0;
        for (auto &j : jobs) total += j.n;
        const unsigned hw = std::max(1u, std::min(16u, std::thread::hardware_concurrency()));
        const unsigned nthreads = total > (1u << 16) ? hw : 1u;
        auto work = [&](unsigned tid) {
            for (auto &j : jobs) {
                const uint64_t lo = j.n * tid / nthreads, hi = j.n * (tid + 1) / nthreads;
                if (j.es == 4)
                    for (uint64_t i = lo; i < hi; ++i) std::memcpy(j.dst + 4 * i, j.src + i * j.stride, 4);
                else
                    for (uint64_t i = lo; i < hi; ++i) std::memcpy(j.dst + 8 * i, j.src + i * j.stride, 8);
            }
        };
        std::vector<std::thread> pool;
        for (unsigned t = 1; t < nthreads; ++t) pool.emplace_back(work, t);
        work(0);
        for (auto &th : pool) th.join();
        // pinned sources: load_impl DMAs them directly and waits before returning (the extraction
        // buffers are the library's and reused by the next call: never lent)
        return load_impl(e, tabs.data(), ntables, updates, nupdates, epoch, flags & ~H2TAP_LOAD_BORROW);
    });
}

h2tap_status h2tap_load_snapshot_rows(h2tap_engine *e, const h2tap_row_table *tables,
                                      uint32_t ntables, uint64_t epoch, uint32_t flags) {
    return h2tap_refresh_rows(e, tables, ntables, nullptr, 0, epoch, flags);
}

h2tap_status h2tap_load_snapshot(h2tap_engine *e, const h2tap_table *tables, uint32_t ntables,
                                 uint64_t epoch) {
    return h2tap_load_snapshot_ex(e, tables, ntables, epoch, 0);
}

h2tap_status h2tap_sync(h2tap_engine *e, uint64_t *published_epoch) {
    if (!e) return fail(H2TAP_EINVAL, "engine is NULL");
    return guarded([&]() -> h2tap_status {
        CK(cudaSetDevice(e->device));
        publish_ready(e, true);
        std::lock_guard<std::mutex> gv(e->view_mu);
        if (published_epoch) *published_epoch = e->published ? e->published->epoch : 0;
        return H2TAP_OK;
    });
}

h2tap_status h2tap_run_query_ex(h2tap_engine *e, uint32_t plan_id, const int64_t *params,
                                uint32_t nparams, uint32_t flags, h2tap_result **out) {
    if (!e) return fail(H2TAP_EINVAL, "engine is NULL");
    return guarded([&] { return query_impl(e, plan_id, params, nparams, flags, out); });
}

h2tap_status h2tap_run_query(h2tap_engine *e, uint32_t plan_id, const int64_t *params,
                             uint32_t nparams, h2tap_result **out) {
    return h2tap_run_query_ex(e, plan_id, params, nparams, 0, out);
}

h2tap_status h2tap_run_queries(h2tap_engine *e, const h2tap_query *queries, uint32_t nqueries,
                               h2tap_result **out) {
    if (!e) return fail(H2TAP_EINVAL, "engine is NULL");
    return guarded([&] { return queries_impl(e, queries, nqueries, out); });
}

h2tap_status h2tap_last_batch_ms(h2tap_engine *e, double *device_ms) {
    if (!e || !device_ms) return fail(H2TAP_EINVAL, "engine / device_ms is NULL");
    std::lock_guard<std::mutex> g(e->query_mu);
    if (e->last_batch_ms < 0.f) return fail(H2TAP_EPLAN, "no batch has completed on this engine");
    *device_ms = e->last_batch_ms;
    return H2TAP_OK;
}

void h2tap_free(h2tap_result *r) {
    if (!r) return;
    delete static_cast<ResultImpl *>(r);
}

void h2tap_close(h2tap_engine *e) {
    if (!e) return;
    engines_on_device_add(e->device, -1);
    cudaSetDevice(e->device);
    try { publish_ready(e, true); } catch (...) {}
    cudaStreamSynchronize(e->compute);
    cudaStreamSynchronize(e->copy);
    for (void *p : e->peer.opened) cudaIpcCloseMemHandle(p);
    if (e->peer.seg) cudaFree(e->peer.seg);
    if (e->pages_dev) cudaFree(e->pages_dev);
    if (e->peer.err_host) cudaFreeHost(e->peer.err_host);
    for (auto &p : e->pending) {
        for (cudaEvent_t ev : {p.done, p.t0, p.t1, p.t2, p.t3}) cudaEventDestroy(ev);
        e->host_pool->put(p.stats_block.first, p.stats_block.second);
    }
    for (int k = 0; k < Staging::kSlots; ++k) {
        if (e->staging.buf[k]) cudaFreeHost(e->staging.buf[k]);
        if (e->staging.ev[k]) cudaEventDestroy(e->staging.ev[k]);
    }
    for (auto ev : e->prof.pool) cudaEventDestroy(ev);
    cudaEventDestroy(e->q_begin);
    cudaEventDestroy(e->q_end);
    cudaEventDestroy(e->b_begin);
    cudaEventDestroy(e->b_end);
    cudaFreeHost(e->small_host);
    e->published.reset();
    e->accepted.reset();
    for (auto &t : e->tables) for (auto &c : t.col) { c.cur.reset(); c.alt.reset(); c.bits.reset(); c.bits_next.reset(); }
    e->arena.release();
    e->load_arena.release();
    cudaStreamSynchronize(e->compute);
    cudaStreamSynchronize(e->copy);
    cudaStreamSynchronize(e->reaper);
    cudaStreamDestroy(e->compute);
    cudaStreamDestroy(e->copy);
    cudaStreamSynchronize(e->side);
    cudaStreamDestroy(e->side);
    cudaEventDestroy(e->ev_fork);
    cudaEventDestroy(e->ev_join);
    cudaStreamDestroy(e->reaper);
    delete e;
}

const char *h2tap_last_error(void) { return g_err.c_str(); }

h2tap_status h2tap_peer_handle(h2tap_engine *e, void *out64) {
    return guarded([&]() -> h2tap_status {
        if (!e || !out64) return fail(H2TAP_EINVAL, "engine/out is NULL");
        if (e->world < 2) return fail(H2TAP_EINVAL, "world == 1: no peer segment");
        CK(cudaSetDevice(e->device));
        cudaIpcMemHandle_t h;
        static_assert(sizeof(cudaIpcMemHandle_t) == 64, "CUDA IPC handles are 64 bytes");
        CK(cudaIpcGetMemHandle(&h, e->peer.seg));
        std::memcpy(out64, &h, 64);
        return H2TAP_OK;
    });
}

h2tap_status h2tap_peer_connect(h2tap_engine *e, const void *handles, uint32_t world) {
    return guarded([&]() -> h2tap_status {
        if (!e || !handles) return fail(H2TAP_EINVAL, "engine/handles is NULL");
        if ((int)world != e->world || e->world < 2) return fail(H2TAP_EINVAL, "world %u != engine world %d", world, e->world);
        if (e->peer.connected) return fail(H2TAP_EINVAL, "peers already connected");
        CK(cudaSetDevice(e->device));
        auto &P = e->peer;
        for (int k = 0; k < e->world; ++k) {
            if (k == e->rank) { P.args.seg[k] = P.seg; continue; }
            cudaIpcMemHandle_t h;
            std::memcpy(&h, static_cast<const char *>(handles) + 64 * k, 64);
            void *p = nullptr;
            CK(cudaIpcOpenMemHandle(&p, h, cudaIpcMemLazyEnablePeerAccess));
            P.opened.push_back(p);
            P.args.seg[k] = static_cast<char *>(p);
        }
        P.connected = true;
        return H2TAP_OK;
    });
}

h2tap_status h2tap_peer_connect_local(h2tap_engine *const *engines, uint32_t n) {
    return guarded([&]() -> h2tap_status {
        if (!engines || n < 2 || n > (uint32_t)kMaxRanks) return fail(H2TAP_EINVAL, "need 2..%d engines", kMaxRanks);
        for (uint32_t i = 0; i < n; ++i) {
            if (!engines[i]) return fail(H2TAP_EINVAL, "engine %u is NULL", i);
            if (engines[i]->rank != (int)i || engines[i]->world != (int)n)
                return fail(H2TAP_EINVAL, "engine %u has rank %d / world %d (want %u / %u)", i, engines[i]->rank,
                            engines[i]->world, i, n);
            if (engines[i]->peer.connected) return fail(H2TAP_EINVAL, "engine %u already connected", i);
        }
        for (uint32_t i = 0; i < n; ++i) {
            h2tap_engine *e = engines[i];
            CK(cudaSetDevice(e->device));
            for (uint32_t k = 0; k < n; ++k) {
                if (engines[k]->device != e->device) {  // another GPU of this process: peer access
                    const cudaError_t r = cudaDeviceEnablePeerAccess(engines[k]->device, 0);
                    if (r == cudaErrorPeerAccessAlreadyEnabled) cudaGetLastError();
                    else CK(r);
                }
                e->peer.args.seg[k] = engines[k]->peer.seg;
            }
        }
        for (uint32_t i = 0; i < n; ++i) {
            int shared = 0;
            for (uint32_t k = 0; k < n; ++k) shared |= (k != i && engines[k]->device == engines[i]->device);
            engines[i]->peer.args.shared_device = shared;
            engines[i]->peer.connected = true;
        }
        return H2TAP_OK;
    });
}

h2tap_status h2tap_compute_stream(h2tap_engine *e, void **stream) {
    if (!e || !stream) return fail(H2TAP_EINVAL, "NULL argument");
    *stream = e->compute;
    return H2TAP_OK;
}

int h2tap_c_last_name(int32_t code, char *buf, size_t buflen) {
    // TPC-C 4.3.2.3: C_LAST is the concatenation of the syllables of the three digits of code
    static const char *syl[10] = {"BAR", "OUGHT", "ABLE", "PRI", "PRES",
                                  "ESE", "ANTI", "CALLY", "ATION", "EING"};
    if (code < 0 || code > 999 || !buf) return -1;
    const int n = snprintf(buf, buflen, "%s%s%s", syl[code / 100], syl[(code / 10) % 10], syl[code % 10]);
    return (n < 0 || (size_t)n >= buflen) ? -1 : n;
}

}  // extern "C"
