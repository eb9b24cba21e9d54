// ch_kernels.cu — NEXT-2: CH-benCHmark Q14, Q12 and Q4 on the same snapshot,
// join index and aggregation machinery as the hot path, for sm_100a.
//
//  Q14  order_line ⋈ item: one fused scan of (delivery 8 B, i_id 4 B, amount 8 B) per row with
//       the item side as a 2-bit-per-id map (exists, i_data LIKE 'PR%') held in shared memory
//       (25 KB for TPC-C's 100 000 items); int64 sums, last-block fold, promo ratio in double.
//  Q12  orders ⋈ order_line GROUP BY o_ol_cnt: stream (w, d, o, delivery) per line, one lookup of
//       the orders join index per run of equal keys inside a lane, gather (entry, carrier,
//       ol_cnt), count per group in thread-private 16-bit shared-memory counters.
//  Q4   orders ⋉ order_line (EXISTS): the same stream marks orders rows that have a qualifying
//       line (idempotent byte store), then one pass over orders counts marked rows per o_ol_cnt.
// The paper gives no plans for these queries (it evaluates TPC-H Q6 only);
// like the hot path they run on an epoch's snapshot (L555-572). DESIGN.md §4.8.
#include <algorithm>
#include <cstdint>
#include <cuda_runtime.h>

#include "join_index.cuh"
#include "kernels.cuh"
#include "peer.cuh"

namespace h2tap {
namespace {
using namespace jx;

constexpr unsigned kFull = 0xffffffffu;
constexpr int kThreads = 256;

__device__ __forceinline__ long long warp_sum64(long long v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
    return v;
}

unsigned grid_for(uint64_t work, int threads, int num_sms, int per_sm) {
    uint64_t want = (work + threads - 1) / threads;
    const uint64_t cap = (uint64_t)num_sms * per_sm;
    if (want > cap) want = cap;
    return want ? (unsigned)want : 1u;
}

// ============================================================ small groups ==
// GROUP BY o_ol_cnt with three counters per group (a, b, rows). Per warp step the lanes with a
// contribution are grouped by key (__match_any_sync); one leader per distinct key adds the
// group's popcounts to the block's shared counters (keys in [0, kSgDense)) or to a global
// open-addressing table (other keys; TPC-C never produces them). The block's counters are folded
// into g.dense once at the end. Shared memory stays tiny, so occupancy is not limited by it.
struct SgSmem {
    unsigned int c[kSgDense][3];
};

__device__ __forceinline__ unsigned int hash32(unsigned int x) {
    x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16;
    return x;
}

__device__ void sg_global_add(const SmallGroups &g, int key, unsigned long long a, unsigned long long b,
                              unsigned long long rows) {
    const unsigned long long tag = (1ull << 32) | (unsigned int)key;
    unsigned int h = hash32((unsigned int)key) & (kSgSlots - 1);
    for (int p = 0; p < kSgSlots; ++p) {
        const unsigned long long prev = atomicCAS(g.gtag + h, 0ull, tag);
        if (prev == 0ull || prev == tag) {
            if (a) atomicAdd(g.gacc + 3 * h + 0, a);
            if (b) atomicAdd(g.gacc + 3 * h + 1, b);
            atomicAdd(g.gacc + 3 * h + 2, rows);
            return;
        }
        h = (h + 1) & (kSgSlots - 1);
    }
    atomicOr(g.flags, 1u);  // more distinct groups than kSgSlots: reported as ENOMEM
}

__device__ __forceinline__ void sg_clear(SgSmem &S) {
    for (int i = threadIdx.x; i < 3 * kSgDense; i += blockDim.x) (&S.c[0][0])[i] = 0;
}

// Warp-collective: every lane calls it (ok = this lane contributes a row to group `key`, with
// flags a and b). One shared (or global) update per distinct key of the warp.
__device__ __forceinline__ void sg_warp_add(SgSmem &S, const SmallGroups &g, bool ok, int key, bool a, bool b) {
    const unsigned okm = __ballot_sync(kFull, ok);
    if (!okm) return;
    const unsigned am = __ballot_sync(kFull, ok && a), bm = __ballot_sync(kFull, ok && b);
    if (!ok) return;
    const unsigned grp = __match_any_sync(okm, key);
    if ((int)(threadIdx.x & 31) != __ffs(grp) - 1) return;
    const unsigned na = __popc(grp & am), nb = __popc(grp & bm), nr = __popc(grp);
    if ((unsigned)key < (unsigned)kSgDense) {
        if (na) atomicAdd(&S.c[key][0], na);
        if (nb) atomicAdd(&S.c[key][1], nb);
        atomicAdd(&S.c[key][2], nr);
    } else {
        sg_global_add(g, key, na, nb, nr);
    }
}

// Thread-private variant for the probe (Q12): c[counter][key][thread] in 16-bit counters (a thread
// sees at most 2^31 / (148 * 8 * 256) < 65 536 rows), lane-distinct halves of a word, no atomics.
struct SgPriv {
    unsigned short c[3][kSgDense][kThreads];
};
__device__ __forceinline__ void sgp_clear(SgPriv &P) {
    unsigned int *p = reinterpret_cast<unsigned int *>(&P.c[0][0][0]);
    for (int i = threadIdx.x; i < 3 * kSgDense * kThreads / 2; i += blockDim.x) p[i] = 0;
}
__device__ __forceinline__ void sgp_add(SgPriv &P, const SmallGroups &g, int key, bool a, bool b) {
    if ((unsigned)key < (unsigned)kSgDense) {
        P.c[0][key][threadIdx.x] += a;
        P.c[1][key][threadIdx.x] += b;
        P.c[2][key][threadIdx.x] += 1;
    } else {
        sg_global_add(g, key, a, b, 1);
    }
}
// warp r sums counter row r (over the 256 threads), one 64-bit atomic per non-zero row
__device__ void sgp_flush(SgPriv &P, const SmallGroups &g) {
    __syncthreads();
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    for (int r = warp; r < 3 * kSgDense; r += blockDim.x / 32) {
        const unsigned short *row = &P.c[r / kSgDense][r % kSgDense][0];
        long long v = 0;
        for (int t = lane; t < kThreads; t += 32) v += row[t];
        v = warp_sum64(v);
        if (lane == 0 && v) atomicAdd(g.dense + (r % kSgDense) * 3 + r / kSgDense, (unsigned long long)v);
    }
}

// fold the block's counters into g.dense: one 64-bit atomic per non-zero (key, counter)
__device__ void sg_flush(SgSmem &S, const SmallGroups &g) {
    __syncthreads();
    for (int i = threadIdx.x; i < 3 * kSgDense; i += blockDim.x) {
        const unsigned v = (&S.c[0][0])[i];
        if (v) atomicAdd(g.dense + i, (unsigned long long)v);
    }
}

__global__ void sg_reset_kernel(SmallGroups g) {
    for (int i = blockIdx.x * blockDim.x + threadIdx.x; i < kSgSlots * 4 + 3 * kSgDense;
         i += gridDim.x * blockDim.x) {
        if (i < kSgSlots) g.gtag[i] = 0;
        else if (i < 4 * kSgSlots) g.gacc[i - kSgSlots] = 0;
        else g.dense[i - 4 * kSgSlots] = 0;
    }
    if (blockIdx.x == 0 && threadIdx.x == 0) *g.flags = 0;
}

// One block: collect the groups (dense keys with rows > 0, occupied global slots), rank them by
// key, write the output columns and the group count, then clear the tables for the next query.
constexpr int kEmitThreads = 1024;
constexpr int kSgMax = kSgSlots + kSgDense;
__global__ void __launch_bounds__(kEmitThreads) sg_emit_kernel(SmallGroups g) {
    __shared__ int key[kSgMax];
    __shared__ unsigned long long va[kSgMax], vb[kSgMax];
    __shared__ unsigned int n;
    if (threadIdx.x == 0) n = 0;
    __syncthreads();
    for (int i = threadIdx.x; i < kSgMax; i += blockDim.x) {
        int k;
        unsigned long long a, b, rows;
        if (i < kSgDense) {
            k = i; a = g.dense[3 * i]; b = g.dense[3 * i + 1]; rows = g.dense[3 * i + 2];
        } else {
            const unsigned long long t = g.gtag[i - kSgDense];
            k = (int)(unsigned int)t;
            a = g.gacc[3 * (i - kSgDense)]; b = g.gacc[3 * (i - kSgDense) + 1];
            rows = t ? g.gacc[3 * (i - kSgDense) + 2] : 0;
        }
        if (rows) {  // a group exists iff at least one row reached it
            const unsigned int s = atomicAdd(&n, 1u);
            key[s] = k; va[s] = a; vb[s] = b;
        }
    }
    __syncthreads();
    const unsigned int m = n;
    for (unsigned int i = threadIdx.x; i < m; i += blockDim.x) {
        unsigned int r = 0;  // keys are distinct: rank = number of smaller keys
        for (unsigned int j = 0; j < m; ++j) r += key[j] < key[i];
        g.o_key[r] = key[i];
        g.o_a[r] = (long long)va[i];
        g.o_b[r] = (long long)vb[i];
    }
    if (threadIdx.x == 0) *g.ngroups = m;
    for (int i = threadIdx.x; i < kSgSlots * 4 + 3 * kSgDense; i += blockDim.x) {  // self-clean
        if (i < kSgSlots) g.gtag[i] = 0;
        else if (i < 4 * kSgSlots) g.gacc[i - kSgSlots] = 0;
        else g.dense[i - 4 * kSgSlots] = 0;
    }
}

// multi-GPU: fold another rank's (dense + sparse) tables into this rank's
// Multi-GPU (a7): every rank pushed its whole table (dense | gtag | gacc, launch_peer_push) into
// this rank's mailbox (arrival awaited by launch_peer_wait); fold the OTHER ranks' tables into the
// local one.
__global__ void sg_peer_merge_kernel(PeerArgs p, SmallGroups g) {
    pdl_wait();
    pdl_trigger();
    const unsigned long long seq = peer::cur_seq(p);
    const int i = blockIdx.x * blockDim.x + threadIdx.x;
    for (int k = 0; k < p.world; ++k) {
        if (k == p.rank) continue;
        const unsigned long long *t = reinterpret_cast<const unsigned long long *>(
            peer::mbox(p, p.rank, (int)(seq & 1), k) + 16);
        const unsigned long long *dense = t, *gtag = t + 3 * kSgDense, *gacc = gtag + kSgSlots;
        if (i < 3 * kSgDense) {
            const unsigned long long v = __ldcg(dense + i);
            if (v) atomicAdd(g.dense + i, v);
        } else if (i < 3 * kSgDense + kSgSlots) {
            const int s = i - 3 * kSgDense;
            const unsigned long long tg = __ldcg(gtag + s);
            if (tg) sg_global_add(g, (int)(unsigned int)tg, __ldcg(gacc + 3 * s), __ldcg(gacc + 3 * s + 1),
                                  __ldcg(gacc + 3 * s + 2));
        }
    }
}

// ========================================================= orders index ==
// Clustered orders (as for Q18): count the rows not at their own dense slot; 0 =
// the index is the identity and nothing is cleared or built. Resets the next query's counter.
__global__ void jx_verify_kernel(JoinIndex j, const int32_t *__restrict__ w, const int32_t *__restrict__ d,
                                 const int32_t *__restrict__ id, uint64_t n) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    const uint64_t n_pad = (n + 31) & ~31ull;
    for (uint64_t r = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; r < n_pad; r += stride) {
        unsigned long long s = 0;
        const bool bad = r < n && (!dense_slot(j, __ldcs(w + r), __ldcs(d + r), __ldcs(id + r), s) || s != r);
        const unsigned int b = __ballot_sync(kFull, bad);
        if (b && (threadIdx.x & 31) == __ffs(b) - 1) atomicAdd(j.viol, 1u);
    }
    if (blockIdx.x == 0 && threadIdx.x == 0 && j.viol_next) *j.viol_next = 0u;
}

__global__ void jx_clear_kernel(JoinIndex j) {
    if (jx_identity(j)) return;  // positional: the slots are never read
    const uint64_t words = jx_words(j);
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < words;
         i += (uint64_t)gridDim.x * blockDim.x)
        jx_clear(j, i);
}

__global__ void jx_build_orders_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                                       const int32_t *__restrict__ o_id, uint64_t n, JoinIndex j,
                                       unsigned int *err, uint8_t *mark) {
    const bool ident = jx_identity(j);
    if (ident && !mark) return;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (uint64_t)gridDim.x * blockDim.x) {
        if (mark) mark[i] = 0;
        if (!ident && !jx_insert(j, o_w[i], o_d[i], o_id[i], (unsigned int)i, err, kErrDupOrders))
            atomicOr(err, kErrDomain);
    }
}

// ======================================================= Q12 / Q4 probes ==
// Each lane owns 4 consecutive order_line rows (128-bit loads of w, d, o, two of delivery). The
// lane first issues the orders-index lookups of every run start among its 4 rows (independent
// loads, all in flight together; lines of an order are adjacent so ~1.4 per lane), then the
// gathers of the looked-up rows' fields, then evaluates — two memory round trips per 4 rows
// instead of one chain per row.
struct OrderCols { const int64_t *entry; const int32_t *carrier, *cnt; };

// fn(row[4], dl[4], valid): called once per lane per 4 rows (warp-uniform; rows past the end
// have valid = false). row[j] = orders row of line j or kNoRow.
template <class Fn>
__device__ __forceinline__ void probe_rows4(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
                                            const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_dl,
                                            uint64_t n, const JoinIndex &jo, Fn &&fn) {
    const uint64_t nvec = n >> 2;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    const unsigned lane = threadIdx.x & 31;
    uint64_t base = (uint64_t)blockIdx.x * blockDim.x + (threadIdx.x & ~31u);
    int4 nW = make_int4(0, 0, 0, 0), nD = nW, nO = nW;
    longlong2 nL0 = make_longlong2(0, 0), nL1 = nL0;
    auto load = [&](uint64_t x) {
        if (x < nvec) {
            nW = __ldcs(reinterpret_cast<const int4 *>(ol_w) + x);
            nD = __ldcs(reinterpret_cast<const int4 *>(ol_d) + x);
            nO = __ldcs(reinterpret_cast<const int4 *>(ol_o) + x);
            nL0 = __ldcs(reinterpret_cast<const longlong2 *>(ol_dl) + 2 * x);
            nL1 = __ldcs(reinterpret_cast<const longlong2 *>(ol_dl) + 2 * x + 1);
        }
    };
    load(base + lane);
    for (; base < nvec; base += stride) {
        const bool valid = base + lane < nvec;
        const int4 W = nW, D = nD, O = nO;
        const long long dl[4] = {nL0.x, nL0.y, nL1.x, nL1.y};
        load(base + stride + lane);  // next group's loads in flight while this one is probed
        const bool s1 = (W.y != W.x) | (D.y != D.x) | (O.y != O.x);
        const bool s2 = (W.z != W.y) | (D.z != D.y) | (O.z != O.y);
        const bool s3 = (W.w != W.z) | (D.w != D.z) | (O.w != O.z);
        unsigned int r[4];
        r[0] = valid ? jx_lookup(jo, W.x, D.x, O.x) : kNoRow;
        r[1] = valid && s1 ? jx_lookup(jo, W.y, D.y, O.y) : kNoRow;
        r[2] = valid && s2 ? jx_lookup(jo, W.z, D.z, O.z) : kNoRow;
        r[3] = valid && s3 ? jx_lookup(jo, W.w, D.w, O.w) : kNoRow;
        if (!s1) r[1] = r[0];
        if (!s2) r[2] = r[1];
        if (!s3) r[3] = r[2];
        fn(r, dl, valid);
    }
    // ragged tail (< 4 rows): the first warp of block 0, one row per lane (warp-uniform call)
    if (blockIdx.x == 0 && threadIdx.x < 32) {
        const uint64_t t = 4 * nvec + lane;
        const bool valid = t < n;
        unsigned int r[4] = {valid ? jx_lookup(jo, ol_w[t], ol_d[t], ol_o[t]) : kNoRow, kNoRow, kNoRow, kNoRow};
        const long long dl[4] = {valid ? ol_dl[t] : 0ll, kNullTs, kNullTs, kNullTs};
        fn(r, dl, valid);
    }
}

__global__ void __launch_bounds__(kThreads)
q12_probe_kernel(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
                 const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_dl, uint64_t n,
                 JoinIndex jo, OrderCols oc, long long d_hi, SmallGroups g) {
    __shared__ SgPriv P;
    sgp_clear(P);
    __syncthreads();
    probe_rows4(ol_w, ol_d, ol_o, ol_dl, n, jo, [&](const unsigned int (&r)[4], const long long (&dl)[4], bool) {
        // gathers of the distinct looked-up rows (independent loads)
        long long entry[4];
        int carrier[4], cnt[4];
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            if (r[j] != kNoRow && (j == 0 || r[j] != r[j - 1])) {
                entry[j] = __ldg(oc.entry + r[j]);
                carrier[j] = __ldg(oc.carrier + r[j]);
                cnt[j] = __ldg(oc.cnt + r[j]);
            } else if (j > 0) {
                entry[j] = entry[j - 1]; carrier[j] = carrier[j - 1]; cnt[j] = cnt[j - 1];
            } else {
                entry[j] = 0; carrier[j] = -1; cnt[j] = 0;
            }
        }
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            // inner join (orphan lines drop out); o_entry_d <= ol_delivery_d AND
            // ol_delivery_d < d_hi, a NULL delivery date is UNKNOWN (R5)
            if (r[j] == kNoRow || dl[j] == kNullTs || dl[j] < entry[j] || dl[j] >= d_hi) continue;
            // carrier = 1 OR carrier = 2 / carrier <> 1 AND carrier <> 2; NULL (-1) -> neither
            const bool hi = (carrier[j] == 1) | (carrier[j] == 2);
            const bool lo = (carrier[j] != -1) & !hi;
            sgp_add(P, g, cnt[j], hi, lo);
        }
    });
    sgp_flush(P, g);
}

__global__ void __launch_bounds__(kThreads)
q4_mark_kernel(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
               const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_dl, uint64_t n,
               JoinIndex jo, const int64_t *__restrict__ o_entry, long long e_lo, long long e_hi,
               uint8_t *mark) {
    probe_rows4(ol_w, ol_d, ol_o, ol_dl, n, jo, [&](const unsigned int (&r)[4], const long long (&dl)[4], bool) {
        long long entry[4];
#pragma unroll
        for (int j = 0; j < 4; ++j)
            entry[j] = (r[j] != kNoRow && (j == 0 || r[j] != r[j - 1])) ? __ldg(o_entry + r[j])
                       : (j > 0 ? entry[j - 1] : 0);
#pragma unroll
        for (int j = 0; j < 4; ++j)
            // the order is in the entry window and this line has ol_delivery_d >= o_entry_d
            if (r[j] != kNoRow && entry[j] >= e_lo && entry[j] < e_hi && dl[j] != kNullTs && dl[j] >= entry[j])
                mark[r[j]] = 1;
    });
}

__global__ void __launch_bounds__(kThreads)
q4_count_kernel(const uint8_t *__restrict__ mark, const int32_t *__restrict__ o_cnt, uint64_t n,
                SmallGroups g) {
    __shared__ SgSmem S;
    sg_clear(S);
    __syncthreads();
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t b = (uint64_t)blockIdx.x * blockDim.x + (threadIdx.x & ~31u); b < n; b += stride) {
        const uint64_t i = b + (threadIdx.x & 31);  // warp-uniform loop
        const bool ok = i < n && mark[i];
        sg_warp_add(S, g, ok, ok ? __ldg(o_cnt + i) : 0, true, false);
    }
    sg_flush(S, g);
}

// ================================================================== Q14 ==
__global__ void item_map_clear_kernel(ItemMap m) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < m.words;
         i += (uint64_t)gridDim.x * blockDim.x)
        m.bits[i] = 0u;
}

// bit 2k: item i0+k exists; bit 2k+1: its i_data starts with the 2-character prefix
__global__ void item_map_kernel(const int32_t *__restrict__ i_id, const int32_t *__restrict__ p2,
                                uint64_t n, int prefix2, ItemMap m, unsigned int *err) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (uint64_t)gridDim.x * blockDim.x) {
        const unsigned long long k = (unsigned long long)((long long)i_id[i] - m.i0);
        if (k >= m.range) { atomicOr(err, kErrDomain); continue; }
        const unsigned int sh = 2u * (unsigned int)(k & 15);
        const unsigned int bits = (1u | (p2[i] == prefix2 ? 2u : 0u)) << sh;
        const unsigned int old = atomicOr(m.bits + (k >> 4), bits);
        if (old & (1u << sh)) atomicOr(err, kErrDupItem);
    }
}

constexpr int kQ14SmemWords = 16384;  // 64 KB: item maps of up to 262 144 ids live in shared memory

template <bool kSmemMap>
__global__ void __launch_bounds__(kThreads)
q14_kernel(const longlong2 *__restrict__ deliv, const int4 *__restrict__ iid,
           const longlong2 *__restrict__ amt, uint64_t n, long long d_lo, long long d_hi, ItemMap m,
           long long *__restrict__ part, unsigned int *__restrict__ counter, long long *__restrict__ out) {
    extern __shared__ __align__(16) unsigned int smap[];
    const unsigned int *map = m.bits;
    if (kSmemMap) {
        for (uint64_t i = threadIdx.x; i < m.words; i += blockDim.x) smap[i] = __ldg(m.bits + i);
        __syncthreads();
        map = smap;
    }
    long long sp = 0, sa = 0, cnt = 0;
    auto row = [&](long long d, int id, long long a) {
        // ol_delivery_d >= d_lo AND ol_delivery_d < d_hi (NULL -> UNKNOWN), ol_i_id = i_id
        const unsigned long long k = (unsigned long long)((long long)id - m.i0);
        if ((d == kNullTs) | (d < d_lo) | (d >= d_hi) | (k >= m.range)) return;
        const unsigned int code = (map[k >> 4] >> (2u * (unsigned int)(k & 15))) & 3u;
        if (!(code & 1u)) return;  // no such item: the inner join drops the line
        sa += a;
        sp += (code & 2u) ? a : 0;
        cnt += 1;
    };
    const uint64_t nvec = n >> 2;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < nvec; v += stride) {
        const longlong2 d0 = __ldcs(deliv + 2 * v), d1 = __ldcs(deliv + 2 * v + 1);
        const int4 q = __ldcs(iid + v);
        const longlong2 a0 = __ldcs(amt + 2 * v), a1 = __ldcs(amt + 2 * v + 1);
        row(d0.x, q.x, a0.x);
        row(d0.y, q.y, a0.y);
        row(d1.x, q.z, a1.x);
        row(d1.y, q.w, a1.y);
    }
    {
        const uint64_t t = 4 * nvec + (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
        if (t < n)
            row(reinterpret_cast<const long long *>(deliv)[t], reinterpret_cast<const int *>(iid)[t],
                reinterpret_cast<const long long *>(amt)[t]);
    }
    __shared__ long long s3[3][kThreads / 32];
    __shared__ bool s_last;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    sp = warp_sum64(sp); sa = warp_sum64(sa); cnt = warp_sum64(cnt);
    if (lane == 0) { s3[0][warp] = sp; s3[1][warp] = sa; s3[2][warp] = cnt; }
    __syncthreads();
    if (threadIdx.x == 0) {
        long long P = 0, A = 0, Cn = 0;
        for (int w = 0; w < kThreads / 32; ++w) { P += s3[0][w]; A += s3[1][w]; Cn += s3[2][w]; }
        part[3 * blockIdx.x] = P; part[3 * blockIdx.x + 1] = A; part[3 * blockIdx.x + 2] = Cn;
        __threadfence();
        s_last = atomicAdd(counter, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (s_last && warp == 0) {  // last block folds the block partials (fixed order, exact ints)
        __threadfence();
        long long P = 0, A = 0, Cn = 0;
        for (unsigned b = lane; b < gridDim.x; b += 32) {
            P += __ldcg(part + 3 * b); A += __ldcg(part + 3 * b + 1); Cn += __ldcg(part + 3 * b + 2);
        }
        P = warp_sum64(P); A = warp_sum64(A); Cn = warp_sum64(Cn);
        if (lane == 0) { out[0] = P; out[1] = A; out[2] = Cn; *counter = 0; }
    }
}

// promo_revenue = 100.00 * SUM(promo) / (1 + SUM(amount)) in currency units
//              = (100.0 * P) / (100.0 + S) with P, S in cents (R30)
__global__ void q14_finalize_kernel(const long long *out, double *promo) {
    *promo = (100.0 * (double)out[0]) / (100.0 + (double)out[1]);
}

}  // namespace

// ================================================================ launch ==
void launch_sg_reset(const SmallGroups &g, cudaStream_t st) {
    sg_reset_kernel<<<(kSgSlots * 4 + 3 * kSgDense + 255) / 256, 256, 0, st>>>(g);
}
void launch_sg_emit(const SmallGroups &g, cudaStream_t st) {
    sg_emit_kernel<<<1, kEmitThreads, 0, st>>>(g);
    count_launches(1);
}
void launch_sg_peer_merge(const PeerArgs &p, const SmallGroups &g, cudaStream_t st) {
    launch_pdl(sg_peer_merge_kernel, (3 * kSgDense + kSgSlots + 255) / 256, 256, 0, st, p, g);
    count_launches(1);
}

void launch_jx_build_orders(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, uint64_t n_o,
                            const JoinIndex &jo, unsigned int *err, uint8_t *mark, int num_sms,
                            cudaStream_t st) {
    if (jo.may_ident) {
        jx_verify_kernel<<<grid_for(n_o, 256, num_sms, 8), 256, 0, st>>>(jo, o_w, o_d, o_id, n_o);
        count_launches(1);
    }
    jx_clear_kernel<<<grid_for(jx_words(jo), 256, num_sms, 8), 256, 0, st>>>(jo);
    if (n_o) jx_build_orders_kernel<<<grid_for(n_o, 256, num_sms, 8), 256, 0, st>>>(o_w, o_d, o_id, n_o, jo, err, mark);
    count_launches(n_o ? 2 : 1);
}

void launch_q12_probe(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o, const int64_t *ol_dl,
                      uint64_t n_ol, const JoinIndex &jo, const int64_t *o_entry, const int32_t *o_carrier,
                      const int32_t *o_cnt, int64_t d_hi, const SmallGroups &g, int num_sms, cudaStream_t st) {
    const unsigned grid = grid_for((n_ol + 3) / 4, kThreads, num_sms, 8);
    q12_probe_kernel<<<grid, kThreads, 0, st>>>(ol_w, ol_d, ol_o, ol_dl, n_ol, jo,
                                                             OrderCols{o_entry, o_carrier, o_cnt}, d_hi, g);
    count_launches(1);
}

void launch_q4(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o, const int64_t *ol_dl,
               uint64_t n_ol, const JoinIndex &jo, const int64_t *o_entry, const int32_t *o_cnt,
               uint64_t n_o, int64_t e_lo, int64_t e_hi, uint8_t *mark, const SmallGroups &g,
               int num_sms, cudaStream_t st, PhaseMarks *marks) {
    if (marks) marks->begin("q4_semijoin_mark");
    if (n_ol)
        q4_mark_kernel<<<grid_for((n_ol + 3) / 4, kThreads, num_sms, 8), kThreads, 0, st>>>(
            ol_w, ol_d, ol_o, ol_dl, n_ol, jo, o_entry, e_lo, e_hi, mark);
    if (marks) marks->end();
    if (marks) marks->begin("q4_count");
    if (n_o)
        q4_count_kernel<<<grid_for(n_o, kThreads, num_sms, 8), kThreads, 0, st>>>(mark, o_cnt, n_o, g);
    if (marks) marks->end();
    count_launches((n_ol ? 1 : 0) + (n_o ? 1 : 0));
}

void launch_item_map(const int32_t *i_id, const int32_t *p2, uint64_t n, int32_t prefix2, const ItemMap &m,
                     unsigned int *err, int num_sms, cudaStream_t st) {
    item_map_clear_kernel<<<grid_for(m.words, 256, num_sms, 4), 256, 0, st>>>(m);
    if (n) item_map_kernel<<<grid_for(n, 256, num_sms, 4), 256, 0, st>>>(i_id, p2, n, prefix2, m, err);
    count_launches(n ? 2 : 1);
}

int q14_max_blocks(int num_sms) { return num_sms * 8; }

void launch_q14(const int64_t *deliv, const int32_t *i_id, const int64_t *amt, uint64_t n, int64_t d_lo,
                int64_t d_hi, const ItemMap &m, const Q14Scratch &s, int num_sms, cudaStream_t st) {
    const bool smem_map = m.words <= (uint64_t)kQ14SmemWords;
    // 4 blocks per SM (each copies the map into shared memory; more blocks measured slower)
    const int per_sm = smem_map ? (m.words * 4 > (48u << 10) ? 2 : 4) : 8;
    const unsigned grid = grid_for((n + 3) / 4, kThreads, num_sms, per_sm);
    const auto *D = reinterpret_cast<const longlong2 *>(deliv);
    const auto *I = reinterpret_cast<const int4 *>(i_id);
    const auto *A = reinterpret_cast<const longlong2 *>(amt);
    if (smem_map)
        q14_kernel<true><<<grid, kThreads, m.words * 4, st>>>(D, I, A, n, d_lo, d_hi, m, s.block_part,
                                                              s.done_counter, s.out);
    else
        q14_kernel<false><<<grid, kThreads, 0, st>>>(D, I, A, n, d_lo, d_hi, m, s.block_part,
                                                     s.done_counter, s.out);
    count_launches(1);
}

void launch_q14_finalize(const Q14Scratch &s, cudaStream_t st) {
    q14_finalize_kernel<<<1, 1, 0, st>>>(s.out, s.promo);
    count_launches(1);
}

// Load every kernel of this file now (CUDA lazy loading would otherwise load a kernel at its first
// launch, which waits for the device to idle — with N logical ranks on one device, behind another
// rank's kernel that is waiting for this rank: a deadlock).
static cudaError_t force_load(const void *const *fs, size_t n) {
    for (size_t i = 0; i < n; ++i) {
        cudaFuncAttributes a;
        const cudaError_t e = cudaFuncGetAttributes(&a, fs[i]);
        if (e != cudaSuccess) return e;
    }
    return cudaSuccess;
}

cudaError_t set_attributes_ch(int num_sms) {
    static const void *const kKernels[] = {
        (const void *)item_map_clear_kernel,
        (const void *)item_map_kernel,
        (const void *)jx_build_orders_kernel,
        (const void *)jx_clear_kernel,
        (const void *)jx_verify_kernel,
        (const void *)q12_probe_kernel,
        (const void *)q14_finalize_kernel,
        (const void *)q14_kernel<false>,
        (const void *)q14_kernel<true>,
        (const void *)q4_count_kernel,
        (const void *)q4_mark_kernel,
        (const void *)sg_emit_kernel,
        (const void *)sg_peer_merge_kernel,
        (const void *)sg_reset_kernel};
    const cudaError_t le = force_load(kKernels, sizeof kKernels / sizeof kKernels[0]);
    if (le != cudaSuccess) return le;

    (void)num_sms;
    return cudaFuncSetAttribute(q14_kernel<true>, cudaFuncAttributeMaxDynamicSharedMemorySize, kQ14SmemWords * 4);
}

}  // namespace h2tap
