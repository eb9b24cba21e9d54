// ch_kernels.cu — NEXT-2: CH-benCHmark Q14, Q12 and Q4 on the same snapshot,
// join index and aggregation machinery as the hot path, for sm_100a.
//
//  Q14  order_line ⋈ item: one fused scan of (delivery 8 B, i_id 4 B, amount 8 B) per row with
//       the item side as a 2-bit-per-id map (exists, i_data LIKE 'PR%') held in shared memory
//       (25 KB for TPC-C's 100 000 items); int64 sums, last-block fold, promo ratio in double.
//  Q12  orders ⋈ order_line GROUP BY o_ol_cnt: stream (w, d, o, delivery) per line, one lookup of
//       the orders join index per run of equal keys inside a lane, gather (entry, carrier,
//       ol_cnt), count per group in thread-private shared-memory counters.
//  Q4   orders ⋉ order_line (EXISTS): the same stream marks orders rows that have a qualifying
//       line (idempotent byte store), then one pass over orders counts marked rows per o_ol_cnt.
// The paper gives no plans for these queries (it evaluates TPC-H Q6 only);
// like the hot path they run on an epoch's snapshot (L555-572). DESIGN.md §4.8.
#include <cstdint>
#include <cuda_runtime.h>

#include "join_index.cuh"
#include "kernels.cuh"

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
// GROUP BY o_ol_cnt with three counters per group (a, b, rows). Keys in [0, kSgDense) are counted
// in thread-private shared memory (no atomics) and folded once per block; other keys go to a
// global open-addressing table (atomics; TPC-C never produces them).
struct SgSmem {
    unsigned int c[3][kSgDense][kThreads];  // [counter][key][thread]: lane-distinct banks
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
    unsigned int *p = &S.c[0][0][0];
    for (int i = threadIdx.x; i < 3 * kSgDense * kThreads; i += blockDim.x) p[i] = 0;
}

__device__ __forceinline__ void sg_add(SgSmem &S, const SmallGroups &g, int key, unsigned a, unsigned b) {
    if ((unsigned)key < (unsigned)kSgDense) {
        S.c[0][key][threadIdx.x] += a;
        S.c[1][key][threadIdx.x] += b;
        S.c[2][key][threadIdx.x] += 1;
    } else {
        sg_global_add(g, key, a, b, 1);
    }
}

// fold the block's private counters into g.dense: warp w sums rows w, w+8, ... (lanes stride the
// 256 threads), one 64-bit atomic per non-zero (counter, key)
__device__ void sg_flush(SgSmem &S, const SmallGroups &g) {
    __syncthreads();
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    for (int r = warp; r < 3 * kSgDense; r += blockDim.x / 32) {
        const unsigned int *row = &S.c[r / kSgDense][r % kSgDense][0];
        long long v = 0;
        for (int t = lane; t < kThreads; t += 32) v += row[t];
        v = warp_sum64(v);
        if (lane == 0 && v) atomicAdd(g.dense + (r % kSgDense) * 3 + r / kSgDense, (unsigned long long)v);
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
__global__ void sg_merge_kernel(const unsigned long long *__restrict__ dense,
                                const unsigned long long *__restrict__ gtag,
                                const unsigned long long *__restrict__ gacc, SmallGroups g) {
    const int i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i < 3 * kSgDense) {
        if (dense[i]) atomicAdd(g.dense + i, dense[i]);
    } else if (i < 3 * kSgDense + kSgSlots) {
        const int s = i - 3 * kSgDense;
        const unsigned long long t = gtag[s];
        if (t) sg_global_add(g, (int)(unsigned int)t, gacc[3 * s], gacc[3 * s + 1], gacc[3 * s + 2]);
    }
}

// ========================================================= orders index ==
__global__ void jx_clear_kernel(JoinIndex j) {
    const uint64_t words = jx_words(j);
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < words;
         i += (uint64_t)gridDim.x * blockDim.x)
        jx_clear(j, i);
}

__global__ void jx_build_orders_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                                       const int32_t *__restrict__ o_id, uint64_t n, JoinIndex j,
                                       unsigned int *err, uint8_t *mark) {
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (uint64_t)gridDim.x * blockDim.x) {
        if (mark) mark[i] = 0;
        if (!jx_insert(j, o_w[i], o_d[i], o_id[i], (unsigned int)i, err, kErrDupOrders))
            atomicOr(err, kErrDomain);
    }
}

// ======================================================= Q12 / Q4 probes ==
// Each lane owns 4 consecutive order_line rows (128-bit loads of w, d, o, two of delivery); the
// orders row is looked up once per run of equal keys inside the lane (lines of an order are
// adjacent), and the row's (entry, carrier, ol_cnt) gathered once per lookup.
struct OrderCols { const int64_t *entry; const int32_t *carrier, *cnt; };

template <class RowFn>
__device__ __forceinline__ void probe_rows(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
                                           const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_dl,
                                           uint64_t n, const JoinIndex &jo, RowFn &&fn) {
    const uint64_t nvec = n >> 2;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
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
    load(v);
    for (; v < nvec; v += stride) {
        const int w[4] = {nW.x, nW.y, nW.z, nW.w}, d[4] = {nD.x, nD.y, nD.z, nD.w},
                  o[4] = {nO.x, nO.y, nO.z, nO.w};
        const long long dl[4] = {nL0.x, nL0.y, nL1.x, nL1.y};
        load(v + stride);  // next group's loads in flight while this one is probed
        unsigned int row = kNoRow;
#pragma unroll
        for (int j = 0; j < 4; ++j) {
            if (j == 0 || w[j] != w[j - 1] || d[j] != d[j - 1] || o[j] != o[j - 1])
                row = jx_lookup(jo, w[j], d[j], o[j]);
            fn(row, dl[j]);
        }
    }
    // ragged tail (< 4 rows): the first threads, one row each
    const uint64_t t = 4 * nvec + (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
    if (t < n) fn(jx_lookup(jo, ol_w[t], ol_d[t], ol_o[t]), ol_dl[t]);
}

__global__ void __launch_bounds__(kThreads)
q12_probe_kernel(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
                 const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_dl, uint64_t n,
                 JoinIndex jo, OrderCols oc, long long d_hi, SmallGroups g) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    SgSmem &S = *reinterpret_cast<SgSmem *>(smem_raw);
    sg_clear(S);
    __syncthreads();
    // cache the gathered orders fields of the last looked-up row
    unsigned int last = kNoRow;
    long long entry = 0;
    int carrier = -1, cnt = 0;
    probe_rows(ol_w, ol_d, ol_o, ol_dl, n, jo, [&](unsigned int row, long long dl) {
        if (row == kNoRow) return;  // inner join: orphan lines drop out
        if (row != last) {
            last = row;
            entry = __ldg(oc.entry + row);
            carrier = __ldg(oc.carrier + row);
            cnt = __ldg(oc.cnt + row);
        }
        // o_entry_d <= ol_delivery_d AND ol_delivery_d < d_hi; NULL delivery -> UNKNOWN (R5)
        if (dl == kNullTs || dl < entry || dl >= d_hi) return;
        // carrier = 1 OR carrier = 2 / carrier <> 1 AND carrier <> 2; NULL (-1) -> neither
        const unsigned hi = (carrier == 1) | (carrier == 2);
        const unsigned lo = (carrier != -1) & !hi;
        sg_add(S, g, cnt, hi, lo);
    });
    sg_flush(S, g);
}

__global__ void __launch_bounds__(kThreads)
q4_mark_kernel(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
               const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_dl, uint64_t n,
               JoinIndex jo, const int64_t *__restrict__ o_entry, long long e_lo, long long e_hi,
               uint8_t *mark) {
    unsigned int last = kNoRow;
    long long entry = 0;
    probe_rows(ol_w, ol_d, ol_o, ol_dl, n, jo, [&](unsigned int row, long long dl) {
        if (row == kNoRow) return;
        if (row != last) { last = row; entry = __ldg(o_entry + row); }
        // the order is in the entry window and this line has ol_delivery_d >= o_entry_d
        if (entry >= e_lo && entry < e_hi && dl != kNullTs && dl >= entry) mark[row] = 1;
    });
}

__global__ void __launch_bounds__(kThreads)
q4_count_kernel(const uint8_t *__restrict__ mark, const int32_t *__restrict__ o_cnt, uint64_t n,
                SmallGroups g) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    SgSmem &S = *reinterpret_cast<SgSmem *>(smem_raw);
    sg_clear(S);
    __syncthreads();
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n;
         i += (uint64_t)gridDim.x * blockDim.x)
        if (mark[i]) sg_add(S, g, __ldg(o_cnt + i), 1u, 0u);
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
void launch_sg_merge(const unsigned long long *dense, const unsigned long long *gtag,
                     const unsigned long long *gacc, const SmallGroups &g, cudaStream_t st) {
    sg_merge_kernel<<<(3 * kSgDense + kSgSlots + 255) / 256, 256, 0, st>>>(dense, gtag, gacc, g);
    count_launches(1);
}

void launch_jx_build_orders(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, uint64_t n_o,
                            const JoinIndex &jo, unsigned int *err, uint8_t *mark, int num_sms,
                            cudaStream_t st) {
    jx_clear_kernel<<<grid_for(jx_words(jo), 256, num_sms, 8), 256, 0, st>>>(jo);
    if (n_o) jx_build_orders_kernel<<<grid_for(n_o, 256, num_sms, 8), 256, 0, st>>>(o_w, o_d, o_id, n_o, jo, err, mark);
    count_launches(n_o ? 2 : 1);
}

void launch_q12_probe(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o, const int64_t *ol_dl,
                      uint64_t n_ol, const JoinIndex &jo, const int64_t *o_entry, const int32_t *o_carrier,
                      const int32_t *o_cnt, int64_t d_hi, const SmallGroups &g, int num_sms, cudaStream_t st) {
    static bool attr = false;
    if (!attr) {
        cudaFuncSetAttribute(q12_probe_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sizeof(SgSmem));
        attr = true;
    }
    const unsigned grid = grid_for((n_ol + 3) / 4, kThreads, num_sms, 4);
    q12_probe_kernel<<<grid, kThreads, sizeof(SgSmem), st>>>(ol_w, ol_d, ol_o, ol_dl, n_ol, jo,
                                                             OrderCols{o_entry, o_carrier, o_cnt}, d_hi, g);
    count_launches(1);
}

void launch_q4(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o, const int64_t *ol_dl,
               uint64_t n_ol, const JoinIndex &jo, const int64_t *o_entry, const int32_t *o_cnt,
               uint64_t n_o, int64_t e_lo, int64_t e_hi, uint8_t *mark, const SmallGroups &g,
               int num_sms, cudaStream_t st, PhaseMarks *marks) {
    static bool attr = false;
    if (!attr) {
        cudaFuncSetAttribute(q4_count_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sizeof(SgSmem));
        attr = true;
    }
    if (marks) marks->begin("q4_semijoin_mark");
    if (n_ol)
        q4_mark_kernel<<<grid_for((n_ol + 3) / 4, kThreads, num_sms, 8), kThreads, 0, st>>>(
            ol_w, ol_d, ol_o, ol_dl, n_ol, jo, o_entry, e_lo, e_hi, mark);
    if (marks) marks->end();
    if (marks) marks->begin("q4_count");
    if (n_o)
        q4_count_kernel<<<grid_for(n_o, kThreads, num_sms, 4), kThreads, sizeof(SgSmem), st>>>(mark, o_cnt, n_o, g);
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
    static bool attr = false;
    if (!attr) {
        cudaFuncSetAttribute(q14_kernel<true>, cudaFuncAttributeMaxDynamicSharedMemorySize, kQ14SmemWords * 4);
        attr = true;
    }
    const int per_sm = smem_map ? (m.words * 4 > 48 * 1024 ? 2 : 4) : 8;
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

}  // namespace h2tap
