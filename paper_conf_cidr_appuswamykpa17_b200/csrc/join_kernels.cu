// join_kernels.cu — K3 join-index build, K4 probe + group-join aggregation, K5 HAVING +
// compaction + customer probe + gather, for CH Q18 (customer ⋈ orders ⋈ order_line, GROUP BY,
// HAVING) on sm_100a.
//
// The paper gives no join algorithm (hash joins on accelerators appear only as related work,
// PAPER.md L1224-1227); its runtime hands kernels the snapshot's column pointers (L568-570).
// Design: a join index per build side maps the primary key (w, d, id) to a row.
// It is a perfect hash (slot = dense rank of the key in the build side's [min, max] box, from
// the snapshot's column statistics) when that box is small, else an open-addressing hash table
// (16-byte slots, linear probing, capacity pow2 >= 2n, insert by 64-bit atomicCAS). Q18's
// GROUP BY key (o_id, o_w_id, o_d_id, c_id, c_last, o_entry_d, o_ol_cnt) is functionally
// determined by the orders row once the orders and customer PKs are unique (checked:
// EDUPKEY), so the group-by collapses onto the orders row: acc[orders row] += (amount, 1).
#include <cstdint>
#include <cuda_runtime.h>

#include "kernels.cuh"

namespace h2tap {
namespace {

constexpr unsigned kFull = 0xffffffffu;

__device__ __forceinline__ unsigned long long fmix64(unsigned long long k) {
    k ^= k >> 33; k *= 0xff51afd7ed558ccdull; k ^= k >> 33; k *= 0xc4ceb9fe1a85ec53ull; k ^= k >> 33;
    return k;
}

// (w, d, id) -> 64-bit key, injective on the supported domain (R16).
__device__ __forceinline__ bool pack_key(int w, int d, int id, unsigned long long &k) {
    k = ((unsigned long long)(unsigned)w << 40) | ((unsigned long long)(unsigned)d << 32) |
        (unsigned long long)(unsigned)id;
    return ((unsigned)w < (1u << 23)) & ((unsigned)d < 256u) & (id >= 0);
}

// Dense slot of (w, d, id) in the index's box, or false when outside it.
__device__ __forceinline__ bool dense_slot(const JoinIndex &j, int w, int d, int id,
                                          unsigned long long &slot) {
    const unsigned dw = (unsigned)(w - j.w0), dd = (unsigned)(d - j.d0), dk = (unsigned)(id - j.k0);
    slot = ((unsigned long long)dw * j.nd + dd) * j.nk + dk;
    return (dw < j.nw) & (dd < j.nd) & (dk < j.nk);
}

// Insert; returns false on a key outside the supported domain. Duplicates set `dupbit`.
__device__ __forceinline__ bool jx_insert(const JoinIndex &j, int w, int d, int id, unsigned int row,
                                          unsigned int *err, unsigned int dupbit) {
    if (j.dense) {
        unsigned long long s;
        if (!dense_slot(j, w, d, id, s)) return false;  // stats must cover every build row
        if (atomicCAS(j.slots + s, kNoRow, row) != kNoRow) atomicOr(err, dupbit);
        return true;
    }
    unsigned long long key;
    if (!pack_key(w, d, id, key)) return false;
    unsigned long long h = fmix64(key) & j.mask;
    while (true) {
        const unsigned long long prev = atomicCAS(&j.ht[h].key, kEmpty, key);
        if (prev == kEmpty) { j.ht[h].row = row; return true; }
        if (prev == key) { atomicOr(err, dupbit); return true; }
        h = (h + 1) & j.mask;
    }
}

__device__ __forceinline__ unsigned int jx_lookup(const JoinIndex &j, int w, int d, int id) {
    if (j.dense) {
        unsigned long long s;
        if (!dense_slot(j, w, d, id, s)) return kNoRow;  // outside the build box: no match
        return __ldcg(j.slots + s);
    }
    unsigned long long key;
    if (!pack_key(w, d, id, key)) return kNoRow;  // no build key can lie outside the domain
    unsigned long long h = fmix64(key) & j.mask;
    while (true) {
        const ulonglong2 s = __ldcg(reinterpret_cast<const ulonglong2 *>(j.ht + h));
        if (s.x == key) return (unsigned int)s.y;
        if (s.x == kEmpty) return kNoRow;
        h = (h + 1) & j.mask;
    }
}

unsigned grid_for(uint64_t work, int threads, int num_sms, int per_sm) {
    uint64_t want = (work + threads - 1) / threads;
    uint64_t cap = (uint64_t)num_sms * per_sm;
    if (want > cap) want = cap;
    return want ? (unsigned)want : 1u;
}

// ------------------------------------------------------------------- init --
// Empties both join indexes, zeroes the group accumulators and the counters: one launch.
__host__ __device__ __forceinline__ uint64_t jx_words(const JoinIndex &j) {  // 16-byte units
    return j.dense ? (j.range + 3) / 4 : j.mask + 1;
}
__device__ __forceinline__ void jx_clear(const JoinIndex &j, uint64_t i) {
    if (j.dense) reinterpret_cast<uint4 *>(j.slots)[i] = make_uint4(kNoRow, kNoRow, kNoRow, kNoRow);
    else reinterpret_cast<ulonglong2 *>(j.ht)[i] = make_ulonglong2(kEmpty, 0ull);
}

__global__ void q18_init_kernel(Q18Scratch s, uint64_t n_orders) {
    const uint64_t a = jx_words(s.jo), b = jx_words(s.jc);
    const uint64_t total = a + b + n_orders;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < total; i += stride) {
        if (i < a) jx_clear(s.jo, i);
        else if (i < a + b) jx_clear(s.jc, i - a);
        else reinterpret_cast<ulonglong2 *>(s.acc)[i - a - b] = make_ulonglong2(0ull, 0ull);
    }
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        *s.err = 0;
        *s.nout = 0;
        Q18Stats st;
        st.amt_min = INT64_MAX; st.amt_max = INT64_MIN; st.ent_min = INT64_MAX; st.ent_max = INT64_MIN;
        st.w_min = INT32_MAX; st.w_max = INT32_MIN; st.d_min = INT32_MAX; st.d_max = INT32_MIN;
        st.o_min = INT32_MAX; st.o_max = INT32_MIN; st.pad0 = st.pad1 = 0;
        *s.stats = st;
    }
}

// ------------------------------------------------------------------ K3 build --
__global__ void q18_build_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                                 const int32_t *__restrict__ o_id, uint64_t n_o,
                                 const int32_t *__restrict__ c_w, const int32_t *__restrict__ c_d,
                                 const int32_t *__restrict__ c_id, uint64_t n_c, Q18Scratch s) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n_o + n_c; i += stride) {
        bool ok;
        if (i < n_o) {
            ok = jx_insert(s.jo, o_w[i], o_d[i], o_id[i], (unsigned int)i, s.err, kErrDupOrders);
        } else {
            const uint64_t j = i - n_o;
            ok = jx_insert(s.jc, c_w[j], c_d[j], c_id[j], (unsigned int)j, s.err, kErrDupCustomer);
        }
        if (!ok) atomicOr(s.err, kErrDomain);
    }
}

// ------------------------------------------------------- K4 probe + group-join --
// One warp iteration covers 32 consecutive order_line rows (coalesced 4 B / 8 B loads).
// Lines of one order are usually contiguous, so equal keys form runs: a segmented inclusive
// scan (shuffles) sums each run, the run head probes the orders index once, and the run tail
// issues the two atomics — ~3 runs per 32 rows instead of 32 probes and 64 atomics.
constexpr int kProbeThreads = 256;
constexpr int kProbeUnroll = 4;

__global__ void __launch_bounds__(kProbeThreads)
q18_probe_kernel(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
                 const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_amt, uint64_t n,
                 Q18Scratch s) {
    const int lane = threadIdx.x & 31;
    const uint64_t gwarp = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    const unsigned le_mask = 0xffffffffu >> (31 - lane);  // lanes 0..lane
    for (uint64_t base = gwarp * 32 * kProbeUnroll; base < n; base += nwarps * 32 * kProbeUnroll) {
        int w[kProbeUnroll], d[kProbeUnroll], o[kProbeUnroll];
        long long amt[kProbeUnroll];
        bool valid[kProbeUnroll];
#pragma unroll
        for (int u = 0; u < kProbeUnroll; ++u) {
            const uint64_t i = base + u * 32 + lane;
            valid[u] = i < n;
            if (valid[u]) {
                w[u] = __ldcs(ol_w + i); d[u] = __ldcs(ol_d + i); o[u] = __ldcs(ol_o + i);
                amt[u] = __ldcs(ol_amt + i);
            } else {  // tail rows: never probe, never aggregate
                w[u] = 0; d[u] = 0; o[u] = 0; amt[u] = 0;
            }
        }
#pragma unroll
        for (int u = 0; u < kProbeUnroll; ++u) {
            const bool same = (__shfl_up_sync(kFull, w[u], 1) == w[u]) &
                              (__shfl_up_sync(kFull, d[u], 1) == d[u]) &
                              (__shfl_up_sync(kFull, o[u], 1) == o[u]) &
                              (__shfl_up_sync(kFull, (int)valid[u], 1) == (int)valid[u]);
            const bool head = lane == 0 || !same;
            const unsigned heads = __ballot_sync(kFull, head);
            const int leader = 31 - __clz(heads & le_mask);
            long long sum = amt[u];
#pragma unroll
            for (int off = 1; off < 32; off <<= 1) {
                const long long t = __shfl_up_sync(kFull, sum, off);
                if (lane - off >= leader) sum += t;
            }
            const bool tail = lane == 31 || ((heads >> (lane + 1)) & 1u);
            unsigned int row = kNoRow;
            if (head && valid[u]) row = jx_lookup(s.jo, w[u], d[u], o[u]);
            row = __shfl_sync(kFull, row, leader);
            if (tail && row != kNoRow) {
                atomicAdd(reinterpret_cast<unsigned long long *>(&s.acc[row].sum),
                          (unsigned long long)sum);
                atomicAdd(&s.acc[row].cnt, (unsigned int)(lane - leader + 1));
            }
        }
    }
}

// ---------------------------------------- K5 HAVING + customer probe + compaction --
constexpr int kHavingThreads = 256;

__device__ __forceinline__ long long wmin64(long long v) {
    for (int o = 16; o; o >>= 1) { long long t = __shfl_xor_sync(kFull, v, o); v = t < v ? t : v; }
    return v;
}
__device__ __forceinline__ long long wmax64(long long v) {
    for (int o = 16; o; o >>= 1) { long long t = __shfl_xor_sync(kFull, v, o); v = t > v ? t : v; }
    return v;
}

struct StatAcc {
    long long amin = INT64_MAX, amax = INT64_MIN, emin = INT64_MAX, emax = INT64_MIN;
    int wmin = INT32_MAX, wmax = INT32_MIN, dmin = INT32_MAX, dmax = INT32_MIN;
    int omin = INT32_MAX, omax = INT32_MIN;
    __device__ void add(long long a, long long e, int w, int d, int o) {
        amin = a < amin ? a : amin; amax = a > amax ? a : amax;
        emin = e < emin ? e : emin; emax = e > emax ? e : emax;
        wmin = min(wmin, w); wmax = max(wmax, w); dmin = min(dmin, d); dmax = max(dmax, d);
        omin = min(omin, o); omax = max(omax, o);
    }
    __device__ void flush(Q18Stats *st) {  // warp-reduce, lane 0 issues the atomics
        amin = wmin64(amin); amax = wmax64(amax); emin = wmin64(emin); emax = wmax64(emax);
        wmin = __reduce_min_sync(kFull, wmin); wmax = __reduce_max_sync(kFull, wmax);
        dmin = __reduce_min_sync(kFull, dmin); dmax = __reduce_max_sync(kFull, dmax);
        omin = __reduce_min_sync(kFull, omin); omax = __reduce_max_sync(kFull, omax);
        if ((threadIdx.x & 31) == 0 && amin <= amax) {
            atomicMin(&st->amt_min, amin); atomicMax(&st->amt_max, amax);
            atomicMin(&st->ent_min, emin); atomicMax(&st->ent_max, emax);
            atomicMin(&st->w_min, wmin); atomicMax(&st->w_max, wmax);
            atomicMin(&st->d_min, dmin); atomicMax(&st->d_max, dmax);
            atomicMin(&st->o_min, omin); atomicMax(&st->o_max, omax);
        }
    }
};

// Each block iteration covers kHavingRows consecutive orders rows (kHavingUnroll per thread);
// passing rows get output slots from ONE atomicAdd per block iteration (block-wide exclusive
// scan of the per-thread counts), so the output counter sees ~n/1024 atomics, not n/32.
constexpr int kHavingUnroll = 4;
constexpr int kHavingRows = kHavingThreads * kHavingUnroll;

__global__ void __launch_bounds__(kHavingThreads)
q18_having_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                  const int32_t *__restrict__ o_id, const int32_t *__restrict__ o_c,
                  const int32_t *__restrict__ o_cnt, const int64_t *__restrict__ o_ent, uint64_t n,
                  const int32_t *__restrict__ c_last, long long having, Q18Scratch s) {
    __shared__ unsigned int wsum[kHavingThreads / 32];
    __shared__ unsigned long long s_base;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    StatAcc stat;
    for (uint64_t base = (uint64_t)blockIdx.x * kHavingRows; base < n;
         base += (uint64_t)gridDim.x * kHavingRows) {
        unsigned int crow[kHavingUnroll];
        long long sum[kHavingUnroll];
        int w[kHavingUnroll], d[kHavingUnroll], c[kHavingUnroll];
        unsigned int mine = 0;
#pragma unroll
        for (int u = 0; u < kHavingUnroll; ++u) {
            const uint64_t r = base + u * kHavingThreads + threadIdx.x;
            crow[u] = kNoRow;
            sum[u] = 0;
            w[u] = d[u] = c[u] = 0;
            if (r < n) {
                const ulonglong2 a = __ldcs(reinterpret_cast<const ulonglong2 *>(s.acc + r));
                sum[u] = (long long)a.x;
                // inner join: a group exists only with >= 1 order_line row; HAVING SUM > having
                if ((unsigned int)a.y > 0 && sum[u] > having) {
                    w[u] = o_w[r]; d[u] = o_d[r]; c[u] = o_c[r];
                    crow[u] = jx_lookup(s.jc, w[u], d[u], c[u]);  // customer ⋈ orders
                }
            }
            mine += crow[u] != kNoRow;
        }
        // block-wide exclusive scan of `mine`, one atomic for the block's output range
        unsigned int x = mine;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const unsigned int t = __shfl_up_sync(kFull, x, o);
            if (lane >= o) x += t;
        }
        if (lane == 31) wsum[warp] = x;
        __syncthreads();
        unsigned int before = 0, total = 0;
#pragma unroll
        for (int k = 0; k < kHavingThreads / 32; ++k) {
            before += k < warp ? wsum[k] : 0u;
            total += wsum[k];
        }
        if (threadIdx.x == 0) s_base = total ? atomicAdd(s.nout, (unsigned long long)total) : 0ull;
        __syncthreads();
        uint64_t p = s_base + before + x - mine;
#pragma unroll
        for (int u = 0; u < kHavingUnroll; ++u) {
            if (crow[u] == kNoRow) continue;
            const uint64_t r = base + u * kHavingThreads + threadIdx.x;
            Q18Row row;
            row.amount_sum = sum[u];
            row.o_entry_d = o_ent[r];
            row.c_last = c_last[crow[u]];
            row.c_id = c[u];
            row.o_id = o_id[r];
            row.o_ol_cnt = o_cnt[r];
            row.o_w_id = w[u];
            row.o_d_id = d[u];
            s.rows[p++] = row;
            stat.add(sum[u], row.o_entry_d, w[u], d[u], row.o_id);
        }
        __syncthreads();  // wsum / s_base reuse
    }
    stat.flush(s.stats);
}

__global__ void q18_stats_kernel(const Q18Row *__restrict__ rows, uint64_t n, Q18Stats *st) {
    StatAcc stat;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        const Q18Row r = rows[i];
        stat.add(r.amount_sum, r.o_entry_d, r.o_w_id, r.o_d_id, r.o_id);
    }
    stat.flush(st);
}

}  // namespace

void launch_q18_init(const Q18Scratch &s, uint64_t n_orders, int num_sms, cudaStream_t st) {
    const uint64_t words = jx_words(s.jo) + jx_words(s.jc) + n_orders;
    q18_init_kernel<<<grid_for(words, 256, num_sms, 8), 256, 0, st>>>(s, n_orders);
    count_launches(1);
}

void launch_q18_build(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, uint64_t n_o,
                      const int32_t *c_w, const int32_t *c_d, const int32_t *c_id, uint64_t n_c,
                      const Q18Scratch &s, int num_sms, cudaStream_t st) {
    q18_build_kernel<<<grid_for(n_o + n_c, 256, num_sms, 8), 256, 0, st>>>(o_w, o_d, o_id, n_o, c_w,
                                                                         c_d, c_id, n_c, s);
    count_launches(1);
}

void launch_q18_probe(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o,
                      const int64_t *ol_amt, uint64_t n_ol, const Q18Scratch &s, int num_sms,
                      cudaStream_t st) {
    q18_probe_kernel<<<grid_for((n_ol + kProbeUnroll - 1) / kProbeUnroll, kProbeThreads, num_sms, 8),
                       kProbeThreads, 0, st>>>(ol_w, ol_d, ol_o, ol_amt, n_ol, s);
    count_launches(1);
}

void launch_q18_having(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id,
                       const int32_t *o_c, const int32_t *o_cnt, const int64_t *o_ent,
                       uint64_t n_o, const int32_t *c_last, int64_t having,
                       const Q18Scratch &s, int num_sms, cudaStream_t st) {
    q18_having_kernel<<<grid_for((n_o + kHavingUnroll - 1) / kHavingUnroll, kHavingThreads, num_sms, 8),
                        kHavingThreads, 0, st>>>(
        o_w, o_d, o_id, o_c, o_cnt, o_ent, n_o, c_last, having, s);
    count_launches(1);
}

void launch_q18_stats(const Q18Row *rows, uint64_t n, Q18Stats *stats, int num_sms,
                      cudaStream_t st) {
    q18_stats_kernel<<<grid_for(n, 256, num_sms, 4), 256, 0, st>>>(rows, n, stats);
    count_launches(1);
}

}  // namespace h2tap
