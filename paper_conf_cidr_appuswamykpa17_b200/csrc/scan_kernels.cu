// scan_kernels.cu — K1 (CH Q6 fused scan-filter-sum) and K2 (CH Q1 fused scan-filter-group-by)
// for sm_100a.
//
// Paper anchor: the data-parallel archipelago runs OLAP scans over a columnar (DSM) snapshot
// (Fig. 3); "GPUs coalesce global memory loads ... threads should access
// memory locations sequentially" (L511-517), which is what DSM buys (L987-990). The paper runs
// one CUDA kernel per primitive with materialised intermediates and calls that sub-optimal
// (L527-535) with fusion as future work (L552-554): here each query is ONE fused kernel plus a
// tiny finaliser, and the scan is HBM-bound (20 B/row for Q6, 24 B/row for Q1).
#include <algorithm>
#include <cstdlib>
#include <cstdint>
#include <cuda_runtime.h>

#include "bulk_pipeline.cuh"
#include "kernels.cuh"
#include "peer.cuh"
#include "probe_device.cuh"

namespace h2tap {
namespace {

constexpr unsigned kFull = 0xffffffffu;

// 128-bit streaming loads: read-only path, do not allocate in L1 (each byte is read once).
__device__ __forceinline__ longlong2 ld_stream(const longlong2 *p) {
    longlong2 r;
    asm volatile("ld.global.nc.L1::no_allocate.v2.s64 {%0, %1}, [%2];"
                 : "=l"(r.x), "=l"(r.y) : "l"(p));
    return r;
}
__device__ __forceinline__ int4 ld_stream(const int4 *p) {
    int4 r;
    asm volatile("ld.global.nc.L1::no_allocate.v4.s32 {%0, %1, %2, %3}, [%4];"
                 : "=r"(r.x), "=r"(r.y), "=r"(r.z), "=r"(r.w) : "l"(p));
    return r;
}

__device__ __forceinline__ long long warp_sum(long long v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
    return v;
}

// ================================================================== Q6 ====
constexpr int kQ6Threads = 256;
constexpr int kQ6Unroll = 2;  // 4-row vectors per thread per iteration

struct Q6Pred {
    long long d_lo, d_hi, q_lo, q_hi;
    // WHERE ol_delivery_d >= d_lo AND ol_delivery_d < d_hi AND ol_quantity BETWEEN q_lo AND q_hi;
    // a NULL delivery date (INT64_MIN) makes the conjunction UNKNOWN -> row excluded (R5).
    __device__ __forceinline__ bool operator()(long long d, int q) const {
        return (d != kNullTs) & (d >= d_lo) & (d < d_hi) & ((long long)q >= q_lo) &
               ((long long)q <= q_hi);
    }
};

__global__ void __launch_bounds__(kQ6Threads)
q6_kernel(const longlong2 *__restrict__ deliv, const int4 *__restrict__ qty,
          const longlong2 *__restrict__ amt, uint64_t n, Q6Pred pred,
          long long *__restrict__ part, unsigned int *__restrict__ counter,
          long long *__restrict__ out, long long *__restrict__ host_out) {
    long long sum = 0, cnt = 0;
    const uint64_t nvec = n >> 2;  // 4 rows per vector: 2x16B deliv, 16B qty, 2x16B amount
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;

    auto row = [&](long long d, int q, long long a) {
        const bool p = pred(d, q);
        sum += p ? a : 0;
        cnt += p;
    };
    for (; v + (kQ6Unroll - 1) * stride < nvec; v += kQ6Unroll * stride) {
        longlong2 d0[kQ6Unroll], d1[kQ6Unroll], a0[kQ6Unroll], a1[kQ6Unroll];
        int4 q[kQ6Unroll];
#pragma unroll
        for (int u = 0; u < kQ6Unroll; ++u) {
            const uint64_t x = v + u * stride;
            d0[u] = ld_stream(deliv + 2 * x);
            d1[u] = ld_stream(deliv + 2 * x + 1);
            q[u] = ld_stream(qty + x);
            a0[u] = ld_stream(amt + 2 * x);
            a1[u] = ld_stream(amt + 2 * x + 1);
        }
#pragma unroll
        for (int u = 0; u < kQ6Unroll; ++u) {
            row(d0[u].x, q[u].x, a0[u].x);
            row(d0[u].y, q[u].y, a0[u].y);
            row(d1[u].x, q[u].z, a1[u].x);
            row(d1[u].y, q[u].w, a1[u].y);
        }
    }
    for (; v < nvec; v += stride) {
        const longlong2 d0 = ld_stream(deliv + 2 * v), d1 = ld_stream(deliv + 2 * v + 1);
        const int4 q = ld_stream(qty + v);
        const longlong2 a0 = ld_stream(amt + 2 * v), a1 = ld_stream(amt + 2 * v + 1);
        row(d0.x, q.x, a0.x);
        row(d0.y, q.y, a0.y);
        row(d1.x, q.z, a1.x);
        row(d1.y, q.w, a1.y);
    }
    {  // ragged tail: rows [4*nvec, n), at most 3, masked by the visible row count
        const uint64_t t = 4 * nvec + (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
        if (t < n) {
            const long long *D = reinterpret_cast<const long long *>(deliv);
            const int *Q = reinterpret_cast<const int *>(qty);
            const long long *A = reinterpret_cast<const long long *>(amt);
            row(D[t], Q[t], A[t]);
        }
    }

    // block reduction: warp shuffles -> shared -> warp 0
    __shared__ long long s_sum[kQ6Threads / 32], s_cnt[kQ6Threads / 32];
    __shared__ bool s_last;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    sum = warp_sum(sum);
    cnt = warp_sum(cnt);
    if (lane == 0) { s_sum[warp] = sum; s_cnt[warp] = cnt; }
    __syncthreads();
    if (warp == 0) {
        sum = lane < kQ6Threads / 32 ? s_sum[lane] : 0;
        cnt = lane < kQ6Threads / 32 ? s_cnt[lane] : 0;
        sum = warp_sum(sum);
        cnt = warp_sum(cnt);
        if (lane == 0) {
            part[2 * blockIdx.x] = sum;
            part[2 * blockIdx.x + 1] = cnt;
            __threadfence();
            const unsigned int ticket = atomicAdd(counter, 1u);
            s_last = ticket == gridDim.x - 1;
        }
    }
    __syncthreads();
    if (s_last) {  // last block to finish folds all block partials (fixed order, exact ints)
        __threadfence();
        long long ts = 0, tc = 0;
        for (unsigned b = threadIdx.x; b < gridDim.x; b += blockDim.x) {
            ts += __ldcg(part + 2 * b);
            tc += __ldcg(part + 2 * b + 1);
        }
        ts = warp_sum(ts);
        tc = warp_sum(tc);
        if (lane == 0) { s_sum[warp] = ts; s_cnt[warp] = tc; }
        __syncthreads();
        if (threadIdx.x == 0) {
            long long S = 0, C = 0;
            for (int w = 0; w < kQ6Threads / 32; ++w) { S += s_sum[w]; C += s_cnt[w]; }
            out[0] = S;
            out[1] = C;
            if (host_out) { host_out[0] = S; host_out[1] = C; }  // mapped pinned: no D2H copy
            *counter = 0;  // self-reset for the next launch
        }
    }
}

// ------------------------------------------------- Q6, TMA-bulk pipelined variant --
// One persistent block per SM: warp 8's elected lane streams 2048-row chunks of the three columns
// into a 4-stage shared-memory ring with cp.async.bulk (mbarrier complete_tx); warps 0-7
// evaluate the predicate from shared memory and release the stage. 160 KB in flight per SM
// without any load registers; same arithmetic and last-block fold as q6_kernel.
constexpr int kTmaConsumerWarps = 8;
constexpr int kTmaThreads = (kTmaConsumerWarps + 1) * 32;
constexpr int kQ6Chunk = 2048;
constexpr int kQ6Stages = 4;
struct Q6TmaSmem {
    long long deliv[kQ6Stages][kQ6Chunk];
    long long amt[kQ6Stages][kQ6Chunk];
    int qty[kQ6Stages][kQ6Chunk];
    uint64_t full[kQ6Stages], empty[kQ6Stages];
};

__global__ void __launch_bounds__(kTmaThreads, 1)
q6_tma_kernel(const long long *__restrict__ deliv, const int *__restrict__ qty,
              const long long *__restrict__ amt, uint64_t n, Q6Pred pred,
              long long *__restrict__ part, unsigned int *__restrict__ counter,
              long long *__restrict__ out, long long *__restrict__ host_out) {
    pdl_wait();
    pdl_trigger();
    extern __shared__ __align__(128) unsigned char smem_raw[];
    Q6TmaSmem &S = *reinterpret_cast<Q6TmaSmem *>(smem_raw);
    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const uint64_t nchunks = (n + kQ6Chunk - 1) / kQ6Chunk;
    if (threadIdx.x == 0) {
        for (int s = 0; s < kQ6Stages; ++s) {
            mbar_init(&S.full[s], 1);
            mbar_init(&S.empty[s], kTmaConsumerWarps);
        }
        fence_mbar_init();
    }
    __syncthreads();
    long long sum = 0, cnt = 0;
    if (warp == kTmaConsumerWarps) {  // producer
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            int it = 0;
            for (uint64_t c = blockIdx.x; c < nchunks; c += gridDim.x, ++it) {
                const int s = it % kQ6Stages;
                const unsigned ph = (unsigned)(it / kQ6Stages) & 1u;
                if (it >= kQ6Stages) mbar_wait(&S.empty[s], ph ^ 1u);
                const uint64_t r0 = c * kQ6Chunk;
                const unsigned rows = (unsigned)(n - r0 < (uint64_t)kQ6Chunk ? n - r0 : (uint64_t)kQ6Chunk);
                const unsigned b8 = round16(rows * 8), b4 = round16(rows * 4);
                mbar_arrive_expect_tx(&S.full[s], 2 * b8 + b4);
                bulk_g2s(S.deliv[s], deliv + r0, b8, &S.full[s], pol);
                bulk_g2s(S.amt[s], amt + r0, b8, &S.full[s], pol);
                bulk_g2s(S.qty[s], qty + r0, b4, &S.full[s], pol);
            }
        }
    } else {  // consumers
        int it = 0;
        for (uint64_t c = blockIdx.x; c < nchunks; c += gridDim.x, ++it) {
            const int s = it % kQ6Stages;
            mbar_wait(&S.full[s], (unsigned)(it / kQ6Stages) & 1u);
            const unsigned rows = (unsigned)(n - c * kQ6Chunk < (uint64_t)kQ6Chunk ? n - c * kQ6Chunk : (uint64_t)kQ6Chunk);
#pragma unroll 4
            for (unsigned r = threadIdx.x; r < rows; r += kTmaConsumerWarps * 32) {
                const long long d = S.deliv[s][r];
                const bool p = pred(d, S.qty[s][r]);
                sum += p ? S.amt[s][r] : 0;
                cnt += p;
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&S.empty[s]);
        }
    }
    // block reduction (9 warps) -> per-block partial -> last block folds all partials
    __shared__ long long s_sum[kTmaConsumerWarps + 1], s_cnt[kTmaConsumerWarps + 1];
    __shared__ bool s_last;
    sum = warp_sum(sum);
    cnt = warp_sum(cnt);
    if (lane == 0) { s_sum[warp] = sum; s_cnt[warp] = cnt; }
    __syncthreads();
    if (threadIdx.x == 0) {
        long long S0 = 0, C0 = 0;
        for (int w = 0; w <= kTmaConsumerWarps; ++w) { S0 += s_sum[w]; C0 += s_cnt[w]; }
        part[2 * blockIdx.x] = S0;
        part[2 * blockIdx.x + 1] = C0;
        __threadfence();
        s_last = atomicAdd(counter, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (s_last && warp == 0) {
        __threadfence();
        long long ts = 0, tc = 0;
        for (unsigned b = lane; b < gridDim.x; b += 32) {
            ts += __ldcg(part + 2 * b);
            tc += __ldcg(part + 2 * b + 1);
        }
        ts = warp_sum(ts);
        tc = warp_sum(tc);
        if (lane == 0) {
            out[0] = ts;
            out[1] = tc;
            if (host_out) { host_out[0] = ts; host_out[1] = tc; }
            *counter = 0;
        }
    }
}

// ================================================================== Q1 ====
constexpr int kQ1Threads = 256;
constexpr int kQ1Unroll = 2;   // 4-row vectors per lane per warp iteration
constexpr int kQ1Sparse = 256; // per-block shared hash slots for keys outside [0, kQ1Dense)

template <int kT> struct Q1SmemT {       // kT aggregating threads
    unsigned int cnt[kQ1Dense][kT];          // [key][thread]: lane-distinct banks, no conflicts
    long long qty[kQ1Dense][kT];
    long long amt[kQ1Dense][kT];
    unsigned long long stag[kQ1Sparse];      // 0 = empty, else (1<<32 | (u32)key)
    unsigned long long sacc[kQ1Sparse][3];
};
using Q1Smem = Q1SmemT<kQ1Threads>;

__device__ __forceinline__ unsigned int hash32(unsigned int x) {
    x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16;
    return x;
}

__device__ void q1_global_add(const Q1Scratch &g, unsigned long long tag, unsigned long long c,
                              long long q, long long a) {
    unsigned int h = hash32((unsigned int)tag) & (kQ1GlobalSlots - 1);
    for (int p = 0; p < kQ1GlobalSlots; ++p) {
        const unsigned long long prev = atomicCAS(g.gtag + h, 0ull, tag);
        if (prev == 0ull || prev == tag) {
            if (prev == 0ull) atomicOr(g.flags, kQ1GlobalUsed);  // the compact must scan the table
            atomicAdd(g.gacc + 3 * h + 0, c);
            atomicAdd(g.gacc + 3 * h + 1, (unsigned long long)q);
            atomicAdd(g.gacc + 3 * h + 2, (unsigned long long)a);
            return;
        }
        h = (h + 1) & (kQ1GlobalSlots - 1);
    }
    atomicOr(g.flags, 1u);  // more distinct groups than kQ1GlobalSlots: reported as ENOMEM
}

template <class Sm>
__device__ void q1_sparse_add(Sm &sm, const Q1Scratch &g, int key, unsigned long long c,
                              long long q, long long a) {
    const unsigned long long tag = (1ull << 32) | (unsigned int)key;
    unsigned int h = hash32((unsigned int)key) & (kQ1Sparse - 1);
    for (int p = 0; p < kQ1Sparse; ++p) {
        const unsigned long long prev = atomicCAS(&sm.stag[h], 0ull, tag);
        if (prev == 0ull || prev == tag) {
            atomicAdd(&sm.sacc[h][0], c);
            atomicAdd(&sm.sacc[h][1], (unsigned long long)q);
            atomicAdd(&sm.sacc[h][2], (unsigned long long)a);
            return;
        }
        h = (h + 1) & (kQ1Sparse - 1);
    }
    q1_global_add(g, tag, c, q, a);  // block table full: go straight to the global table
}

// Warp-aggregated shared-memory atomics: lanes with the same key are grouped (one ballot per
// distinct key present in the warp), their values are reduced with shuffles, and only the
// group leader touches the hash table. Called convergently by all 32 lanes.
template <class Sm>
__device__ __forceinline__ void q1_sparse_warp(Sm &sm, const Q1Scratch &g, bool need, int key,
                                               long long q, long long a) {
    const int lane = threadIdx.x & 31;
    unsigned int pend = __ballot_sync(kFull, need);
    while (pend) {
        const int leader = __ffs(pend) - 1;
        const int lk = __shfl_sync(kFull, key, leader);
        const bool in = need && key == lk;
        const unsigned int grp = __ballot_sync(kFull, in);
        const long long qs = warp_sum(in ? q : 0);
        const long long as = warp_sum(in ? a : 0);
        if (lane == leader) q1_sparse_add(sm, g, lk, __popc(grp), qs, as);
        need = need && !in;
        pend &= ~grp;
    }
}

// Block end: dense keys, one warp per key, one global atomic per (key, accumulator) per block;
// the block's sparse table into the global table. Threads tid < kQ1Threads take part.
template <int kT = kQ1Threads>
__device__ void q1_block_merge(Q1SmemT<kT> &sm, const Q1Scratch &g, int tid) {
    if (tid >= kT) return;
    const int lane = tid & 31, warp = tid >> 5;
    for (int k = warp; k < kQ1Dense; k += kT / 32) {
        long long c = 0, q = 0, a = 0;
        for (int t = lane; t < kT; t += 32) { c += sm.cnt[k][t]; q += sm.qty[k][t]; a += sm.amt[k][t]; }
        c = warp_sum(c); q = warp_sum(q); a = warp_sum(a);
        if (lane == 0 && c) {
            atomicAdd(g.dense + 3 * k + 0, (unsigned long long)c);
            atomicAdd(g.dense + 3 * k + 1, (unsigned long long)q);
            atomicAdd(g.dense + 3 * k + 2, (unsigned long long)a);
        }
    }
    for (int s = tid; s < kQ1Sparse; s += kT)
        if (sm.stag[s]) q1_global_add(g, sm.stag[s], sm.sacc[s][0], (long long)sm.sacc[s][1],
                                      (long long)sm.sacc[s][2]);
}

__global__ void __launch_bounds__(kQ1Threads, 2)
q1_kernel(const int4 *__restrict__ number, const longlong2 *__restrict__ deliv,
          const int4 *__restrict__ qty, const longlong2 *__restrict__ amt, uint64_t n,
          long long cutoff, Q1Scratch g) {
    extern __shared__ __align__(16) unsigned char smem_raw[];
    Q1Smem &sm = *reinterpret_cast<Q1Smem *>(smem_raw);
    const int tid = threadIdx.x, lane = tid & 31;
#pragma unroll
    for (int k = 0; k < kQ1Dense; ++k) { sm.cnt[k][tid] = 0; sm.qty[k][tid] = 0; sm.amt[k][tid] = 0; }
    for (int s = tid; s < kQ1Sparse; s += kQ1Threads) {
        sm.stag[s] = 0; sm.sacc[s][0] = 0; sm.sacc[s][1] = 0; sm.sacc[s][2] = 0;
    }
    if (blockIdx.x == 0 && tid == 0) *g.ngroups = 0;  // consumed by q1_compact (stream-ordered)
    __syncthreads();

    // WHERE ol_delivery_d > cutoff (NULL -> UNKNOWN -> excluded), GROUP BY ol_number
    auto row = [&](bool valid, int key, long long d, int q, long long a, bool &sparse) {
        const bool pass = valid & (d != kNullTs) & (d > cutoff);
        sparse = pass & ((unsigned)key >= (unsigned)kQ1Dense);
        if (pass & ((unsigned)key < (unsigned)kQ1Dense)) {  // thread-private dense slot
            sm.cnt[key][tid] += 1;
            sm.qty[key][tid] += q;
            sm.amt[key][tid] += a;
        }
    };

    const uint64_t nvec = n >> 2;
    const uint64_t gwarp = ((uint64_t)blockIdx.x * kQ1Threads + tid) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * kQ1Threads) >> 5;
    // warp-uniform trip count so that ballots in the sparse path are convergent. Software
    // pipeline: the next iteration's 12 loads are issued before this iteration's rows are
    // aggregated, so HBM requests stay in flight during the shared-memory updates.
    const uint64_t step = nwarps * 32 * kQ1Unroll;
    int4 pnb[kQ1Unroll], pqv[kQ1Unroll];
    longlong2 pd0[kQ1Unroll], pd1[kQ1Unroll], pa0[kQ1Unroll], pa1[kQ1Unroll];
    auto load = [&](uint64_t base) {
#pragma unroll
        for (int u = 0; u < kQ1Unroll; ++u) {
            const uint64_t x = base + u * 32 + lane;
            if (x < nvec) {
                pnb[u] = ld_stream(number + x);
                pd0[u] = ld_stream(deliv + 2 * x);
                pd1[u] = ld_stream(deliv + 2 * x + 1);
                pqv[u] = ld_stream(qty + x);
                pa0[u] = ld_stream(amt + 2 * x);
                pa1[u] = ld_stream(amt + 2 * x + 1);
            }
        }
    };
    load(gwarp * 32 * kQ1Unroll);
    for (uint64_t base = gwarp * 32 * kQ1Unroll; base < nvec; base += step) {
        int4 nb[kQ1Unroll], qv[kQ1Unroll];
        longlong2 d0[kQ1Unroll], d1[kQ1Unroll], a0[kQ1Unroll], a1[kQ1Unroll];
        bool ok[kQ1Unroll];
#pragma unroll
        for (int u = 0; u < kQ1Unroll; ++u) {
            const uint64_t x = base + u * 32 + lane;
            ok[u] = x < nvec;
            if (ok[u]) {
                nb[u] = pnb[u]; d0[u] = pd0[u]; d1[u] = pd1[u]; qv[u] = pqv[u]; a0[u] = pa0[u]; a1[u] = pa1[u];
            } else {
                nb[u] = make_int4(0, 0, 0, 0); qv[u] = nb[u];
                d0[u] = make_longlong2(kNullTs, kNullTs); d1[u] = d0[u];
                a0[u] = make_longlong2(0, 0); a1[u] = a0[u];
            }
        }
        load(base + step);
        bool sp[kQ1Unroll][4];
#pragma unroll
        for (int u = 0; u < kQ1Unroll; ++u) {
            row(ok[u], nb[u].x, d0[u].x, qv[u].x, a0[u].x, sp[u][0]);
            row(ok[u], nb[u].y, d0[u].y, qv[u].y, a0[u].y, sp[u][1]);
            row(ok[u], nb[u].z, d1[u].x, qv[u].z, a1[u].x, sp[u][2]);
            row(ok[u], nb[u].w, d1[u].y, qv[u].w, a1[u].y, sp[u][3]);
        }
        bool any = false;
#pragma unroll
        for (int u = 0; u < kQ1Unroll; ++u) any |= sp[u][0] | sp[u][1] | sp[u][2] | sp[u][3];
        if (__any_sync(kFull, any)) {  // rare for TPC-C data (ol_number in 1..15)
#pragma unroll
            for (int u = 0; u < kQ1Unroll; ++u) {
                q1_sparse_warp(sm, g, sp[u][0], nb[u].x, qv[u].x, a0[u].x);
                q1_sparse_warp(sm, g, sp[u][1], nb[u].y, qv[u].y, a0[u].y);
                q1_sparse_warp(sm, g, sp[u][2], nb[u].z, qv[u].z, a1[u].x);
                q1_sparse_warp(sm, g, sp[u][3], nb[u].w, qv[u].w, a1[u].y);
            }
        }
    }
    if (blockIdx.x == 0 && tid < 32) {  // ragged tail rows [4*nvec, n) (<= 3), warp 0 of block 0
        const uint64_t t = 4 * nvec + lane;
        const bool valid = t < n;
        const int *N = reinterpret_cast<const int *>(number);
        const long long *D = reinterpret_cast<const long long *>(deliv);
        const int *Q = reinterpret_cast<const int *>(qty);
        const long long *A = reinterpret_cast<const long long *>(amt);
        const int key = valid ? N[t] : 0;
        const long long d = valid ? D[t] : kNullTs;
        const int q = valid ? Q[t] : 0;
        const long long a = valid ? A[t] : 0;
        bool sparse;
        row(valid, key, d, q, a, sparse);
        q1_sparse_warp(sm, g, sparse, key, q, a);
    }
    __syncthreads();

    q1_block_merge(sm, g, tid);
}

// Q1, TMA-bulk pipelined variant: one block per SM; the producer warp streams 1024-row chunks of
// the four columns into a 4-stage ring (96 KB) next to 12 aggregating warps' slot tables
// (120 KB): thread-private dense slots, warp-aggregated sparse path (as q1_kernel). 12 warps
// instead of 8: the slot updates are latency-bound.
constexpr int kQ1Chunk = 1024;
// the full pass's extra columns (Q18's join keys), present only in the probe variant
template <int kS, int kC, bool kP> struct ScanKeysT {};
template <int kS, int kC> struct ScanKeysT<kS, kC, true> { int w[kS][kC], d[kS][kC], o[kS][kC]; };
template <int kS, int kC = kQ1Chunk, bool kP = false> struct Q1StagesT {
    long long deliv[kS][kC];
    long long amt[kS][kC];
    int number[kS][kC];
    int qty[kS][kC];
    ScanKeysT<kS, kC, kP> key;
    uint64_t full[kS], empty[kS];
};
// Q1 alone: 12 aggregating warps, 4 stages (216 KB). Shared with Q6: 12 aggregating warps (their
// latency-bound slot updates were the shared pass's limit) and 4 stages (224 KB).
constexpr int kQ6SideWarps = 6;
// The full pass's geometry (build-time constants for A/B variants,
// scripts/build_variants.py). Measured at W = 100 (pass time): 12 Q1 warps / 3 stages / 7 probe
// warps 297 us — each probe warp must finish one ~300-instruction step per chunk, a latency chain
// of shuffles; two probe groups taking alternate chunks 200-206 us; 8 Q1 warps / 4 stages / 896-row
// chunks / 2 x 7 probe warps / 4 Q6 warps 191 us (the default); 768-row chunks x 5 stages 208 us,
// 6 Q1 warps x 5 stages 211 us; a try_wait suspend hint: no change.
#ifndef H2TAP_FULL_DIAG
#define H2TAP_FULL_DIAG 0   // A/B diagnosis only: 1 = the probe warps skip their step (wrong Q18)
#endif
#ifndef H2TAP_FULL_W
#define H2TAP_FULL_W 8      // Q1 aggregating warps
#endif
#ifndef H2TAP_FULL_S
#define H2TAP_FULL_S 4      // ring stages
#endif
#ifndef H2TAP_FULL_C
#define H2TAP_FULL_C 896    // rows per chunk (a multiple of 128: one probe warp step per 128 rows)
#endif
#ifndef H2TAP_FULL_PG
#define H2TAP_FULL_PG 2     // probe warp groups; group g takes the chunks it == g (mod PG)
#endif
#ifndef H2TAP_FULL_Q6W
#define H2TAP_FULL_Q6W 4    // Q6 side warps in the full pass
#endif
#ifndef H2TAP_FULL_SLEEP_NS
#define H2TAP_FULL_SLEEP_NS 0  // consumer waits: try_wait suspend-time hint (0: none)
#endif
template <bool kQ6, bool kProbe = false> struct Q1TmaCfg {
    static constexpr int kW = kProbe ? H2TAP_FULL_W : 12;           // aggregating warps
    static constexpr int kT = kW * 32;
    static constexpr int kS = kProbe ? H2TAP_FULL_S : 4;            // ring stages
    static constexpr int kC = kProbe ? H2TAP_FULL_C : kQ1Chunk;     // rows per chunk
    static constexpr int kQ6W = kQ6 ? (kProbe ? H2TAP_FULL_Q6W : kQ6SideWarps) : 0;  // Q6 side warps
    static constexpr int kPG = kProbe ? H2TAP_FULL_PG : 1;            // probe warp groups
    static constexpr int kPW = kProbe ? kC / 128 : 0;                // Q18 probe warps per group
    static constexpr int kThreads = (kW + 1 + kQ6W + kPG * kPW) * 32;
    using Stages = Q1StagesT<kS, kC, kProbe>;
    static constexpr size_t kSmem = sizeof(Stages) + sizeof(Q1SmemT<kT>);
    static_assert(!kProbe || kC % 128 == 0, "probe warps take 128-row steps");
};

// kQ6: shared scan of a batch's Q6 and Q1 — Q6 reads a subset of Q1's columns
// (ol_delivery_d, ol_quantity, ol_amount), so the same staged chunk also feeds Q6's predicate and
// sum; the block tail adds Q6's reduction (as q6_tma_kernel). One pass over 24 B/row instead of
// 20 + 24.
// Shared-scan block: warps 0-11 Q1, warp 12 the producer, then the Q6 side warps on the same
// staged chunks (registers only) — Q6 added to the Q1 warps' rows lengthened their dependent
// shared-memory update chains (145 vs 117 us); separate warps run it alongside.
// kProbe (the batch's full pass): the chunks also carry Q18's join keys
// (ol_w_id, ol_d_id, ol_o_id) and kC / 128 probe warps run the K4 warp step (probe_device.cuh)
// on them: the batch reads order_line once, 36 B/row, instead of 24 + 20 B/row (ol_amount is
// shared by all three queries). The orders join index must be built before the pass.
constexpr int kQ61Threads = Q1TmaCfg<true>::kThreads;
template <bool kQ6, bool kProbe = false>
__global__ void __launch_bounds__(Q1TmaCfg<kQ6, kProbe>::kThreads, 1)
q1_tma_kernel(const int *__restrict__ number, const long long *__restrict__ deliv,
              const int *__restrict__ qty, const long long *__restrict__ amt, uint64_t n,
              long long cutoff, Q1Scratch g, Q6Pred pred6, long long *__restrict__ part6,
              unsigned int *__restrict__ counter6, long long *__restrict__ out6,
              long long *__restrict__ host_out6, const int *__restrict__ ol_w,
              const int *__restrict__ ol_d, const int *__restrict__ ol_o, Q18Scratch ps) {
    pdl_wait();
    pdl_trigger();
    extern __shared__ __align__(128) unsigned char smem_raw[];
    using Cfg = Q1TmaCfg<kQ6, kProbe>;
    constexpr int kQ1W = Cfg::kW, kQ1T = Cfg::kT, kQ1Stages = Cfg::kS, kC = Cfg::kC;
    constexpr int kQ6W = Cfg::kQ6W, kPW = Cfg::kPW, kPG = Cfg::kPG;
    typename Cfg::Stages &P = *reinterpret_cast<typename Cfg::Stages *>(smem_raw);
    Q1SmemT<kQ1T> &sm = *reinterpret_cast<Q1SmemT<kQ1T> *>(smem_raw + sizeof(typename Cfg::Stages));
    auto wait_full = [&](int s, int it) {
        if constexpr (kProbe && H2TAP_FULL_SLEEP_NS > 0)
            mbar_wait_hint(&P.full[s], (unsigned)(it / kQ1Stages) & 1u, H2TAP_FULL_SLEEP_NS);
        else
            mbar_wait(&P.full[s], (unsigned)(it / kQ1Stages) & 1u);
    };
    const int tid = threadIdx.x, lane = tid & 31, warp = tid >> 5;
    long long sum6 = 0, cnt6 = 0;  // kQ6 only
    if (tid < kQ1T) {
#pragma unroll
        for (int k = 0; k < kQ1Dense; ++k) { sm.cnt[k][tid] = 0; sm.qty[k][tid] = 0; sm.amt[k][tid] = 0; }
        for (int s = tid; s < kQ1Sparse; s += kQ1T) {
            sm.stag[s] = 0; sm.sacc[s][0] = 0; sm.sacc[s][1] = 0; sm.sacc[s][2] = 0;
        }
    }
    if (tid == 0) {
        for (int s = 0; s < kQ1Stages; ++s) {
            mbar_init(&P.full[s], 1);
            mbar_init(&P.empty[s], kQ1W + kQ6W + kPW);
        }
        fence_mbar_init();
        if (blockIdx.x == 0) *g.ngroups = 0;  // consumed by q1_compact (stream-ordered)
    }
    __syncthreads();
    const uint64_t nchunks = (n + kC - 1) / kC;
    if (warp == kQ1W) {  // producer
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            int it = 0;
            for (uint64_t c = blockIdx.x; c < nchunks; c += gridDim.x, ++it) {
                const int s = it % kQ1Stages;
                const unsigned ph = (unsigned)(it / kQ1Stages) & 1u;
                if (it >= kQ1Stages) mbar_wait(&P.empty[s], ph ^ 1u);
                const uint64_t r0 = c * kC;
                const unsigned rows = (unsigned)(n - r0 < (uint64_t)kC ? n - r0 : (uint64_t)kC);
                const unsigned b8 = round16(rows * 8), b4 = round16(rows * 4);
                mbar_arrive_expect_tx(&P.full[s], 2 * b8 + (kProbe ? 5 : 2) * b4);
                bulk_g2s(P.deliv[s], deliv + r0, b8, &P.full[s], pol);
                bulk_g2s(P.amt[s], amt + r0, b8, &P.full[s], pol);
                bulk_g2s(P.number[s], number + r0, b4, &P.full[s], pol);
                bulk_g2s(P.qty[s], qty + r0, b4, &P.full[s], pol);
                if constexpr (kProbe) {
                    bulk_g2s(P.key.w[s], ol_w + r0, b4, &P.full[s], pol);
                    bulk_g2s(P.key.d[s], ol_d + r0, b4, &P.full[s], pol);
                    bulk_g2s(P.key.o[s], ol_o + r0, b4, &P.full[s], pol);
                }
            }
        }
    } else if (kProbe && warp > kQ1W + kQ6W) {  // Q18 probe warps: one 128-row step per chunk each
      if constexpr (kProbe) {
        using namespace pd;
        const bool ident = jx::jx_identity(ps.jo);  // read once (after pdl_wait: verify has run)
        const int pw = (warp - (kQ1W + 1 + kQ6W)) % kPW, pg = (warp - (kQ1W + 1 + kQ6W)) / kPW;
        static_assert(kPW == kC / 128, "one 128-row step per probe warp per chunk");
        int it = pg;
        for (uint64_t c = blockIdx.x + (uint64_t)pg * gridDim.x; c < nchunks; c += (uint64_t)kPG * gridDim.x, it += kPG) {
            const int s = it % kQ1Stages;
            wait_full(s, it);
            const unsigned rows = (unsigned)(n - c * kC < (uint64_t)kC ? n - c * kC : (uint64_t)kC);
            const unsigned r = pw * 128 + lane * 4;  // this lane's 4 consecutive rows
            H2TAP_CHECK(rows <= (unsigned)kC && (c * kC + rows <= n) && s < kQ1Stages);
            Key3 k[4];
            long long a[4];
            const bool valid = r + 3 < rows;
            if (valid) {
                const int4 W = *reinterpret_cast<const int4 *>(&P.key.w[s][r]);
                const int4 D = *reinterpret_cast<const int4 *>(&P.key.d[s][r]);
                const int4 O = *reinterpret_cast<const int4 *>(&P.key.o[s][r]);
                const longlong2 A0 = *reinterpret_cast<const longlong2 *>(&P.amt[s][r]);
                const longlong2 A1 = *reinterpret_cast<const longlong2 *>(&P.amt[s][r + 2]);
                k[0] = {W.x, D.x, O.x}; k[1] = {W.y, D.y, O.y}; k[2] = {W.z, D.z, O.z}; k[3] = {W.w, D.w, O.w};
                a[0] = A0.x; a[1] = A0.y; a[2] = A1.x; a[3] = A1.y;
            } else {
                for (int j = 0; j < 4; ++j) { k[j] = {0, 0, 0}; a[j] = 0; }
            }
            // rows of a partial last group (< 4, last chunk only) go one by one
            if (!valid && r < rows)
                for (unsigned j = r; j < rows; ++j)
                    flush_run<false>(ps, Key3{P.key.w[s][j], P.key.d[s][j], P.key.o[s][j]}, P.amt[s][j], 1u, ident);
            // the stage is released before the step (the step works on registers)
            __syncwarp();
            if (lane == 0) mbar_arrive(&P.empty[s]);
#if H2TAP_FULL_DIAG != 1
            probe_lane_group<false>(ps, k, a, valid, lane, ident);
#else
            if (a[0] == 0x7fffffffffffffffll && k[0].w == 12345) probe_lane_group<false>(ps, k, a, valid, lane, ident);
#endif
        }
      }
    } else if (kQ6 && warp > kQ1W) {  // Q6 side warps: 4 row pairs each
        // the predicate as two unsigned range tests (same result as Q6Pred: a NULL date is
        // INT64_MIN, below every lower bound > INT64_MIN; an empty range passes nothing)
        const long long dlo = pred6.d_lo > kNullTs ? pred6.d_lo : kNullTs + 1;
        const unsigned long long dspan = pred6.d_hi > dlo ? (unsigned long long)pred6.d_hi - (unsigned long long)dlo : 0ull;
        const bool qempty = pred6.q_lo > pred6.q_hi;
        const unsigned long long qspan = (unsigned long long)pred6.q_hi - (unsigned long long)pred6.q_lo;
        auto pass = [&](long long d, int q) {
            return ((unsigned long long)d - (unsigned long long)dlo < dspan) &
                   ((unsigned long long)(long long)q - (unsigned long long)pred6.q_lo <= qspan) & !qempty;
        };
        const int t6 = tid - (kQ1W + 1) * 32;
        unsigned int c32 = 0;
        int it = 0;
        for (uint64_t c = blockIdx.x; c < nchunks; c += gridDim.x, ++it) {
            const int s = it % kQ1Stages;
            wait_full(s, it);
            const unsigned rows = (unsigned)(n - c * kC < (uint64_t)kC ? n - c * kC : (uint64_t)kC);
            if (rows == (unsigned)kC) {  // full chunk: 128-bit / 64-bit shared loads of pairs
                constexpr int kPairs = kC / 2, kStep = kQ6W * 32;
#pragma unroll
                for (int k = 0; k < (kPairs + kStep - 1) / kStep; ++k) {
                    const unsigned pr = t6 + k * kStep;
                    if (kPairs % kStep != 0 && pr >= (unsigned)kPairs) break;
                    const longlong2 d2 = reinterpret_cast<const longlong2 *>(P.deliv[s])[pr];
                    const longlong2 a2 = reinterpret_cast<const longlong2 *>(P.amt[s])[pr];
                    const int2 q2 = reinterpret_cast<const int2 *>(P.qty[s])[pr];
                    const bool p0 = pass(d2.x, q2.x), p1 = pass(d2.y, q2.y);
                    sum6 += (p0 ? a2.x : 0) + (p1 ? a2.y : 0);
                    c32 += (unsigned)p0 + (unsigned)p1;
                }
            } else {
                for (unsigned r = t6; r < rows; r += kQ6W * 32) {
                    const bool p0 = pass(P.deliv[s][r], P.qty[s][r]);
                    sum6 += p0 ? P.amt[s][r] : 0;
                    c32 += p0;
                }
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&P.empty[s]);
        }
        cnt6 = c32;
    } else {  // Q1 consumers: 256 threads, 4 rows each per chunk (warp-uniform trip count)
        int it = 0;
        for (uint64_t c = blockIdx.x; c < nchunks; c += gridDim.x, ++it) {
            const int s = it % kQ1Stages;
            wait_full(s, it);
            const unsigned rows = (unsigned)(n - c * kC < (uint64_t)kC ? n - c * kC : (uint64_t)kC);
            // all four rows' loads first: the stage and the tables share one shared-memory
            // buffer, so loads after a table store would wait for it (possible aliasing)
            constexpr int kU = (kC + kQ1T - 1) / kQ1T;
            int keys[kU], qs[kU];
            long long ds[kU], as[kU];
#pragma unroll
            for (int u = 0; u < kU; ++u) {
                const unsigned r = u * kQ1T + tid;
                const bool valid = r < rows;
                keys[u] = valid ? P.number[s][r] : 0;
                ds[u] = valid ? P.deliv[s][r] : kNullTs;
                qs[u] = valid ? P.qty[s][r] : 0;
                as[u] = valid ? P.amt[s][r] : 0;
            }
#pragma unroll
            for (int u = 0; u < kU; ++u) {
                const unsigned r = u * kQ1T + tid;
                const bool valid = r < rows;
                const int key = keys[u];
                const long long d = ds[u];
                const int q = qs[u];
                const long long a = as[u];
                // WHERE ol_delivery_d > cutoff (NULL -> UNKNOWN -> excluded), GROUP BY ol_number
                const bool pass = valid & (d != kNullTs) & (d > cutoff);
                const bool sparse = pass & ((unsigned)key >= (unsigned)kQ1Dense);
                if (pass & ((unsigned)key < (unsigned)kQ1Dense)) {
                    sm.cnt[key][tid] += 1;
                    sm.qty[key][tid] += q;
                    sm.amt[key][tid] += a;
                }
                if (__any_sync(kFull, sparse)) q1_sparse_warp(sm, g, sparse, key, q, a);
            }
            __syncwarp();
            if (lane == 0) mbar_arrive(&P.empty[s]);
        }
    }
    __syncthreads();
    q1_block_merge<kQ1T>(sm, g, tid);
    if (kQ6) {  // Q6: block reduction -> per-block partial -> last block folds (q6_tma_kernel)
        constexpr int kW = Cfg::kThreads / 32;
        __shared__ long long s_sum[kW], s_cnt[kW];
        __shared__ bool s_last;
        sum6 = warp_sum(sum6);
        cnt6 = warp_sum(cnt6);
        if (lane == 0) { s_sum[warp] = sum6; s_cnt[warp] = cnt6; }
        __syncthreads();
        if (tid == 0) {
            long long S0 = 0, C0 = 0;
            for (int w = 0; w < kW; ++w) { S0 += s_sum[w]; C0 += s_cnt[w]; }
            part6[2 * blockIdx.x] = S0;
            part6[2 * blockIdx.x + 1] = C0;
            __threadfence();
            s_last = atomicAdd(counter6, 1u) == gridDim.x - 1;
        }
        __syncthreads();
        if (s_last && warp == 0) {
            __threadfence();
            long long ts = 0, tc = 0;
            for (unsigned b = lane; b < gridDim.x; b += 32) {
                ts += __ldcg(part6 + 2 * b);
                tc += __ldcg(part6 + 2 * b + 1);
            }
            ts = warp_sum(ts);
            tc = warp_sum(tc);
            if (lane == 0) {
                out6[0] = ts;
                out6[1] = tc;
                if (host_out6) { host_out6[0] = ts; host_out6[1] = tc; }
                *counter6 = 0;
            }
        }
    }
}

// Collect the dense and global tables into groups[] and clear them for the next query. When no
// group reached the global table (kQ1GlobalUsed clear: every key was dense, the TPC-C case) block
// 0 alone does it and also writes the ranked output (dense keys are already in key order), and
// q1_emit only publishes the counts (kQ1Emitted): one warp instead of a 64 K-slot scan + rank.
__global__ void q1_compact_kernel(Q1Scratch g) {
    pdl_wait();
    pdl_trigger();
    if (!(*reinterpret_cast<volatile unsigned int *>(g.flags) & kQ1GlobalUsed)) {
        if (blockIdx.x != 0 || threadIdx.x >= 32) return;
        const int lane = threadIdx.x;
        unsigned long long c = 0, qs = 0, as = 0;
        if (lane < kQ1Dense) { c = g.dense[3 * lane]; qs = g.dense[3 * lane + 1]; as = g.dense[3 * lane + 2]; }
        const unsigned present = __ballot_sync(kFull, c != 0);
        if (c) {
            const int r = __popc(present & ((1u << lane) - 1u));  // rank = key order
            g.groups[r] = Q1Group{(long long)lane, (long long)c, (long long)qs, (long long)as};
            g.o_key[r] = lane;
            g.o_qty[r] = (long long)qs;
            g.o_amt[r] = (long long)as;
            g.o_cnt[r] = (long long)c;
            g.o_avg_qty[r] = (double)(long long)qs / (double)(long long)c;
            g.o_avg_amt[r] = ((double)(long long)as / (double)(long long)c) / 100.0;
            g.dense[3 * lane] = g.dense[3 * lane + 1] = g.dense[3 * lane + 2] = 0;
        }
        if (lane == 0) {
            *g.ngroups = __popc(present);
            atomicOr(g.flags, kQ1Emitted);
        }
        return;
    }
    const uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
    if (i == 0) atomicAnd(g.flags, ~kQ1Emitted);
    if (i < (uint64_t)kQ1Dense) {
        const unsigned long long c = g.dense[3 * i];
        if (c) {
            const unsigned long long p = atomicAdd(g.ngroups, 1ull);
            g.groups[p] = Q1Group{(long long)i, (long long)c, (long long)g.dense[3 * i + 1],
                                  (long long)g.dense[3 * i + 2]};
            g.dense[3 * i] = g.dense[3 * i + 1] = g.dense[3 * i + 2] = 0;
        }
    }
    if (i < (uint64_t)kQ1GlobalSlots) {
        const unsigned long long tag = g.gtag[i];
        if (tag) {
            const unsigned long long p = atomicAdd(g.ngroups, 1ull);
            g.groups[p] = Q1Group{(long long)(int)(unsigned int)tag, (long long)g.gacc[3 * i],
                                  (long long)g.gacc[3 * i + 1], (long long)g.gacc[3 * i + 2]};
            g.gtag[i] = 0;
            g.gacc[3 * i] = g.gacc[3 * i + 1] = g.gacc[3 * i + 2] = 0;
        }
    }
}

__global__ void __launch_bounds__(256) q1_peer_merge_kernel(PeerArgs p, Q1Scratch g) {
    pdl_wait();
    pdl_trigger();
    const unsigned long long s = peer::cur_seq(p);
    if (blockIdx.x == 0 && threadIdx.x == 0) *g.ngroups = 0;
    const int par = (int)(s & 1);
    const unsigned long long stride = (unsigned long long)gridDim.x * blockDim.x;
    for (int k = 0; k < p.world; ++k) {
        const char *slot = peer::mbox(p, p.rank, par, k);
        const unsigned long long n = *reinterpret_cast<const volatile unsigned long long *>(slot);
        const Q1Group *list = reinterpret_cast<const Q1Group *>(slot + 16);
        for (unsigned long long i = (unsigned long long)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
            // (.cg: peer-written data is read from L2, never from a possibly stale L1 line)
            const longlong2 a = __ldcg(reinterpret_cast<const longlong2 *>(list + i));
            const longlong2 b = __ldcg(reinterpret_cast<const longlong2 *>(list + i) + 1);
            const Q1Group x{a.x, a.y, b.x, b.y};
            q1_global_add(g, (1ull << 32) | (unsigned int)(int)x.key, (unsigned long long)x.cnt, x.qty, x.amt);
        }
    }
}

// ORDER BY ol_number: keys are distinct, so each group's output position is its rank
// (number of smaller keys). AVG = SUM / COUNT in IEEE double, money / 100 (R7).
__global__ void q1_emit_kernel(Q1Scratch g) {
    pdl_wait();
    pdl_trigger();
    __shared__ long long tile[1024];
    const uint64_t ng = *g.ngroups;  // read on the device: no host round trip before emitting
    const unsigned fl = *reinterpret_cast<volatile unsigned int *>(g.flags);
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        if (g.host_small) {  // mapped pinned: no D2H copies
            g.host_small[0] = ng;
            reinterpret_cast<unsigned int *>(g.host_small)[2] = fl & 1u;
        }
        atomicAnd(g.flags, ~kQ1GlobalUsed);  // the compact has emptied the global table
    }
    if (fl & kQ1Emitted) return;  // the compact wrote the output (dense keys only)
    if ((uint64_t)blockIdx.x * blockDim.x >= ng) return;  // grid sized for the maximum
    const uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
    const long long mine = i < ng ? g.groups[i].key : 0;
    uint64_t rank = 0;
    for (uint64_t t0 = 0; t0 < ng; t0 += 1024) {
        for (uint64_t t = threadIdx.x; t < 1024 && t0 + t < ng; t += blockDim.x)
            tile[t] = g.groups[t0 + t].key;
        __syncthreads();
        const uint64_t lim = ng - t0 < 1024 ? ng - t0 : 1024;
        for (uint64_t t = 0; t < lim; ++t) rank += tile[t] < mine;
        __syncthreads();
    }
    if (i < ng) {
        const Q1Group x = g.groups[i];
        g.o_key[rank] = (int32_t)x.key;
        g.o_qty[rank] = x.qty;
        g.o_amt[rank] = x.amt;
        g.o_cnt[rank] = x.cnt;
        g.o_avg_qty[rank] = (double)x.qty / (double)x.cnt;
        g.o_avg_amt[rank] = ((double)x.amt / (double)x.cnt) / 100.0;
    }
}

}  // namespace

// ------------------------------------------------------------------ launchers --
int q6_max_blocks(int num_sms) { return num_sms * 8; }

void launch_q6(const int64_t *deliv, const int32_t *qty, const int64_t *amt, uint64_t n,
               int64_t d_lo, int64_t d_hi, int64_t q_lo, int64_t q_hi, const Q6Scratch &s,
               int num_sms, cudaStream_t st) {
    static int occ = 0;
    if (!occ) cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, q6_kernel, kQ6Threads, 0);
    int per_sm = occ < 8 ? (occ > 0 ? occ : 1) : 8;
    uint64_t want = ((n >> 2) + kQ6Threads - 1) / kQ6Threads;
    uint64_t grid = (uint64_t)num_sms * per_sm;
    if (want < grid) grid = want ? want : 1;
    q6_kernel<<<(unsigned)grid, kQ6Threads, 0, st>>>(
        reinterpret_cast<const longlong2 *>(deliv), reinterpret_cast<const int4 *>(qty),
        reinterpret_cast<const longlong2 *>(amt), n, Q6Pred{d_lo, d_hi, q_lo, q_hi},
        s.block_part, s.done_counter, s.out, s.host_out);
        count_launches(1);
}

// SMs the TMA scans use (H2TAP_SCAN_SMS, A/B: a scan on part of the GPU, the rest free for
// concurrent work)
int scan_sms(int num_sms) {
    static const int lim = [] { const char *v = std::getenv("H2TAP_SCAN_SMS"); return v ? std::atoi(v) : 0; }();
    return lim > 0 && lim < num_sms ? lim : num_sms;
}

void launch_q6_tma(const int64_t *deliv, const int32_t *qty, const int64_t *amt, uint64_t n,
                   int64_t d_lo, int64_t d_hi, int64_t q_lo, int64_t q_hi, const Q6Scratch &s,
                   int num_sms, cudaStream_t st) {
    const uint64_t nchunks = (n + kQ6Chunk - 1) / kQ6Chunk;
    const unsigned grid = (unsigned)std::max<uint64_t>(1, std::min<uint64_t>(nchunks, (uint64_t)scan_sms(num_sms)));
    launch_pdl(q6_tma_kernel, grid, kTmaThreads, sizeof(Q6TmaSmem), st,
        reinterpret_cast<const long long *>(deliv), qty, reinterpret_cast<const long long *>(amt), n,
        Q6Pred{d_lo, d_hi, q_lo, q_hi}, s.block_part, s.done_counter, s.out, s.host_out);
    count_launches(1);
}

void launch_q1_reset(const Q1Scratch &s, cudaStream_t st) {
    cudaMemsetAsync(s.dense, 0, sizeof(unsigned long long) * kQ1Dense * 3, st);
    cudaMemsetAsync(s.gtag, 0, sizeof(unsigned long long) * kQ1GlobalSlots, st);
    cudaMemsetAsync(s.gacc, 0, sizeof(unsigned long long) * kQ1GlobalSlots * 3, st);
    cudaMemsetAsync(s.flags, 0, sizeof(unsigned int), st);
    cudaMemsetAsync(s.ngroups, 0, sizeof(unsigned long long), st);
}

void launch_q1(const int32_t *number, const int64_t *deliv, const int32_t *qty,
               const int64_t *amt, uint64_t n, int64_t cutoff, const Q1Scratch &s, int num_sms,
               cudaStream_t st) {
    uint64_t want = ((n >> 2) + kQ1Threads - 1) / kQ1Threads;
    uint64_t grid = (uint64_t)num_sms * 2;
    if (want < grid) grid = want ? want : 1;
    q1_kernel<<<(unsigned)grid, kQ1Threads, sizeof(Q1Smem), st>>>(
        reinterpret_cast<const int4 *>(number), reinterpret_cast<const longlong2 *>(deliv),
        reinterpret_cast<const int4 *>(qty), reinterpret_cast<const longlong2 *>(amt), n, cutoff,
        s);
        count_launches(1);
}

void launch_q1_tma(const int32_t *number, const int64_t *deliv, const int32_t *qty,
                   const int64_t *amt, uint64_t n, int64_t cutoff, const Q1Scratch &s, int num_sms,
                   cudaStream_t st) {
    using Cfg = Q1TmaCfg<false>;
    const uint64_t nchunks = (n + Cfg::kC - 1) / Cfg::kC;
    const unsigned grid = (unsigned)std::max<uint64_t>(1, std::min<uint64_t>(nchunks, (uint64_t)scan_sms(num_sms)));
    launch_pdl(q1_tma_kernel<false>, grid, Cfg::kThreads, Cfg::kSmem, st, number, reinterpret_cast<const long long *>(deliv), qty,
               reinterpret_cast<const long long *>(amt), n, cutoff, s, Q6Pred{0, 0, 0, 0}, nullptr, nullptr,
               nullptr, nullptr, nullptr, nullptr, nullptr, Q18Scratch{});
    count_launches(1);
}

void launch_q61_tma(const int32_t *number, const int64_t *deliv, const int32_t *qty,
                    const int64_t *amt, uint64_t n, int64_t cutoff, const Q1Scratch &s, int64_t d_lo,
                    int64_t d_hi, int64_t q_lo, int64_t q_hi, const Q6Scratch &s6, int num_sms,
                    cudaStream_t st) {
    using Cfg = Q1TmaCfg<true>;
    const uint64_t nchunks = (n + Cfg::kC - 1) / Cfg::kC;
    const unsigned grid = (unsigned)std::max<uint64_t>(1, std::min<uint64_t>(nchunks, (uint64_t)scan_sms(num_sms)));
    launch_pdl(q1_tma_kernel<true>, grid, Cfg::kThreads, Cfg::kSmem, st, number, reinterpret_cast<const long long *>(deliv),
               qty, reinterpret_cast<const long long *>(amt), n, cutoff, s, Q6Pred{d_lo, d_hi, q_lo, q_hi},
               s6.block_part, s6.done_counter, s6.out, s6.host_out, nullptr, nullptr, nullptr, Q18Scratch{});
    count_launches(1);
}

void launch_q6118_tma(const int32_t *number, const int64_t *deliv, const int32_t *qty, const int64_t *amt,
                      const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o, uint64_t n, int64_t cutoff,
                      const Q1Scratch &s, int64_t d_lo, int64_t d_hi, int64_t q_lo, int64_t q_hi,
                      const Q6Scratch &s6, const Q18Scratch &s18, int num_sms, cudaStream_t st) {
    using Cfg = Q1TmaCfg<true, true>;
    const uint64_t nchunks = (n + Cfg::kC - 1) / Cfg::kC;
    const unsigned grid = (unsigned)std::max<uint64_t>(1, std::min<uint64_t>(nchunks, (uint64_t)scan_sms(num_sms)));
    launch_pdl(q1_tma_kernel<true, true>, grid, Cfg::kThreads, Cfg::kSmem, st, number,
               reinterpret_cast<const long long *>(deliv), qty, reinterpret_cast<const long long *>(amt), n, cutoff,
               s, Q6Pred{d_lo, d_hi, q_lo, q_hi}, s6.block_part, s6.done_counter, s6.out, s6.host_out, ol_w, ol_d,
               ol_o, s18);
    count_launches(1);
}

void launch_q1_compact(const Q1Scratch &s, cudaStream_t st) {
    launch_pdl(q1_compact_kernel, kQ1GlobalSlots / 256, 256, 0, st, s);
    count_launches(1);
}

void launch_q1_peer_merge(const PeerArgs &p, const Q1Scratch &s, int num_sms, cudaStream_t st) {
    launch_pdl(q1_peer_merge_kernel, (unsigned)num_sms, 256, 0, st, p, s);
    count_launches(1);
}

void launch_q1_emit(const Q1Scratch &s, uint64_t max_groups, cudaStream_t st) {
    launch_pdl(q1_emit_kernel, (unsigned)((max_groups + 255) / 256), 256, 0, st, s);
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

cudaError_t set_attributes_scan(int num_sms) {
    static const void *const kKernels[] = {
        (const void *)q1_compact_kernel,
        (const void *)q1_emit_kernel,
        (const void *)q1_kernel,
        (const void *)q1_peer_merge_kernel,
        (const void *)q1_tma_kernel<false>,
        (const void *)q1_tma_kernel<true>,
        (const void *)q1_tma_kernel<true, true>,
        (const void *)q6_kernel,
        (const void *)q6_tma_kernel};
    const cudaError_t le = force_load(kKernels, sizeof kKernels / sizeof kKernels[0]);
    if (le != cudaSuccess) return le;

    (void)num_sms;
    cudaError_t e = cudaFuncSetAttribute(q6_tma_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                         (int)sizeof(Q6TmaSmem));
    if (e == cudaSuccess)
        e = cudaFuncSetAttribute(q1_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sizeof(Q1Smem));
    if (e == cudaSuccess)
        e = cudaFuncSetAttribute(q1_tma_kernel<false>, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                 (int)Q1TmaCfg<false>::kSmem);
    if (e == cudaSuccess)
        e = cudaFuncSetAttribute(q1_tma_kernel<true>, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                 (int)Q1TmaCfg<true>::kSmem);
    if (e == cudaSuccess)
        e = cudaFuncSetAttribute(q1_tma_kernel<true, true>, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                 (int)Q1TmaCfg<true, true>::kSmem);
    return e;
}

}  // namespace h2tap
