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
#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <cuda_runtime.h>

#include "bulk_pipeline.cuh"
#include "cache_hints.cuh"
#include "join_index.cuh"
#include "kernels.cuh"
#include "probe_device.cuh"

namespace h2tap {
namespace {
using namespace jx;
using namespace pd;

constexpr unsigned kFull = 0xffffffffu;

unsigned grid_for(uint64_t work, int threads, int num_sms, int per_sm) {
    uint64_t want = (work + threads - 1) / threads;
    uint64_t cap = (uint64_t)num_sms * per_sm;
    if (want > cap) want = cap;
    return want ? (unsigned)want : 1u;
}

// ------------------------------------------------------------------- init --
// Empties both join indexes, zeroes the group accumulators and the counters: one launch.
// Empties both join indexes, zeroes the group accumulators and the counters: one launch.
// Does every build row sit at its own dense slot (row == rank of its key in the box)? Counts the
// rows that do not (a warp-aggregated atomic per warp with any): 0 = the index is the identity.
__device__ __forceinline__ void verify_identity(const JoinIndex &j, const int32_t *w, const int32_t *d,
                                                const int32_t *id, uint64_t n, Q18Acc *acc = nullptr) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    const uint64_t n_pad = (n + 31) & ~31ull;  // whole warps (ballot)
    constexpr int U = 4;                       // independent key loads in flight per thread
    // the zeroed accumulators stay in L2 for the probe's atomics (48 MB at W=100 of the 126 MB;
    // probe 103 -> 101 us measured)
    const uint64_t keep = l2_policy_evict_last();
    for (uint64_t r0 = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; r0 < n_pad; r0 += U * stride) {
        int kw[U], kd[U], ki[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t r = r0 + u * stride;
            if (r < n) { kw[u] = __ldcs(w + r); kd[u] = __ldcs(d + r); ki[u] = __ldcs(id + r); }
        }
        unsigned int bad = 0;
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t r = r0 + u * stride;
            unsigned long long s;
            bad += r < n && (!dense_slot(j, kw[u], kd[u], ki[u], s) || s != r);
            if (acc && r < n) st16_policy(reinterpret_cast<ulonglong2 *>(acc) + r, 0ull, 0ull, keep);
        }
        const unsigned int b = __ballot_sync(__activemask(), bad != 0);
        if (b && (threadIdx.x & 31) == __ffs(b) - 1) atomicAdd(j.viol, 1u);  // (a count > 0 suffices)
    }
}

// Clustered build sides: count the rows not at their own dense slot; reset the
// counters of the next query. Runs before the init, which then need not clear an identity index.
__global__ void q18_verify_kernel(Q18Scratch s, const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                                  const int32_t *__restrict__ o_id, uint64_t n_o, const int32_t *__restrict__ c_w,
                                  const int32_t *__restrict__ c_d, const int32_t *__restrict__ c_id, uint64_t n_c) {
    pdl_wait();
    pdl_trigger();
    if (s.jo.may_ident) verify_identity(s.jo, o_w, o_d, o_id, n_o, s.acc);  // (+ zeroes acc: no build pass)
    if (s.jc.may_ident) verify_identity(s.jc, c_w, c_d, c_id, n_c);
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        if (s.jo.viol_next) *s.jo.viol_next = 0u;
        if (s.jc.viol_next) *s.jc.viol_next = 0u;
    }
}

__global__ void q18_init_kernel(Q18Scratch s) {
    pdl_wait();
    pdl_trigger();
    // an identity index is never read: nothing to clear (the verify kernel ran before)
    const uint64_t a = jx_identity(s.jo) ? 0 : jx_words(s.jo), b = jx_identity(s.jc) ? 0 : jx_words(s.jc);
    const uint64_t q = s.qbits ? s.qwords : 0;
    const uint64_t total = a + b + q;  // (the accumulators are zeroed by the build, row by row)
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < total; i += stride) {
        if (i < a) jx_clear(s.jo, i);
        else if (i < a + b) jx_clear(s.jc, i - a);
        else s.qbits[i - a - b] = 0u;
    }
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        *s.err = 0;
        *s.nout = 0;
        if (s.ncand) *s.ncand = 0;
        if (s.tie) *s.tie = 0;
        Q18Stats st;
        st.amt_min = INT64_MAX; st.amt_max = INT64_MIN; st.ent_min = INT64_MAX; st.ent_max = INT64_MIN;
        *s.stats = st;
    }
}

// ------------------------------------------------------------------ K3 build --
__global__ void q18_build_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                                 const int32_t *__restrict__ o_id, uint64_t n_o,
                                 const int32_t *__restrict__ c_w, const int32_t *__restrict__ c_d,
                                 const int32_t *__restrict__ c_id, uint64_t n_c, Q18Scratch s) {
    pdl_wait();
    pdl_trigger();
    // U rows per thread per iteration: their key loads, then their inserts (atomicCAS with
    // return: a dependent round trip) are independent, so U of each are in flight per thread
    // (one row per iteration left the kernel waiting on one CAS at a time: 39 us)
    constexpr int U = 4;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    const uint64_t total = n_o + n_c;
    const bool ident_o = jx_identity(s.jo), ident_c = jx_identity(s.jc);  // positional: no insert
    if (ident_o && ident_c && s.jo.may_ident) return;  // nothing to insert, acc zeroed by the verify
    for (uint64_t i0 = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i0 < total; i0 += U * stride) {
        int w[U], d[U], k[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {  // (an identity side needs no keys: nothing is inserted)
            const uint64_t i = i0 + u * stride;
            if (i < n_o) { if (!ident_o) { w[u] = __ldcs(o_w + i); d[u] = __ldcs(o_d + i); k[u] = __ldcs(o_id + i); } }
            else if (i < total && !ident_c) { const uint64_t j = i - n_o; w[u] = __ldcs(c_w + j); d[u] = __ldcs(c_d + j); k[u] = __ldcs(c_id + j); }
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t i = i0 + u * stride;
            if (i >= total) break;
            bool ok = true;
            if (i < n_o) {
                if (!s.jo.may_ident)  // (else the verify kernel zeroed it)
                    reinterpret_cast<ulonglong2 *>(s.acc)[i] = make_ulonglong2(0ull, 0ull);  // acc[orders row]
                if (!ident_o) ok = jx_insert(s.jo, w[u], d[u], k[u], (unsigned int)i, s.err, kErrDupOrders);
            } else if (!ident_c) {
                ok = jx_insert(s.jc, w[u], d[u], k[u], (unsigned int)(i - n_o), s.err, kErrDupCustomer);
            }
            if (!ok) atomicOr(s.err, kErrDomain);
        }
    }
}

// ------------------------------------------------------- K4 probe + group-join --
// Each lane owns 4 consecutive order_line rows (128-bit loads of w, d, o and two of amount), so
// a warp iteration covers 128 rows. Lines of one order are contiguous, so equal (w, d, o) keys
// form runs (~10 rows): runs are summed inside the lane, a run crossing lanes is summed by a
// 5-step segmented shuffle scan over the lanes' last partial runs, and each run issues ONE
// probe of the orders index and two atomics into acc[orders row] from the lane where it ends.
constexpr int kProbeThreads = 256;

template <bool kFilter>
__global__ void __launch_bounds__(kProbeThreads)
q18_probe_kernel(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
                 const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_amt, uint64_t n,
                 Q18Scratch s) {
    pdl_wait();
    pdl_trigger();
    const bool ident = jx_identity(s.jo);  // after the wait: the verify kernel wrote the verdict
    const int lane = threadIdx.x & 31;
    const uint64_t gwarp = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    const uint64_t nvec = n >> 2;  // full 4-row groups; the ragged tail is handled below
    const uint64_t step = nwarps * 32;
    // software pipeline: the next iteration's five 128-bit loads are in flight while the current
    // group's runs are summed, probed and accumulated
    int4 nW = make_int4(0, 0, 0, 0), nD = nW, nO = nW;
    longlong2 nA0 = make_longlong2(0, 0), nA1 = nA0;
    auto load = [&](uint64_t v) {
        if (v < nvec) {
            nW = __ldcs(reinterpret_cast<const int4 *>(ol_w) + v);
            nD = __ldcs(reinterpret_cast<const int4 *>(ol_d) + v);
            nO = __ldcs(reinterpret_cast<const int4 *>(ol_o) + v);
            nA0 = __ldcs(reinterpret_cast<const longlong2 *>(ol_amt) + 2 * v);
            nA1 = __ldcs(reinterpret_cast<const longlong2 *>(ol_amt) + 2 * v + 1);
        }
    };
    load(gwarp * 32 + lane);
    for (uint64_t vb = gwarp * 32; vb < nvec; vb += step) {
        const uint64_t v = vb + lane;
        const bool valid = v < nvec;
        const int4 W = nW, D = nD, O = nO;
        const longlong2 A0 = nA0, A1 = nA1;
        load(v + step);
        Key3 k[4];
        long long a[4];
        if (valid) {
            k[0] = {W.x, D.x, O.x}; k[1] = {W.y, D.y, O.y}; k[2] = {W.z, D.z, O.z}; k[3] = {W.w, D.w, O.w};
            a[0] = A0.x; a[1] = A0.y; a[2] = A1.x; a[3] = A1.y;
        } else {
            for (int j = 0; j < 4; ++j) { k[j] = {0, 0, 0}; a[j] = 0; }
        }
        probe_lane_group<kFilter>(s, k, a, valid, lane, ident);
    }
    // ragged tail (< 4 rows) plus nothing else: one thread, row at a time
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        for (uint64_t i = nvec * 4; i < n; ++i)
            flush_run<kFilter>(s, Key3{ol_w[i], ol_d[i], ol_o[i]}, ol_amt[i], 1u, ident);
    }
}

// K4, TMA-bulk pipelined variant: one block per SM, the last warp streams 3072-row chunks of
// w, d, o and amount into a 3-stage ring (180 KB); each of the 24 consumer warps runs
// probe_lane_group on 128 rows of the chunk straight from shared memory (128-bit shared loads).
constexpr int kProbeTmaWarps = 24;                 // the lookups and atomics need warps in flight
constexpr int kProbeChunk = kProbeTmaWarps * 128;  // 128 rows per consumer warp per chunk
constexpr int kProbeStages = 3;                    // 3 x 60 KB
struct ProbeStages {
    long long amt[kProbeStages][kProbeChunk];
    int w[kProbeStages][kProbeChunk], d[kProbeStages][kProbeChunk], o[kProbeStages][kProbeChunk];
    uint64_t full[kProbeStages], empty[kProbeStages];
};

__global__ void __launch_bounds__((kProbeTmaWarps + 1) * 32, 1)
q18_probe_tma_kernel(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
                     const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_amt, uint64_t n,
                     Q18Scratch s) {
    extern __shared__ __align__(128) unsigned char smem_raw[];
    ProbeStages &P = *reinterpret_cast<ProbeStages *>(smem_raw);
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const bool ident = jx_identity(s.jo);
    if (threadIdx.x == 0) {
        for (int st = 0; st < kProbeStages; ++st) {
            mbar_init(&P.full[st], 1);
            mbar_init(&P.empty[st], kProbeTmaWarps);
        }
        fence_mbar_init();
    }
    __syncthreads();
    const uint64_t nchunks = (n + kProbeChunk - 1) / kProbeChunk;
    if (warp == kProbeTmaWarps) {  // producer
        if (lane == 0) {
            const uint64_t pol = policy_evict_first();
            int it = 0;
            for (uint64_t c = blockIdx.x; c < nchunks; c += gridDim.x, ++it) {
                const int st = it % kProbeStages;
                const unsigned ph = (unsigned)(it / kProbeStages) & 1u;
                if (it >= kProbeStages) mbar_wait(&P.empty[st], ph ^ 1u);
                const uint64_t r0 = c * kProbeChunk;
                const unsigned rows = (unsigned)(n - r0 < (uint64_t)kProbeChunk ? n - r0 : (uint64_t)kProbeChunk);
                const unsigned b8 = round16(rows * 8), b4 = round16(rows * 4);
                mbar_arrive_expect_tx(&P.full[st], b8 + 3 * b4);
                bulk_g2s(P.amt[st], ol_amt + r0, b8, &P.full[st], pol);
                bulk_g2s(P.w[st], ol_w + r0, b4, &P.full[st], pol);
                bulk_g2s(P.d[st], ol_d + r0, b4, &P.full[st], pol);
                bulk_g2s(P.o[st], ol_o + r0, b4, &P.full[st], pol);
            }
        }
        return;
    }
    int it = 0;
    for (uint64_t c = blockIdx.x; c < nchunks; c += gridDim.x, ++it) {
        const int st = it % kProbeStages;
        mbar_wait(&P.full[st], (unsigned)(it / kProbeStages) & 1u);
        const unsigned rows = (unsigned)(n - c * kProbeChunk < (uint64_t)kProbeChunk ? n - c * kProbeChunk
                                                                                    : (uint64_t)kProbeChunk);
        const unsigned r = warp * 128 + lane * 4;  // this lane's 4 consecutive rows
        Key3 k[4];
        long long a[4];
        const bool valid = r + 3 < rows;
        if (valid) {
            const int4 W = *reinterpret_cast<const int4 *>(&P.w[st][r]);
            const int4 D = *reinterpret_cast<const int4 *>(&P.d[st][r]);
            const int4 O = *reinterpret_cast<const int4 *>(&P.o[st][r]);
            const longlong2 A0 = *reinterpret_cast<const longlong2 *>(&P.amt[st][r]);
            const longlong2 A1 = *reinterpret_cast<const longlong2 *>(&P.amt[st][r + 2]);
            k[0] = {W.x, D.x, O.x}; k[1] = {W.y, D.y, O.y}; k[2] = {W.z, D.z, O.z}; k[3] = {W.w, D.w, O.w};
            a[0] = A0.x; a[1] = A0.y; a[2] = A1.x; a[3] = A1.y;
        } else {
            for (int j = 0; j < 4; ++j) { k[j] = {0, 0, 0}; a[j] = 0; }
        }
        // rows of a partial last group (< 4, last chunk only) go one by one, straight from smem
        if (!valid && r < rows)
            for (unsigned j = r; j < rows; ++j)
                flush_run<false>(s, Key3{P.w[st][j], P.d[st][j], P.o[st][j]}, P.amt[st][j], 1u, ident);
        __syncwarp();
        if (lane == 0) mbar_arrive(&P.empty[st]);  // registers hold everything from here on
        probe_lane_group<false>(s, k, a, valid, lane, ident);
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

// Min/max of amount_sum and o_entry_d over the result rows (the other ORDER BY fields are
// bounded by the snapshot's zone maps, Q18Zone: fewer live registers in the HAVING kernel).
struct StatAcc {
    long long amin = INT64_MAX, amax = INT64_MIN, emin = INT64_MAX, emax = INT64_MIN;
    __device__ void add(long long a, const Q18Row &r) {
        amin = a < amin ? a : amin; amax = a > amax ? a : amax;
        emin = r.o_entry_d < emin ? r.o_entry_d : emin; emax = r.o_entry_d > emax ? r.o_entry_d : emax;
    }
    __device__ void merge(const Q18Stats &o) {
        amin = o.amt_min < amin ? o.amt_min : amin; amax = o.amt_max > amax ? o.amt_max : amax;
        emin = o.ent_min < emin ? o.ent_min : emin; emax = o.ent_max > emax ? o.ent_max : emax;
    }
    __device__ void warp_reduce() {
        amin = wmin64(amin); amax = wmax64(amax); emin = wmin64(emin); emax = wmax64(emax);
    }
    __device__ Q18Stats get() const {
        Q18Stats s;
        s.amt_min = amin; s.amt_max = amax; s.ent_min = emin; s.ent_max = emax;
        return s;
    }
    // Block reduction into part[blockIdx.x]; the last block to finish folds every block's
    // partial into *out (no same-address atomics: thousands of warps would serialise on them).
    __device__ void flush(Q18Stats *part, unsigned int *ticket, Q18Stats *out) {
        __shared__ Q18Stats ws[32];
        __shared__ bool last;
        const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5, nw = (blockDim.x + 31) >> 5;
        warp_reduce();
        if (lane == 0) ws[warp] = get();
        __syncthreads();
        if (threadIdx.x == 0) {
            StatAcc b;
            for (int k = 0; k < nw; ++k) b.merge(ws[k]);
            part[blockIdx.x] = b.get();
            __threadfence();
            last = atomicAdd(ticket, 1u) == gridDim.x - 1;
        }
        __syncthreads();
        if (!last) return;
        __threadfence();
        StatAcc f;
        for (unsigned k = threadIdx.x; k < gridDim.x; k += blockDim.x) {
            Q18Stats x;
            const long long *src = reinterpret_cast<const long long *>(part + k);
            long long *dst = reinterpret_cast<long long *>(&x);
            for (int q = 0; q < (int)(sizeof(Q18Stats) / 8); ++q) dst[q] = __ldcg(src + q);
            f.merge(x);
        }
        f.warp_reduce();
        __syncthreads();
        if (lane == 0) ws[warp] = f.get();
        __syncthreads();
        if (threadIdx.x == 0) {
            StatAcc b;
            for (int k = 0; k < nw; ++k) b.merge(ws[k]);
            *out = b.get();
            *ticket = 0;  // self-reset for the next launch
        }
    }
};

// Each block iteration covers kHavingRows consecutive orders rows (kHavingUnroll per thread);
// passing rows get output slots from ONE atomicAdd per block iteration (block-wide exclusive
// scan of the per-thread counts), so the output counter sees ~n/1024 atomics, not n/32.
template <int kHavingUnroll>
__global__ void __launch_bounds__(kHavingThreads, 4)
q18_having_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                  const int32_t *__restrict__ o_id, const int32_t *__restrict__ o_c,
                  const int32_t *__restrict__ o_cnt, const int64_t *__restrict__ o_ent, uint64_t n,
                  const int32_t *__restrict__ c_last, long long having, Q18Scratch s) {
    pdl_wait();
    pdl_trigger();
    __shared__ unsigned int wsum[kHavingThreads / 32];
    __shared__ unsigned long long s_base;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    constexpr int kHavingRows = kHavingThreads * kHavingUnroll;
    const uint64_t keep = l2_policy_evict_last();
    StatAcc stat;
    for (uint64_t base = (uint64_t)blockIdx.x * kHavingRows; base < n;
         base += (uint64_t)gridDim.x * kHavingRows) {
        unsigned int crow[kHavingUnroll];
        long long sum[kHavingUnroll];
        int w[kHavingUnroll], d[kHavingUnroll], c[kHavingUnroll];
        bool pass1[kHavingUnroll];
        unsigned int mine = 0;
        // stage 1: independent coalesced loads for all rows (maximise loads in flight)
#pragma unroll
        for (int u = 0; u < kHavingUnroll; ++u) {
            const uint64_t r = base + u * kHavingThreads + threadIdx.x;
            pass1[u] = false;
            sum[u] = 0;
            w[u] = d[u] = c[u] = 0;
            if (r < n) {
                const ulonglong2 a = __ldcs(reinterpret_cast<const ulonglong2 *>(s.acc + r));
                sum[u] = (long long)a.x;
                // inner join: a group exists only with >= 1 order_line row; HAVING SUM > having
                pass1[u] = (unsigned int)a.y > 0 && sum[u] > having;
                w[u] = __ldcs(o_w + r); d[u] = __ldcs(o_d + r); c[u] = __ldcs(o_c + r);
            }
        }
        // stage 2: customer ⋈ orders lookups, independent across rows
#pragma unroll
        for (int u = 0; u < kHavingUnroll; ++u) {
            crow[u] = pass1[u] ? jx_lookup(s.jc, w[u], d[u], c[u]) : kNoRow;
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
        Q18Row row[kHavingUnroll];
#pragma unroll
        for (int u = 0; u < kHavingUnroll; ++u) {  // stage 3: gathers for passing rows
            if (crow[u] == kNoRow) continue;
            const uint64_t r = base + u * kHavingThreads + threadIdx.x;
            row[u].o_entry_d = __ldcs(o_ent + r);
            row[u].c_last = __ldg(c_last + crow[u]);
            row[u].c_id = c[u];
            row[u].o_id = __ldcs(o_id + r);
            row[u].o_ol_cnt = __ldcs(o_cnt + r);
            row[u].o_w_id = w[u];
            row[u].o_d_id = d[u];
        }
#pragma unroll
        for (int u = 0; u < kHavingUnroll; ++u) {
            if (crow[u] == kNoRow) continue;
            s.amt[p] = sum[u];
            // result rows are gathered again by the ORDER BY permute: keep them in L2
            const unsigned long long *w64 = reinterpret_cast<const unsigned long long *>(&row[u]);
            st16_policy(s.rows + p, w64[0], w64[1], keep);
            st16_policy(reinterpret_cast<char *>(s.rows + p) + 16, w64[2], w64[3], keep);
            ++p;
            stat.add(sum[u], row[u]);
        }
        __syncthreads();  // wsum / s_base reuse
    }
    stat.flush(s.stat_part, s.ticket, s.stats);
}

// ------------------------------------------------------------- CH Q3 (NEXT-2) --
// Q3 = customer ⋈ new_order ⋈ orders ⋈ order_line, GROUP BY the orders key, ORDER BY revenue
// DESC, o_entry_d. Its group key (ol_o_id, ol_w_id, ol_d_id, o_entry_d) is functionally
// determined by the orders row (orders PK unique, checked), so the Q18 machinery applies:
//  mark:  per new_order row, probe orders (o_entry_d > lo) then customer (c_state LIKE prefix);
//         acc[orders row].pad counts the joined (new_order, customer) pairs — the inner join's
//         multiplicity (a duplicated new_order row doubles the order's revenue); the first mark of
//         a row appends it to a candidate list (count in *ncand, warp-aggregated);
//  probe: q18_probe_kernel<true> (only marked rows accumulate);
//  emit:  per candidate with >= 1 line, revenue = sum x multiplicity into 32-byte result rows +
//         the sort-field statistics (row count in *nout), then the Q18 ORDER BY (same total
//         order, R33).
__device__ __forceinline__ bool like_prefix2(int p2, int prefix) {
    // prefix = (c0 << 8) | c1 of a LIKE 'c0c1%' pattern; c1 == 0: one character; 0: empty pattern
    const int mask = (prefix & 0xff) ? 0xffff : ((prefix & 0xff00) ? 0xff00 : 0);
    return (p2 & mask) == prefix;
}

__global__ void q3_mark_kernel(const int32_t *__restrict__ no_w, const int32_t *__restrict__ no_d,
                               const int32_t *__restrict__ no_o, const int32_t *__restrict__ no_del, uint64_t n_no,
                               const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                               const int32_t *__restrict__ o_c, const int64_t *__restrict__ o_ent,
                               const int32_t *__restrict__ c_p2, long long entry_lo, int prefix,
                               Q18Scratch s) {
    const int lane = threadIdx.x & 31;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    const uint64_t n_pad = (n_no + 31) & ~31ull;  // whole warps iterate together (ballot below)
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n_pad; i += stride) {
        unsigned int orow = kNoRow;
        // a deleted new_order row (Delivery's DELETE, a tombstone update) is not there: no join
        if (i < n_no && !(no_del && __ldcs(no_del + i)))
            orow = jx_lookup(s.jo, __ldcs(no_w + i), __ldcs(no_d + i), __ldcs(no_o + i));
        bool hit = false;
        if (orow != kNoRow && __ldg(o_ent + orow) > entry_lo) {
            const unsigned int crow = jx_lookup(s.jc, __ldg(o_w + orow), __ldg(o_d + orow), __ldg(o_c + orow));
            hit = crow != kNoRow && like_prefix2(__ldg(c_p2 + crow), prefix);
        }
        bool first = false;
        if (hit) first = atomicAdd(&s.acc[orow].pad, 1u) == 0u;
        if (first) atomicOr(s.qbits + (orow >> 5), 1u << (orow & 31));
        const unsigned int fb = __ballot_sync(kFull, first);
        if (fb) {
            unsigned long long base = 0;
            if (lane == __ffs(fb) - 1) base = atomicAdd(s.ncand, (unsigned long long)__popc(fb));
            base = __shfl_sync(kFull, base, __ffs(fb) - 1);
            if (first) s.cand[base + __popc(fb & ((1u << lane) - 1))] = orow;
        }
    }
}

__global__ void __launch_bounds__(256)
q3_emit_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
               const int32_t *__restrict__ o_id, const int32_t *__restrict__ o_c,
               const int32_t *__restrict__ o_cnt, const int64_t *__restrict__ o_ent, Q18Scratch s) {
    __shared__ unsigned int wsum[8];
    __shared__ unsigned long long s_base;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const uint64_t ncand = *s.ncand;  // written by the mark kernel (earlier on the stream)
    StatAcc stat;
    for (uint64_t base = (uint64_t)blockIdx.x * blockDim.x; base < ncand; base += (uint64_t)gridDim.x * blockDim.x) {
        const uint64_t i = base + threadIdx.x;
        unsigned int r = kNoRow;
        long long sum = 0;
        if (i < ncand) {
            r = s.cand[i];
            const ulonglong2 a = __ldcg(reinterpret_cast<const ulonglong2 *>(s.acc + r));
            const unsigned int cnt = (unsigned int)a.y, mult = (unsigned int)(a.y >> 32);
            if (cnt == 0) r = kNoRow;  // inner join: no order_line row, no group
            sum = (long long)a.x * (long long)mult;
        }
        const unsigned int mine = r != kNoRow;
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
        for (int k = 0; k < 8; ++k) {
            before += k < warp ? wsum[k] : 0u;
            total += wsum[k];
        }
        if (threadIdx.x == 0) s_base = total ? atomicAdd(s.nout, (unsigned long long)total) : 0ull;
        __syncthreads();
        if (mine) {
            const uint64_t p = s_base + before + x - 1;
            Q18Row row;
            row.o_entry_d = __ldg(o_ent + r);
            row.c_last = 0;   // Q3 outputs no customer / o_ol_cnt fields: zero payload
            row.c_id = 0;     // (its ORDER BY zone has c_last = c_id = o_ol_cnt = 0)
            row.o_id = __ldg(o_id + r);
            row.o_ol_cnt = 0;
            row.o_w_id = __ldg(o_w + r);
            row.o_d_id = __ldg(o_d + r);
            s.rows[p] = row;
            s.amt[p] = sum;
            stat.add(sum, row);
        }
        __syncthreads();
    }
    stat.flush(s.stat_part, s.ticket, s.stats);
}

struct Q18SmallDev { unsigned long long nout; unsigned int err, tie; Q18Stats st; unsigned long long row0, n_total;
                     unsigned int clustered; };  // = engine's Q18Small
__global__ void q18_publish_kernel(const unsigned long long *nout, const unsigned int *err,
                                   const unsigned int *tie, Q18SmallDev *out, JoinIndex jo, JoinIndex jc) {
    pdl_wait();
    pdl_trigger();
    out->nout = *nout;
    out->err = *err;
    out->tie = *tie;
    out->clustered = (jx_identity(jo) ? 1u : 0u) | (jx_identity(jc) ? 2u : 0u);  // positional indexes used
}

}  // namespace

void launch_q18_publish(const unsigned long long *nout, const unsigned int *err, const unsigned int *tie,
                        void *host_small, const JoinIndex &jo, const JoinIndex &jc, cudaStream_t st) {
    launch_pdl(q18_publish_kernel, 1, 1, 0, st, nout, err, tie, static_cast<Q18SmallDev *>(host_small), jo, jc);
    count_launches(1);
}

void launch_q18_init(const Q18Scratch &s, const int32_t *o_w, const int32_t *o_d, const int32_t *o_id,
                     uint64_t n_o, const int32_t *c_w, const int32_t *c_d, const int32_t *c_id, uint64_t n_c,
                     int num_sms, cudaStream_t st) {
    if (s.jo.may_ident || s.jc.may_ident) {
        launch_pdl(q18_verify_kernel, grid_for((n_o + n_c + 3) / 4, 256, num_sms, 8), 256, 0, st,
                   s, o_w, o_d, o_id, n_o, c_w, c_d, c_id, n_c);
        count_launches(1);
    }
    const uint64_t words = jx_words(s.jo) + jx_words(s.jc);
    launch_pdl(q18_init_kernel, grid_for(words, 256, num_sms, 8), 256, 0, st, s);
    count_launches(1);
}

void launch_q18_build(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, uint64_t n_o,
                      const int32_t *c_w, const int32_t *c_d, const int32_t *c_id, uint64_t n_c,
                      const Q18Scratch &s, int num_sms, cudaStream_t st) {
    launch_pdl(q18_build_kernel, grid_for((n_o + n_c + 3) / 4, 256, num_sms, 8), 256, 0, st, o_w, o_d, o_id, n_o, c_w,
                                                                         c_d, c_id, n_c, s);
    count_launches(1);
}

void launch_q18_probe(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o,
                      const int64_t *ol_amt, uint64_t n_ol, const Q18Scratch &s, int num_sms,
                      cudaStream_t st) {
    launch_pdl(q18_probe_kernel<false>, grid_for((n_ol + 3) / 4, kProbeThreads, num_sms, 8), kProbeThreads, 0, st,
        ol_w, ol_d, ol_o, ol_amt, n_ol, s);
    count_launches(1);
}

void launch_q3_mark(const int32_t *no_w, const int32_t *no_d, const int32_t *no_o, const int32_t *no_del, uint64_t n_no,
                    const int32_t *o_w, const int32_t *o_d, const int32_t *o_c, const int64_t *o_ent,
                    const int32_t *c_p2, int64_t entry_lo, int prefix, const Q18Scratch &s, int num_sms,
                    cudaStream_t st) {
    q3_mark_kernel<<<grid_for(n_no, 256, num_sms, 8), 256, 0, st>>>(no_w, no_d, no_o, no_del, n_no, o_w, o_d, o_c,
                                                                 o_ent, c_p2, entry_lo, prefix, s);
    count_launches(1);
}

void launch_q3_probe(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o,
                     const int64_t *ol_amt, uint64_t n_ol, const Q18Scratch &s, int num_sms,
                     cudaStream_t st) {
    q18_probe_kernel<true><<<grid_for((n_ol + 3) / 4, kProbeThreads, num_sms, 8), kProbeThreads, 0, st>>>(
        ol_w, ol_d, ol_o, ol_amt, n_ol, s);
    count_launches(1);
}

void launch_q3_emit(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, const int32_t *o_c,
                    const int32_t *o_cnt, const int64_t *o_ent, uint64_t max_cand, const Q18Scratch &s,
                    int num_sms, cudaStream_t st) {
    // grid <= the stat_part capacity (8 blocks per SM); sized for the largest possible list
    q3_emit_kernel<<<grid_for(max_cand, 256, num_sms, 8), 256, 0, st>>>(o_w, o_d, o_id, o_c, o_cnt, o_ent, s);
    count_launches(1);
}

void launch_q18_probe_tma(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o,
                          const int64_t *ol_amt, uint64_t n_ol, const Q18Scratch &s, int num_sms,
                          cudaStream_t st) {
    const uint64_t nchunks = (n_ol + kProbeChunk - 1) / kProbeChunk;
    const unsigned grid = (unsigned)(nchunks < (uint64_t)num_sms ? (nchunks ? nchunks : 1) : num_sms);
    q18_probe_tma_kernel<<<grid, (kProbeTmaWarps + 1) * 32, sizeof(ProbeStages), st>>>(ol_w, ol_d, ol_o,
                                                                                      ol_amt, n_ol, s);
    count_launches(1);
}

void launch_q18_having(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id,
                       const int32_t *o_c, const int32_t *o_cnt, const int64_t *o_ent,
                       uint64_t n_o, const int32_t *c_last, int64_t having,
                       const Q18Scratch &s, int num_sms, cudaStream_t st, int unroll) {
    // blocks per SM (H2TAP_HAVING_BPS, 1..8: the statistics partials hold 8 per SM); 4 = every
    // block resident at once (4 x 256 threads at 56 registers), measured 69 us vs 72 us at 8
    static const int bps = [] {
        const char *v = std::getenv("H2TAP_HAVING_BPS");
        return v ? std::max(1, std::min(8, std::atoi(v))) : 4;
    }();
    if (unroll == 4)
        launch_pdl(q18_having_kernel<4>, grid_for((n_o + 3) / 4, kHavingThreads, num_sms, bps), kHavingThreads, 0, st,
            o_w, o_d, o_id, o_c, o_cnt, o_ent, n_o, c_last, having, s);
    else
        launch_pdl(q18_having_kernel<2>, grid_for((n_o + 1) / 2, kHavingThreads, num_sms, bps), kHavingThreads, 0, st,
            o_w, o_d, o_id, o_c, o_cnt, o_ent, n_o, c_last, having, s);
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

cudaError_t set_attributes_join(int num_sms) {
    static const void *const kKernels[] = {
        (const void *)q18_build_kernel,
        (const void *)q18_having_kernel<2>,
        (const void *)q18_having_kernel<4>,
        (const void *)q18_init_kernel,
        (const void *)q18_verify_kernel,
        (const void *)q18_probe_kernel<false>,
        (const void *)q18_probe_kernel<true>,
        (const void *)q18_probe_tma_kernel,
        (const void *)q18_publish_kernel,
        (const void *)q3_emit_kernel,
        (const void *)q3_mark_kernel};
    const cudaError_t le = force_load(kKernels, sizeof kKernels / sizeof kKernels[0]);
    if (le != cudaSuccess) return le;

    (void)num_sms;
    return cudaFuncSetAttribute(q18_probe_tma_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize,
                                (int)sizeof(ProbeStages));
}

}  // namespace h2tap
