// sort_kernels.cu — a8 finalize for CH Q18: ORDER BY amount_sum DESC, o_entry_d ASC, then the
// (o_w_id, o_d_id, o_id) tie-break (R11), as a stable LSD radix sort of a permutation.
//
// Each sort field is mapped to an unsigned key whose bit width is taken from the data's
// min/max (computed by the HAVING kernel), so only the passes the data needs are run:
//   field 0 (least significant): dense rank of (w, d, o)  asc
//   field 1:                      o_entry_d - min          asc
//   field 2 (most significant):  max - amount_sum          (= DESC)
// One pass = histogram (per 8192-element block tile) -> exclusive scan -> stable scatter.
// Stability inside a tile comes from processing each warp's sub-tile in order with
// __match_any_sync ranks, and tiles in order via the digit-major count layout.
#include <cstdint>
#include <cuda_runtime.h>

#include "kernels.cuh"

namespace h2tap {
namespace {

constexpr unsigned kFull = 0xffffffffu;
constexpr int kThreads = 256;
constexpr int kWarps = kThreads / 32;
constexpr int kItems = 32;                       // per lane per block tile
constexpr int kWarpTile = 32 * kItems;           // 1024
constexpr int kBlockTile = kWarps * kWarpTile;   // 8192

__device__ __forceinline__ unsigned int digit_of(const unsigned long long *__restrict__ key,
                                                 const unsigned int *__restrict__ idx,
                                                 uint64_t j, int shift) {
    const unsigned int e = idx ? idx[j] : (unsigned int)j;
    return (unsigned int)(__ldcg(key + e) >> shift) & 0xffu;
}

__global__ void __launch_bounds__(kThreads)
hist_kernel(const unsigned long long *__restrict__ key, const unsigned int *__restrict__ idx,
            uint64_t n, int shift, unsigned int *__restrict__ counts, uint64_t ntiles) {
    __shared__ unsigned int h[256];
    for (int i = threadIdx.x; i < 256; i += kThreads) h[i] = 0;
    __syncthreads();
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const uint64_t base = (uint64_t)blockIdx.x * kBlockTile + (uint64_t)warp * kWarpTile;
    for (int it = 0; it < kItems; ++it) {
        const uint64_t j = base + it * 32 + lane;
        const bool ok = j < n;
        const unsigned int dg = ok ? digit_of(key, idx, j, shift) : 256u + lane;  // unique dummy
        const unsigned int peers = __match_any_sync(kFull, dg);
        if (ok && lane == __ffs(peers) - 1) atomicAdd(&h[dg], (unsigned int)__popc(peers));
    }
    __syncthreads();
    for (int d = threadIdx.x; d < 256; d += kThreads) counts[(uint64_t)d * ntiles + blockIdx.x] = h[d];
}

// Exclusive scan of `len` counts in place, one block of 1024 threads, coalesced rounds.
__global__ void __launch_bounds__(1024) scan_kernel(unsigned int *__restrict__ c, uint64_t len) {
    __shared__ unsigned int wsum[32];
    __shared__ unsigned int carry_s;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    unsigned int carry = 0;
    for (uint64_t r0 = 0; r0 < len; r0 += 4096) {
        unsigned int v[4];
        const uint64_t b = r0 + 4 * (uint64_t)threadIdx.x;
#pragma unroll
        for (int k = 0; k < 4; ++k) v[k] = b + k < len ? c[b + k] : 0u;
        const unsigned int s = v[0] + v[1] + v[2] + v[3];
        unsigned int x = s;  // inclusive warp scan
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const unsigned int t = __shfl_up_sync(kFull, x, o);
            if (lane >= o) x += t;
        }
        if (lane == 31) wsum[warp] = x;
        __syncthreads();
        if (warp == 0) {
            unsigned int y = wsum[lane];
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                const unsigned int t = __shfl_up_sync(kFull, y, o);
                if (lane >= o) y += t;
            }
            wsum[lane] = y;  // inclusive over warps
            if (lane == 31) carry_s = y;
        }
        __syncthreads();
        unsigned int ex = carry + (warp ? wsum[warp - 1] : 0u) + x - s;
#pragma unroll
        for (int k = 0; k < 4; ++k) {
            if (b + k < len) c[b + k] = ex;
            ex += v[k];
        }
        carry += carry_s;
        __syncthreads();
    }
}

__global__ void __launch_bounds__(kThreads)
scatter_kernel(const unsigned long long *__restrict__ key, const unsigned int *__restrict__ idx_in,
               unsigned int *__restrict__ idx_out, uint64_t n, int shift,
               const unsigned int *__restrict__ offsets, uint64_t ntiles) {
    __shared__ unsigned int wcount[kWarps][256];  // per-warp digit counts -> running offsets
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    for (int i = threadIdx.x; i < kWarps * 256; i += kThreads) (&wcount[0][0])[i] = 0;
    __syncthreads();
    const uint64_t base = (uint64_t)blockIdx.x * kBlockTile + (uint64_t)warp * kWarpTile;
    for (int it = 0; it < kItems; ++it) {  // pass 1: per-warp histogram
        const uint64_t j = base + it * 32 + lane;
        const bool ok = j < n;
        const unsigned int dg = ok ? digit_of(key, idx_in, j, shift) : 256u + lane;
        const unsigned int peers = __match_any_sync(kFull, dg);
        if (ok && lane == __ffs(peers) - 1) wcount[warp][dg] += __popc(peers);
    }
    __syncthreads();
    // running offset of warp w for digit d = tile offset[d] + counts of warps < w
    for (int d = threadIdx.x; d < 256; d += kThreads) {
        unsigned int run = offsets[(uint64_t)d * ntiles + blockIdx.x];
        for (int w = 0; w < kWarps; ++w) {
            const unsigned int c = wcount[w][d];
            wcount[w][d] = run;
            run += c;
        }
    }
    __syncthreads();
    const unsigned lt = (1u << lane) - 1u;
    for (int it = 0; it < kItems; ++it) {  // pass 2: stable scatter in (iteration, lane) order
        const uint64_t j = base + it * 32 + lane;
        const bool ok = j < n;
        const unsigned int dg = ok ? digit_of(key, idx_in, j, shift) : 256u + lane;
        const unsigned int peers = __match_any_sync(kFull, dg);
        if (ok) {
            const unsigned int pos = wcount[warp][dg] + __popc(peers & lt);
            idx_out[pos] = idx_in ? idx_in[j] : (unsigned int)j;
        }
        __syncwarp();
        if (ok && lane == __ffs(peers) - 1) wcount[warp][dg] += __popc(peers);
        __syncwarp();
    }
}

__global__ void sort_keys_kernel(Q18Cols c, uint64_t n, Q18SortSpec sp, SortScratch s) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        const unsigned long long w = (unsigned)(c.o_w_id[i] - sp.w_min);
        const unsigned long long d = (unsigned)(c.o_d_id[i] - sp.d_min);
        const unsigned long long o = (unsigned)(c.o_id[i] - sp.o_min);
        s.key[0][i] = (w * (unsigned long long)sp.nd + d) * (unsigned long long)sp.no + o;
        s.key[1][i] = (unsigned long long)c.o_entry_d[i] - (unsigned long long)sp.ent_min;
        s.key[2][i] = (unsigned long long)sp.amt_max - (unsigned long long)c.amount_sum[i];
    }
}

__global__ void permute_kernel(Q18Cols src, const unsigned int *__restrict__ perm, uint64_t n,
                               Q18Cols dst) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t j = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; j < n; j += stride) {
        const unsigned int i = perm ? perm[j] : (unsigned int)j;
        dst.c_last[j] = src.c_last[i];
        dst.c_id[j] = src.c_id[i];
        dst.o_id[j] = src.o_id[i];
        dst.o_entry_d[j] = src.o_entry_d[i];
        dst.o_ol_cnt[j] = src.o_ol_cnt[i];
        dst.amount_sum[j] = src.amount_sum[i];
        dst.o_w_id[j] = src.o_w_id[i];
        dst.o_d_id[j] = src.o_d_id[i];
    }
}

unsigned grid_cap(uint64_t work, int threads, int num_sms, int per_sm) {
    uint64_t want = (work + threads - 1) / threads;
    uint64_t cap = (uint64_t)num_sms * per_sm;
    if (want > cap) want = cap;
    return want ? (unsigned)want : 1u;
}

}  // namespace

void launch_q18_sort_keys(const Q18Cols &cols, uint64_t n, const Q18SortSpec &spec,
                          const SortScratch &s, int num_sms, cudaStream_t st) {
    sort_keys_kernel<<<grid_cap(n, 256, num_sms, 8), 256, 0, st>>>(cols, n, spec, s);
    count_launches(1);
}

unsigned int *radix_sort_fields(uint64_t n, const int bits[3], const SortScratch &s,
                                cudaStream_t st, int num_sms) {
    (void)num_sms;
    const uint64_t ntiles = (n + kBlockTile - 1) / kBlockTile;
    const unsigned int *in = nullptr;  // identity permutation before the first pass
    unsigned int *out = s.idx_a;
    for (int f = 0; f < 3; ++f) {
        for (int shift = 0; shift < bits[f]; shift += 8) {
            hist_kernel<<<(unsigned)ntiles, kThreads, 0, st>>>(s.key[f], in, n, shift, s.counts, ntiles);
            count_launches(1);
            scan_kernel<<<1, 1024, 0, st>>>(s.counts, 256 * ntiles);
            count_launches(1);
            scatter_kernel<<<(unsigned)ntiles, kThreads, 0, st>>>(s.key[f], in, out, n, shift, s.counts,
                                                                ntiles);
            count_launches(1);
            in = out;
            out = (out == s.idx_a) ? s.idx_b : s.idx_a;
        }
    }
    // nullptr = zero passes were needed (n <= 1 or all keys equal): identity permutation
    return const_cast<unsigned int *>(in);
}

void launch_q18_permute(const Q18Cols &src, const unsigned int *perm, uint64_t n,
                        const Q18Cols &dst, int num_sms, cudaStream_t st) {
    permute_kernel<<<grid_cap(n, 256, num_sms, 8), 256, 0, st>>>(src, perm, n, dst);
    count_launches(1);
}

}  // namespace h2tap
