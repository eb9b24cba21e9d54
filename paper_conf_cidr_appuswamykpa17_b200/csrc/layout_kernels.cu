// layout_kernels.cu — NEXT-3 / NEXT-4: SELECT SUM(col_1 + ... + col_N) over a table of int32
// attributes stored as DSM, PAX or NSM, read from HBM or, zero-copy, from pinned host memory.
//
// Paper: PAPER.md §5.3 "Data sharing with PAX" (L965-1077): a 16-attribute int table in DSM, PAX
// (4 KB pages of 16 minipages x 64 values) and NSM; query template SUM(col1 + ... + colN) for
// N = 1, 2, 4, 8, 16; Fig. 10 = host-resident (UVA) 16 GB, Fig. 11 = GPU-resident 1 GB, N = 2.
// The paper's finding: coalescing decides GPU scan cost; NSM wastes transfers (L979-990), PAX
// and DSM coalesce (L991-1000).
//
// B200 design: each layout is a stream of 16-byte vectors, and the sum is order-independent, so
// no kernel reconstructs records: DSM streams each selected column; PAX streams only the selected
// 256-byte minipages of every page (whole sectors, unselected minipages never touched); NSM
// streams the record array and skips the vectors holding no selected attribute (what remains is
// the sector waste the paper measures). int64 accumulation in registers, warp shuffle, one
// 64-bit atomic per block. The same kernels read HBM or mapped pinned host memory (UVA, the
// paper's Caldera mechanism, L484-490, L568-572): only the pointer differs.
#include <cstdint>
#include <cstdlib>
#include <cuda_runtime.h>

#include "kernels.cuh"

namespace h2tap {
namespace {

constexpr unsigned kFull = 0xffffffffu;
constexpr int kThreads = 256;
constexpr int kUnroll = 4;  // independent 16-byte loads in flight per thread per iteration

__device__ __forceinline__ int4 ld_stream(const int4 *p) {
    int4 r;
    asm volatile("ld.global.nc.L1::no_allocate.v4.s32 {%0, %1, %2, %3}, [%4];"
                 : "=r"(r.x), "=r"(r.y), "=r"(r.z), "=r"(r.w) : "l"(p));
    return r;
}

__device__ __forceinline__ void block_add(long long v, unsigned long long *out) {
    __shared__ long long ws[kThreads / 32];
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(kFull, v, o);
    if ((threadIdx.x & 31) == 0) ws[threadIdx.x >> 5] = v;
    __syncthreads();
    if (threadIdx.x == 0) {
        long long s = 0;
        for (int k = 0; k < kThreads / 32; ++k) s += ws[k];
        if (s) atomicAdd(out, (unsigned long long)s);  // two's complement: exact signed sum
    }
}

__device__ __forceinline__ long long lanes_sum(const int4 x, unsigned sel4) {
    return (long long)((sel4 & 1) ? x.x : 0) + ((sel4 & 2) ? x.y : 0) + ((sel4 & 4) ? x.z : 0) +
           ((sel4 & 8) ? x.w : 0);
}

// DSM: column c starts at data + c * stride (int32 elements). blockIdx.y picks the selected
// column; its unaligned head (< 4 values, when c * stride is not a multiple of 4) and ragged tail
// are summed by single lanes, the aligned body as 16-byte vectors, kUnroll loads in flight per
// thread.
__global__ void __launch_bounds__(kThreads)
dsm_sum_kernel(const int32_t *__restrict__ data, uint64_t stride, uint64_t n, LayoutSel sel,
               unsigned long long *out) {
    const int32_t *col = data + (uint64_t)sel.col[blockIdx.y] * stride;
    const uint64_t head = ((16 - (reinterpret_cast<uintptr_t>(col) & 15)) & 15) >> 2;
    const uint64_t h = head < n ? head : n;
    const int4 *body = reinterpret_cast<const int4 *>(col + h);
    const uint64_t nvec = (n - h) >> 2;
    const uint64_t step = (uint64_t)gridDim.x * blockDim.x;
    long long acc = 0;
    for (uint64_t v = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; v < nvec; v += kUnroll * step) {
        int4 x[kUnroll];
#pragma unroll
        for (int u = 0; u < kUnroll; ++u)
            if (v + u * step < nvec) x[u] = ld_stream(body + v + u * step);
#pragma unroll
        for (int u = 0; u < kUnroll; ++u)
            if (v + u * step < nvec) acc += (long long)x[u].x + x[u].y + x[u].z + x[u].w;
    }
    if (blockIdx.x == 0 && threadIdx.x < 8) {  // head rows [0, h) and tail rows [h + 4 nvec, n)
        const uint64_t r = threadIdx.x < 4 ? threadIdx.x : h + 4 * nvec + (threadIdx.x - 4);
        if ((threadIdx.x < 4 && r < h) || (threadIdx.x >= 4 && r < n)) acc += col[r];
    }
    block_add(acc, out);
}

// PAX: page = ncols minipages of mp_rows values (powers of two, mp_rows >= 4). The work is the
// sequence of (page, selected minipage) pairs q = page * N + j; a warp step covers
// mps = 32 / (mp_rows / 4) consecutive pairs (one 16-byte vector per lane; kUnroll steps in
// flight), so only selected minipages are read — whole sectors — and no lane idles for any N.
// (page, j) is carried incrementally (divisions by N only once per thread, none per vector).
__global__ void __launch_bounds__(kThreads)
pax_sum_kernel(const int32_t *__restrict__ data, uint64_t n, int log_ncols, int log_mp, LayoutSel sel,
               unsigned long long *out) {
    const int lane = threadIdx.x & 31;
    const int log_vpm = log_mp - 2;                           // 16-byte vectors per minipage
    const int vpm = 1 << log_vpm;
    const int mps = vpm >= 32 ? 1 : 32 / vpm;                 // pairs per warp step
    const int sub = vpm >= 32 ? 0 : lane >> log_vpm;          // this lane's pair in the step
    const uint64_t pages = (n + (1ull << log_mp) - 1) >> log_mp;
    const uint64_t N = (uint64_t)sel.n;
    const uint64_t gwarp = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    const uint64_t wstep = (uint64_t)mps * kUnroll;           // pairs per warp iteration
    // iteration base q0 = gwarp * wstep as (p0, j0); stride nwarps * wstep as (sp, sj)
    uint64_t p0 = (gwarp * wstep) / N, j0 = (gwarp * wstep) % N;
    const uint64_t S = nwarps * wstep, sp = S / N, sj = S % N;
    uint64_t dp[kUnroll], dj[kUnroll];                        // offsets u * mps + sub as (page, j)
#pragma unroll
    for (int u = 0; u < kUnroll; ++u) {
        const uint64_t off = (uint64_t)u * mps + sub;
        dp[u] = off / N;
        dj[u] = off % N;
    }
    long long acc = 0;
    for (; p0 < pages;) {
        for (int v0 = 0; v0 < vpm; v0 += 32) {                 // minipages wider than a warp
            const int v = vpm >= 32 ? v0 + lane : (lane & (vpm - 1));
            int4 x[kUnroll];
            unsigned sel4[kUnroll];
#pragma unroll
            for (int u = 0; u < kUnroll; ++u) {
                uint64_t p = p0 + dp[u], j = j0 + dj[u];
                if (j >= N) { j -= N; ++p; }
                sel4[u] = 0;
                if (p < pages) {
                    const uint64_t row0 = (p << log_mp) + 4 * (uint64_t)v;
                    sel4[u] = row0 >= n ? 0u : (n - row0 >= 4 ? 0xfu : (1u << (unsigned)(n - row0)) - 1u);
                    const uint64_t off = (((p << log_ncols) + (unsigned)sel.col[j]) << log_mp) + 4 * (uint64_t)v;
                    if (sel4[u]) x[u] = ld_stream(reinterpret_cast<const int4 *>(data + off));
                }
            }
#pragma unroll
            for (int u = 0; u < kUnroll; ++u)
                if (sel4[u]) acc += lanes_sum(x[u], sel4[u]);
        }
        p0 += sp;
        j0 += sj;
        if (j0 >= N) { j0 -= N; ++p0; }
    }
    block_add(acc, out);
}

// PAX with N (selected attributes) a power of two — the paper's N = 1, 2, 4, 8, 16: the selected
// minipages of page p form V = N x vpm consecutive 16-byte vectors of one stream, and a warp
// iteration takes 128 consecutive stream vectors (4 per lane, all loads in flight first). With V
// and 128 both powers of two every lane's (page offset, minipage, vector) decomposition is either
// the same for every iteration (V <= 128) or shifts by a whole number of minipages (V > 128), so
// the loop does no divisions and little address arithmetic (the general kernel above spent its
// issue slots there: 0.6 of the copy peak at N = 16 where the stream is the whole table).
#ifndef PAX_U
#define PAX_U 4
#endif
constexpr int kPaxU = PAX_U;
__global__ void __launch_bounds__(kThreads)
pax_pow2_sum_kernel(const int32_t *__restrict__ data, uint64_t n, int log_ncols, int log_mp, int log_n,
                    LayoutSel sel, unsigned long long *out) {
    __shared__ int cols[kMaxLayoutSel];
    for (int i = threadIdx.x; i < sel.n; i += kThreads) cols[i] = sel.col[i];
    __syncthreads();
    const int lane = threadIdx.x & 31;
    const int log_vpm = log_mp - 2, log_v = log_n + log_vpm;  // vectors per minipage / per page
    const uint64_t pages = (n + (1ull << log_mp) - 1) >> log_mp;
    const uint64_t total = pages << log_v;                     // stream vectors
    const uint64_t gwarp = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    constexpr int kW = 32 * kPaxU;                              // stream vectors per warp iteration
    const unsigned vmask = (1u << log_vpm) - 1u;
    // this lane's k-th vector of an iteration, o = k * 32 + lane: with V = 2^log_v <= kW the
    // iteration starts on a page boundary and o decomposes into a fixed (page offset, minipage
    // column, vector) — precomputed; with V > kW the minipage shifts by a fixed amount per step
    const bool small_v = log_v <= __ffs(kW) - 1;
    unsigned dpage[kPaxU], colv[kPaxU];                         // colv = (column << 16) | vector
#pragma unroll
    for (int u = 0; u < kPaxU; ++u) {
        const unsigned o = (unsigned)u * 32 + lane;
        const unsigned within = small_v ? (o & ((1u << log_v) - 1u)) : o;
        dpage[u] = small_v ? (o >> log_v) : 0u;
        colv[u] = small_v ? (((unsigned)cols[within >> log_vpm] << 16) | (within & vmask)) : 0u;
    }
    long long acc = 0;
    const uint64_t full = (n >> log_mp) << log_v;  // stream vectors of the complete pages
    for (uint64_t q0 = gwarp * kW; q0 < total; q0 += nwarps * kW) {
        const uint64_t p0 = q0 >> log_v;
        const unsigned j0 = small_v ? 0u : (unsigned)((q0 & ((1ull << log_v) - 1)) >> log_vpm);
        if (q0 + kW <= full) {  // whole pages only (all but the last iterations): no row masks
            int4 x[kPaxU];
#pragma unroll
            for (int u = 0; u < kPaxU; ++u) {
                const unsigned o = (unsigned)u * 32 + lane;
                uint64_t p;
                unsigned col, v;
                if (small_v) { p = p0 + dpage[u]; col = colv[u] >> 16; v = colv[u] & 0xffffu; }
                else { p = p0; col = (unsigned)cols[j0 + (o >> log_vpm)]; v = o & vmask; }
                x[u] = ld_stream(reinterpret_cast<const int4 *>(data + ((((p << log_ncols) + col) << log_mp) + 4 * (uint64_t)v)));
            }
#pragma unroll
            for (int u = 0; u < kPaxU; ++u) acc += (long long)x[u].x + x[u].y + x[u].z + x[u].w;
            continue;
        }
        int4 x[kPaxU];
        unsigned sel4[kPaxU];
#pragma unroll
        for (int u = 0; u < kPaxU; ++u) {
            const unsigned o = (unsigned)u * 32 + lane;
            uint64_t p;
            unsigned col, v;
            if (small_v) { p = p0 + dpage[u]; col = colv[u] >> 16; v = colv[u] & 0xffffu; }
            else { p = p0; col = (unsigned)cols[j0 + (o >> log_vpm)]; v = o & vmask; }
            const uint64_t row0 = (p << log_mp) + 4 * (uint64_t)v;
            sel4[u] = (q0 + o >= total || row0 >= n) ? 0u : (n - row0 >= 4 ? 0xfu : (1u << (unsigned)(n - row0)) - 1u);
            if (sel4[u]) {
                const uint64_t off = (((p << log_ncols) + col) << log_mp) + 4 * (uint64_t)v;
                x[u] = ld_stream(reinterpret_cast<const int4 *>(data + off));
            }
        }
#pragma unroll
        for (int u = 0; u < kPaxU; ++u)
            if (sel4[u]) acc += lanes_sum(x[u], sel4[u]);
    }
    block_add(acc, out);
}

// NSM: records of 2^log_ncols attributes (>= 4) back to back; vector e holds attributes
// (4e mod ncols) .. +3 of record 4e / ncols. Vectors without a selected attribute are not loaded.
__global__ void __launch_bounds__(kThreads)
nsm_sum_kernel(const int32_t *__restrict__ data, uint64_t n, int log_ncols, unsigned long long mask,
               unsigned long long *out) {
    const uint64_t nvec = (n << log_ncols) >> 2;
    const uint64_t step = (uint64_t)gridDim.x * blockDim.x;
    const unsigned vmask = (1u << (log_ncols - 2)) - 1u;  // vector index within a record
    long long acc = 0;
    uint64_t e = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x;
    for (; e < nvec; e += kUnroll * step) {
        int4 x[kUnroll];
        unsigned sel4[kUnroll];
#pragma unroll
        for (int u = 0; u < kUnroll; ++u) {
            const uint64_t ei = e + u * step;
            sel4[u] = ei < nvec ? (unsigned)(mask >> (4 * ((unsigned)ei & vmask))) & 0xfu : 0u;
            if (sel4[u]) x[u] = ld_stream(reinterpret_cast<const int4 *>(data) + ei);
        }
#pragma unroll
        for (int u = 0; u < kUnroll; ++u)
            if (sel4[u]) acc += lanes_sum(x[u], sel4[u]);
    }
    block_add(acc, out);
}

unsigned grid_for(uint64_t items, int num_sms) {
    const uint64_t want = (items + kThreads - 1) / kThreads;
    const uint64_t cap = (uint64_t)num_sms * 8;  // 8 x 256 threads resident per SM
    return (unsigned)(want < 1 ? 1 : (want > cap ? cap : want));
}

}  // namespace

void launch_layout_sum(const int32_t *data, int layout, uint64_t n, int log_ncols, int log_mp,
                       uint64_t dsm_stride, unsigned long long mask, const LayoutSel &sel,
                       unsigned long long *out, int num_sms, cudaStream_t st) {
    if (layout == kLayoutDsm) {
        const unsigned gx = grid_for(((n >> 2) + kUnroll - 1) / kUnroll, num_sms);
        const unsigned per_col = (gx + sel.n - 1) / sel.n;  // total resident blocks ~ one wave
        dsm_sum_kernel<<<dim3(per_col ? per_col : 1, sel.n), kThreads, 0, st>>>(data, dsm_stride, n, sel, out);
    } else if (layout == kLayoutPax) {
        const uint64_t pages = (n + (1ull << log_mp) - 1) >> log_mp;
        const uint64_t vpm = 1ull << (log_mp - 2);
        static const bool general = [] { const char *v = std::getenv("H2TAP_PAX_GENERAL"); return v && v[0] == '1'; }();
        if (!general && (sel.n & (sel.n - 1)) == 0) {  // N a power of two
            int log_n = 0;
            while ((1 << log_n) < sel.n) ++log_n;
            pax_pow2_sum_kernel<<<grid_for(pages * sel.n * vpm / kPaxU, num_sms), kThreads, 0, st>>>(
                data, n, log_ncols, log_mp, log_n, sel, out);
        } else {
            pax_sum_kernel<<<grid_for(pages * sel.n * vpm / kUnroll, num_sms), kThreads, 0, st>>>(
                data, n, log_ncols, log_mp, sel, out);
        }
    } else {
        nsm_sum_kernel<<<grid_for(((n << log_ncols) >> 2) / kUnroll, num_sms), kThreads, 0, st>>>(
            data, n, log_ncols, mask, out);
    }
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

cudaError_t set_attributes_layout(int num_sms) {
    (void)num_sms;
    static const void *const kKernels[] = {
        (const void *)dsm_sum_kernel,
        (const void *)nsm_sum_kernel,
        (const void *)pax_sum_kernel,
        (const void *)pax_pow2_sum_kernel};
    const cudaError_t le = force_load(kKernels, sizeof kKernels / sizeof kKernels[0]);
    if (le != cudaSuccess) return le;
    return cudaSuccess;
}

}  // namespace h2tap
