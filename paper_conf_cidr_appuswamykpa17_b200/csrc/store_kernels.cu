// store_kernels.cu — a1 snapshot refresh helpers: per-column min/max statistics of the rows a
// refresh appends, computed on the copy stream right after the H2D copy (a zone map per column).
// The planner uses them to lay out join indexes; they are metadata of the
// snapshot, exactly like its row counts, and are published atomically with the epoch.
// (Refresh-side kernels are not counted in a query's kernel_launches.)
//
// In-place updates (the paper's copy-on-write): a
// column that receives updates keeps two device buffers, the visible version `cur` and a shadow
// `alt` (the previous version). A one-bit-per-page map records the pages where the two differ.
// A new version is built in the shadow: cow_catchup copies the dirty pages (and the rows
// appended since the shadow was last in sync) cur -> alt, apply_updates scatters the new values
// into alt and marks their pages; then the engine swaps the roles. Views of earlier epochs keep
// reading their own buffer; page-granular traffic replaces a whole-column copy per epoch.
#include <climits>
#include <cstdint>
#include <cuda_runtime.h>

#include "kernels.cuh"

namespace h2tap {
namespace {

__global__ void stats_init_kernel(int *out, int n_pairs) {
    const int i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i < n_pairs) { out[2 * i] = INT_MAX; out[2 * i + 1] = INT_MIN; }
}

__global__ void stats_init64_kernel(long long *out, int n_pairs) {
    const int i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i < n_pairs) { out[2 * i] = INT64_MAX; out[2 * i + 1] = INT64_MIN; }
}

__global__ void __launch_bounds__(256) minmax64_kernel(const int64_t *__restrict__ p, uint64_t n, long long *out) {
    long long mn = INT64_MAX, mx = INT64_MIN;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        const long long v = __ldcs(reinterpret_cast<const long long *>(p) + i);
        mn = min(mn, v);
        mx = max(mx, v);
    }
    for (int o = 16; o; o >>= 1) {
        mn = min(mn, __shfl_xor_sync(0xffffffffu, mn, o));
        mx = max(mx, __shfl_xor_sync(0xffffffffu, mx, o));
    }
    if ((threadIdx.x & 31) == 0 && mn <= mx) {
        atomicMin(out, mn);
        atomicMax(out + 1, mx);
    }
}

__global__ void __launch_bounds__(256) minmax_kernel(const int32_t *__restrict__ p, uint64_t n, int *out) {
    int mn = INT_MAX, mx = INT_MIN;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        const int v = __ldcs(p + i);
        mn = min(mn, v);
        mx = max(mx, v);
    }
    mn = __reduce_min_sync(0xffffffffu, mn);
    mx = __reduce_max_sync(0xffffffffu, mx);
    if ((threadIdx.x & 31) == 0 && mn <= mx) {
        atomicMin(out, mn);
        atomicMax(out + 1, mx);
    }
}

// Profiling gate: holds the stream for `ns` nanoseconds so the host can enqueue a query's
// kernels behind it; per-kernel CUDA events then bracket only GPU execution, not host launch
// latency (used with H2TAP_QUERY_PROFILE only).
__global__ void gate_kernel(unsigned long long ns) {
    unsigned long long t0, t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t0));
    do {
        __nanosleep(1000);
        asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    } while (t - t0 < ns);
}

// Copy, cur -> alt, every page whose dirty bit is set among pages [0, synced_pages) and every
// page overlapping rows [tail_lo, n_rows). One block per page at a time (grid-stride over pages);
// a full page is moved with every load of a thread issued before its stores (16 KB / 32 KB in
// flight per block); byte ranges rounded up to 16 (buffers carry >= kPadRows rows of padding).
// The same launch clears `next_bits`, the map apply_updates fills for the next epoch.
template <int kVecPerThread>  // = kCowPageRows * es / 16 / 256: 4 (int32) or 8 (int64)
__global__ void __launch_bounds__(256) cow_catchup_kernel(uint8_t *__restrict__ dst,
                                                          const uint8_t *__restrict__ src,
                                                          const uint32_t *__restrict__ bits,
                                                          uint32_t *__restrict__ next_bits, uint64_t nwords,
                                                          uint64_t synced_rows, uint64_t n_rows,
                                                          unsigned long long *pages_copied) {
    constexpr uint64_t kPageBytes = (uint64_t)kVecPerThread * 16 * 256;
    for (uint64_t w = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; w < nwords;
         w += (uint64_t)gridDim.x * blockDim.x)
        next_bits[w] = 0u;
    const uint64_t npages = (n_rows + kCowPageRows - 1) / kCowPageRows;
    const uint64_t tail_page = synced_rows / kCowPageRows;
    const uint64_t row_bytes = kPageBytes / kCowPageRows;
    for (uint64_t p = blockIdx.x; p < npages; p += gridDim.x) {
        const bool dirty = p >= tail_page || ((__ldg(bits + (p >> 5)) >> (p & 31)) & 1u);
        if (!dirty) continue;
        const uint4 *s4 = reinterpret_cast<const uint4 *>(src + p * kPageBytes);
        uint4 *d4 = reinterpret_cast<uint4 *>(dst + p * kPageBytes);
        if ((p + 1) * kCowPageRows <= n_rows) {
            uint4 v[kVecPerThread];
#pragma unroll
            for (int k = 0; k < kVecPerThread; ++k) v[k] = __ldcs(s4 + k * 256 + threadIdx.x);
#pragma unroll
            for (int k = 0; k < kVecPerThread; ++k) __stcs(d4 + k * 256 + threadIdx.x, v[k]);
        } else {  // ragged last page
            const uint64_t nv = ((n_rows - p * kCowPageRows) * row_bytes + 15) / 16;
            for (uint64_t i = threadIdx.x; i < nv; i += blockDim.x) __stcs(d4 + i, __ldcs(s4 + i));
        }
        if (threadIdx.x == 0) atomicAdd(pages_copied, 1ull);
    }
}

// alt[rows[i]] = vals[i], and mark the page of rows[i] dirty (cur and alt now differ there).
// Updates arrive clustered (a delivered order's lines are adjacent rows): a lane whose page
// equals its left neighbour's leaves the bit to that lane, and the word is read first, so a page
// costs about one atomic, not one per row.
template <class T>
__global__ void __launch_bounds__(256) apply_updates_kernel(T *__restrict__ col, uint32_t *bits,
                                                            const uint32_t *__restrict__ rows,
                                                            const T *__restrict__ vals, uint64_t n) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    const int lane = threadIdx.x & 31;
    // every lane of a warp runs the same iterations (stride and start are warp-aligned)
    for (uint64_t base = (uint64_t)blockIdx.x * blockDim.x; base < n; base += stride) {
        const uint64_t i = base + threadIdx.x;
        const bool valid = i < n;
        uint32_t page = 0xffffffffu;
        if (valid) {
            const uint32_t r = __ldg(rows + i);
            col[r] = __ldg(vals + i);
            page = r / kCowPageRows;
        }
        const uint32_t left = __shfl_up_sync(0xffffffffu, page, 1);
        const uint32_t m = 1u << (page & 31);
        if (valid && !(lane > 0 && left == page) && !(__ldcg(bits + (page >> 5)) & m))
            atomicOr(bits + (page >> 5), m);
    }
}

}  // namespace

void launch_cow_catchup(void *dst, const void *src, uint32_t es, const uint32_t *bits,
                        uint32_t *next_bits, uint64_t nwords, uint64_t synced_rows, uint64_t n_rows,
                        unsigned long long *pages_copied, int num_sms, cudaStream_t st) {
    const uint64_t npages = (n_rows + kCowPageRows - 1) / kCowPageRows;
    const uint64_t cap = (uint64_t)num_sms * 8;
    uint64_t grid = npages < cap ? npages : cap;
    const uint64_t wgrid = (nwords + 255) / 256;
    if (grid < wgrid) grid = wgrid < cap ? wgrid : cap;
    if (!grid) return;
    auto *d = static_cast<uint8_t *>(dst);
    const auto *s = static_cast<const uint8_t *>(src);
    if (es == 4)
        cow_catchup_kernel<4><<<(unsigned)grid, 256, 0, st>>>(d, s, bits, next_bits, nwords, synced_rows,
                                                              n_rows, pages_copied);
    else
        cow_catchup_kernel<8><<<(unsigned)grid, 256, 0, st>>>(d, s, bits, next_bits, nwords, synced_rows,
                                                              n_rows, pages_copied);
}

void launch_apply_updates(void *col, uint32_t es, uint32_t *bits, const uint32_t *rows,
                          const void *vals, uint64_t n, int num_sms, cudaStream_t st) {
    if (!n) return;
    uint64_t blocks = (n + 255) / 256;
    const uint64_t cap = (uint64_t)num_sms * 8;
    if (blocks > cap) blocks = cap;
    if (es == 4)
        apply_updates_kernel<int32_t><<<(unsigned)blocks, 256, 0, st>>>(
            static_cast<int32_t *>(col), bits, rows, static_cast<const int32_t *>(vals), n);
    else
        apply_updates_kernel<int64_t><<<(unsigned)blocks, 256, 0, st>>>(
            static_cast<int64_t *>(col), bits, rows, static_cast<const int64_t *>(vals), n);
}

void launch_gate(unsigned long long ns, cudaStream_t st) { gate_kernel<<<1, 1, 0, st>>>(ns); }

void launch_stats_init(int *out, int n_pairs, cudaStream_t st) {
    stats_init_kernel<<<(n_pairs + 127) / 128, 128, 0, st>>>(out, n_pairs);
}

void launch_stats_init64(long long *out, int n_pairs, cudaStream_t st) {
    stats_init64_kernel<<<(n_pairs + 127) / 128, 128, 0, st>>>(out, n_pairs);
}

void launch_minmax_i64(const int64_t *p, uint64_t n, long long *out, int num_sms, cudaStream_t st) {
    if (!n) return;
    uint64_t blocks = (n + 255) / 256;
    const uint64_t cap = (uint64_t)num_sms * 4;
    if (blocks > cap) blocks = cap;
    minmax64_kernel<<<(unsigned)blocks, 256, 0, st>>>(p, n, out);
}

void launch_minmax_i32(const int32_t *p, uint64_t n, int *out, int num_sms, cudaStream_t st) {
    if (!n) return;
    uint64_t blocks = (n + 255) / 256;
    const uint64_t cap = (uint64_t)num_sms * 4;
    if (blocks > cap) blocks = cap;
    minmax_kernel<<<(unsigned)blocks, 256, 0, st>>>(p, n, out);
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

cudaError_t set_attributes_store(int num_sms) {
    (void)num_sms;
    static const void *const kKernels[] = {
        (const void *)apply_updates_kernel<int32_t>,
        (const void *)apply_updates_kernel<int64_t>,
        (const void *)cow_catchup_kernel<4>,
        (const void *)cow_catchup_kernel<8>,
        (const void *)gate_kernel,
        (const void *)minmax_kernel,
        (const void *)stats_init_kernel, (const void *)stats_init64_kernel, (const void *)minmax64_kernel};
    const cudaError_t le = force_load(kKernels, sizeof kKernels / sizeof kKernels[0]);
    if (le != cudaSuccess) return le;
    return cudaSuccess;
}

}  // namespace h2tap
