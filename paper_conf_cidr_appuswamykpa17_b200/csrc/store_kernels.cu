// store_kernels.cu — a1 snapshot refresh helpers: per-column min/max statistics of the rows a
// refresh appends, computed on the copy stream right after the H2D copy (a zone map per column).
// The planner uses them to lay out join indexes; they are metadata of the
// snapshot, exactly like its row counts, and are published atomically with the epoch.
// (Refresh-side kernels are not counted in a query's kernel_launches.)
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

}  // namespace

void launch_gate(unsigned long long ns, cudaStream_t st) { gate_kernel<<<1, 1, 0, st>>>(ns); }

void launch_stats_init(int *out, int n_pairs, cudaStream_t st) {
    stats_init_kernel<<<(n_pairs + 127) / 128, 128, 0, st>>>(out, n_pairs);
}

void launch_minmax_i32(const int32_t *p, uint64_t n, int *out, int num_sms, cudaStream_t st) {
    if (!n) return;
    uint64_t blocks = (n + 255) / 256;
    const uint64_t cap = (uint64_t)num_sms * 4;
    if (blocks > cap) blocks = cap;
    minmax_kernel<<<(unsigned)blocks, 256, 0, st>>>(p, n, out);
}

}  // namespace h2tap
