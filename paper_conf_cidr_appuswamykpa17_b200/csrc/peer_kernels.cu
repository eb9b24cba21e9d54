// peer_kernels.cu — the generic cross-GPU merge kernels (a7) over the peer
// segments of peer.cuh: a fused sum-allreduce of a few int64 partials (Q6, Q14), a multi-block
// push of a variable-length list into every rank's mailbox (Q1 group lists, ORDER BY bucket
// histograms, NEXT-2 group tables), and a wait kernel for consumers that are plain kernels.
//
// The paper runs on one GPU and names multi-GPU placement as future work;
// its portability layer is message passing between "archipelagos" (L658-662). Here the messages
// are stores into the receiver's memory over NVLink/NVSwitch, ordered by release/acquire flags.
#include <cstdint>
#include <cuda_runtime.h>

#include "kernels.cuh"
#include "peer.cuh"

namespace h2tap {
namespace {
using namespace peer;

// One warp: push n partials to every rank, signal, wait for all, sum in rank order (integer sums
// are associative: bit-exact whatever the order).
__global__ void peer_allreduce_i64_kernel(PeerArgs p, const long long *src, int n, long long *dst,
                                          long long *host_dst) {
    pdl_wait();
    trigger_before_wait(p);
    const unsigned long long s = next_seq(p);
    const int par = (int)(s & 1);
    const int t = threadIdx.x;
    if (t < n) {
        const long long v = src[t];
        for (int k = 0; k < p.world; ++k)
            reinterpret_cast<long long *>(mbox(p, k, par, p.rank))[t] = v;
    }
    __syncwarp();
    if (t == 0) signal_all(p, s);
    __syncwarp();
    int ok = 0;
    if (t == 0) ok = wait_all(p, s) ? 1 : 0;
    ok = __shfl_sync(0xffffffffu, ok, 0);
    trigger_after_wait(p);
    if (t < n) {
        long long acc = 0;
        if (ok)
            for (int k = 0; k < p.world; ++k) {
                const long long *m = reinterpret_cast<const long long *>(mbox(p, p.rank, par, k));
                acc += __ldcg(m + t);
            }
        dst[t] = acc;
        if (host_dst) host_dst[t] = acc;
    }
}

// Grid-stride copy of the list into every rank's mailbox slot [s & 1][rank]; the last block to
// finish publishes s to every rank. Payload copied in 16-byte units (slots are 16-byte aligned).
__global__ void __launch_bounds__(256)
peer_push_kernel(PeerArgs p, const void *src, const unsigned long long *count_dev,
                 unsigned long long count_const, unsigned int elem_bytes) {
    pdl_wait();
    pdl_trigger();
    const unsigned long long s = next_seq(p);
    const int par = (int)(s & 1);
    unsigned long long count = count_dev ? *count_dev : count_const;
    const unsigned long long cap = (p.slot_bytes - 16) / elem_bytes;
    if (count > cap) count = cap;  // (callers size their lists below the slot; guard anyway)
    const unsigned long long bytes = count * elem_bytes;
    const unsigned long long nvec = (bytes + 15) / 16;
    const uint4 *sv = static_cast<const uint4 *>(src);
    const unsigned long long stride = (unsigned long long)gridDim.x * blockDim.x;
    for (int k = 0; k < p.world; ++k) {
        char *slot = mbox(p, k, par, p.rank);
        if (blockIdx.x == 0 && threadIdx.x == 0) *reinterpret_cast<unsigned long long *>(slot) = count;
        uint4 *dv = reinterpret_cast<uint4 *>(slot + 16);
        for (unsigned long long i = (unsigned long long)blockIdx.x * blockDim.x + threadIdx.x; i < nvec; i += stride)
            dv[i] = __ldg(sv + i);
    }
    if (block_done_last(p)) signal_all(p, s);
}

__global__ void peer_wait_kernel(PeerArgs p) {
    pdl_wait();
    trigger_before_wait(p);
    wait_all(p, cur_seq(p));
    trigger_after_wait(p);
}

}  // namespace

void launch_peer_allreduce_i64(const PeerArgs &p, const long long *src, int n, long long *dst,
                               long long *host_dst, cudaStream_t st) {
    launch_pdl(peer_allreduce_i64_kernel, 1, 32, 0, st, p, src, n, dst, host_dst);
    count_launches(1);
}

void launch_peer_push(const PeerArgs &p, const void *src, const unsigned long long *count_dev,
                      unsigned long long count_const, unsigned int elem_bytes, int num_sms, cudaStream_t st) {
    // the lists are small (Q1: <= 16 groups on TPC-C data; ORDER BY counts: <= 128 KB) and every
    // block ends with a system-scope fence before the last-block ticket: a few blocks, each
    // looping, instead of a block per SM (a 2 MB worst-case list then takes ~16 iterations)
    const unsigned long long max_bytes = count_dev ? p.slot_bytes - 16 : count_const * elem_bytes;
    unsigned long long blocks = (max_bytes / 16 + 255) / 256;
    const unsigned long long cap = (unsigned long long)(num_sms < 32 ? num_sms : 32);
    if (blocks > cap) blocks = cap;
    if (blocks < 1) blocks = 1;
    launch_pdl(peer_push_kernel, (unsigned)blocks, 256, 0, st, p, src, count_dev, count_const, elem_bytes);
    count_launches(1);
}

void launch_peer_wait(const PeerArgs &p, cudaStream_t st) {
    launch_pdl(peer_wait_kernel, 1, 1, 0, st, p);
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

cudaError_t set_attributes_peer(int num_sms) {
    (void)num_sms;
    static const void *const kKernels[] = {
        (const void *)peer_allreduce_i64_kernel,
        (const void *)peer_push_kernel,
        (const void *)peer_wait_kernel};
    const cudaError_t le = force_load(kKernels, sizeof kKernels / sizeof kKernels[0]);
    if (le != cudaSuccess) return le;
    return cudaSuccess;
}

}  // namespace h2tap
