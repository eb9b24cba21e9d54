// peer.cuh — device side of the cross-GPU merge (a7): every rank exposes ONE
// device allocation, its "peer segment", to the other ranks (CUDA IPC across processes, plain
// pointers between engines of one process), and the merge kernels move partial results with
// ordinary stores into the peers' segments over NVLink/NVSwitch, followed by a release flag.
// No host round trip, no NCCL call: a collective is a producer kernel (push + signal) and the
// consumer kernels that wait for every rank's flag, all stream-ordered on the compute stream.
//
// Segment layout (identical on every rank, so offsets are symmetric):
//   [0, kPeerCtlBytes)                       PeerCtl: flags written BY the peers, local counters
//   mailbox[parity][src]                     2 x kMaxRanks slots of PeerArgs::slot_bytes: small
//                                            per-rank payloads (partials, group lists, histograms)
//   heap[parity]                             2 x PeerArgs::heap_half: the ORDER BY exchange
// Protocol (sequence numbers, all device-resident so a batch needs no host value per call):
//   producer:  s = ctl(me).seq + 1; write data into every peer's mailbox[s & 1][me] (or heap);
//              __threadfence_system(); st.release.sys ctl(k).flag[me] = s for every k (incl. me);
//              ctl(me).seq = s.
//   consumer:  (any later kernel before the next producer) s = ctl(me).seq; spin until
//              ld.acquire.sys ctl(me).flag[k] >= s for every k; read mailbox[s & 1][k] locally.
// A rank can run at most one collective ahead of the slowest peer (it cannot finish collective
// s+1 before every peer produced s+1, which each does only after consuming s, in stream order),
// so two parities of every buffer suffice. Waits time out (PeerArgs::timeout_ns): the sticky
// error bit is written to mapped host memory and every later wait returns at once.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "kernels.cuh"

namespace h2tap {
namespace peer {

__device__ __forceinline__ PeerCtl *ctl(const PeerArgs &p, int k) {
    return reinterpret_cast<PeerCtl *>(p.seg[k]);
}
__device__ __forceinline__ char *mbox(const PeerArgs &p, int owner, int parity, int src) {
    return p.seg[owner] + kPeerCtlBytes + (size_t)(parity * kMaxRanks + src) * p.slot_bytes;
}
__device__ __forceinline__ char *heap(const PeerArgs &p, int owner, int parity) {
    return p.seg[owner] + kPeerCtlBytes + (size_t)2 * kMaxRanks * p.slot_bytes + (size_t)parity * p.heap_half;
}

__device__ __forceinline__ unsigned long long ld_acquire_sys(const unsigned long long *a) {
    unsigned long long v;
    asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(a) : "memory");
    return v;
}
__device__ __forceinline__ void st_release_sys(unsigned long long *a, unsigned long long v) {
    asm volatile("st.release.sys.global.u64 [%0], %1;" :: "l"(a), "l"(v) : "memory");
}
__device__ __forceinline__ unsigned long long ld_volatile(const unsigned long long *a) {
    return *reinterpret_cast<const volatile unsigned long long *>(a);
}
__device__ __forceinline__ unsigned long long now_ns() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    return t;
}

// The sequence number of the next collective (producer side).
__device__ __forceinline__ unsigned long long next_seq(const PeerArgs &p) {
    return ld_volatile(&ctl(p, p.rank)->seq) + 1;
}
// The sequence number the consumers of the latest produced collective wait for.
__device__ __forceinline__ unsigned long long cur_seq(const PeerArgs &p) {
    return ld_volatile(&ctl(p, p.rank)->seq);
}

__device__ __forceinline__ void set_err(const PeerArgs &p, unsigned int bits) {
    atomicOr(&ctl(p, p.rank)->err, bits);
    if (p.err_host) atomicOr_system(p.err_host, bits);
}

// One thread: publish collective s to every rank (after this thread's — or, through a
// last-block ticket, every block's — data stores), then record s as issued.
__device__ __forceinline__ void signal_all(const PeerArgs &p, unsigned long long s) {
    __threadfence_system();
    for (int k = 0; k < p.world; ++k) st_release_sys(&ctl(p, k)->flag[p.rank], s);
    ctl(p, p.rank)->seq = s;
}

// One thread: wait until every rank delivered collective s (or time out: sticky error).
// Returns false on a (current or earlier) transport error.
__device__ __forceinline__ bool wait_all(const PeerArgs &p, unsigned long long s) {
    PeerCtl *me = ctl(p, p.rank);
    if (*reinterpret_cast<volatile unsigned int *>(&me->err) & kPeerErrTimeout) return false;
    const unsigned long long t0 = now_ns();
    for (int k = 0; k < p.world; ++k) {
        unsigned int spins = 0;
        while (ld_acquire_sys(&me->flag[k]) < s) {
            if ((++spins & 255u) == 0u && now_ns() - t0 > p.timeout_ns) {
                if (p.err_host) {  // diagnostics for the host's error message: what was missing
                    volatile unsigned int *d = p.err_host;
                    d[1] = (unsigned int)s;
                    d[2] = (unsigned int)k;
                    d[3] = (unsigned int)ld_acquire_sys(&me->flag[k]);
                }
                set_err(p, kPeerErrTimeout);
                return false;
            }
            __nanosleep(64);
        }
    }
    return true;
}

// PDL trigger of a kernel that waits for peers: early when no other rank shares this device, else
// after the wait (PeerArgs::shared_device). Called by every thread at both places.
__device__ __forceinline__ void trigger_before_wait(const PeerArgs &p) { if (!p.shared_device) pdl_trigger(); }
__device__ __forceinline__ void trigger_after_wait(const PeerArgs &p) { if (p.shared_device) pdl_trigger(); }

// Block-level helpers: thread 0 waits, the block learns the outcome.
__device__ __forceinline__ bool block_wait_all(const PeerArgs &p, unsigned long long s) {
    __shared__ int ok;
    if (threadIdx.x == 0) ok = wait_all(p, s) ? 1 : 0;
    __syncthreads();
    return ok != 0;
}

// Last-block detection for multi-block producers: every block calls this after its peer stores;
// returns true in exactly one thread of the last block (all blocks' stores are then ordered
// before that thread's later release stores by the fences + the ticket's atomic).
__device__ __forceinline__ bool block_done_last(const PeerArgs &p) {
    __shared__ int last;
    __threadfence_system();
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned int *t = &ctl(p, p.rank)->ticket;
        last = atomicAdd(t, 1u) == gridDim.x - 1;
        if (last) *t = 0;  // self-reset (no other block touches it any more in this launch)
    }
    __syncthreads();
    return threadIdx.x == 0 && last;
}

}  // namespace peer
}  // namespace h2tap
