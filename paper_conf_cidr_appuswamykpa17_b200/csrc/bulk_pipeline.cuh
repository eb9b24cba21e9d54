// bulk_pipeline.cuh — 1-D TMA bulk copies (cp.async.bulk, SASS UBLKCP) into a shared-memory ring
// of stages guarded by mbarriers: one elected producer thread streams column chunks from HBM,
// consumer warps compute on shared memory. Used by the scan kernels: the copy
// engine keeps `stages x stage bytes` in flight per SM without holding registers.
#pragma once
#include <cstdint>

namespace h2tap {

__device__ __forceinline__ uint32_t smem_u32(const void *p) {
    return static_cast<uint32_t>(__cvta_generic_to_shared(p));
}
__device__ __forceinline__ void mbar_init(uint64_t *bar, unsigned count) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" :: "r"(smem_u32(bar)), "r"(count) : "memory");
}
// make the barrier initialisation visible to the async (TMA) proxy
__device__ __forceinline__ void fence_mbar_init() {
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}
__device__ __forceinline__ void mbar_arrive_expect_tx(uint64_t *bar, unsigned bytes) {
    asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;"
                 :: "r"(smem_u32(bar)), "r"(bytes) : "memory");
}
__device__ __forceinline__ void mbar_arrive(uint64_t *bar) {
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" :: "r"(smem_u32(bar)) : "memory");
}
__device__ __forceinline__ void mbar_wait(uint64_t *bar, unsigned parity) {
    asm volatile(
        "{\n\t.reg .pred p;\n"
        "WAIT_%=:\n\t"
        "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n\t"
        "@!p bra WAIT_%=;\n}"
        :: "r"(smem_u32(bar)), "r"(parity) : "memory");
}
// the same with a suspend-time hint (ns): the waiting warp is parked instead of re-issuing
// try_wait, leaving issue slots to the block's other warps
__device__ __forceinline__ void mbar_wait_hint(uint64_t *bar, unsigned parity, unsigned ns) {
    asm volatile(
        "{\n\t.reg .pred p;\n"
        "WAIT_%=:\n\t"
        "mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1, %2;\n\t"
        "@!p bra WAIT_%=;\n}"
        :: "r"(smem_u32(bar)), "r"(parity), "r"(ns) : "memory");
}
// global -> shared bulk copy (size and addresses multiples of 16 B), completion on `bar`, with
// an L2 evict_first policy (each byte of a scan is read once)
__device__ __forceinline__ void bulk_g2s(void *dst, const void *src, unsigned bytes, uint64_t *bar,
                                         uint64_t policy) {
    asm volatile(
        "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint"
        " [%0], [%1], %2, [%3], %4;"
        :: "r"(smem_u32(dst)), "l"(src), "r"(bytes), "r"(smem_u32(bar)), "l"(policy) : "memory");
}
__device__ __forceinline__ uint64_t policy_evict_first() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(p));
    return p;
}
__device__ __forceinline__ unsigned round16(unsigned b) { return (b + 15u) & ~15u; }

}  // namespace h2tap
