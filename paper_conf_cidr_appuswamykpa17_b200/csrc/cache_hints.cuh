// cache_hints.cuh — L2 eviction-priority policies for data that is re-read by a later kernel of
// the same query (keep it: evict_last) or read for the last time (drop it: evict_first).
#pragma once
#include <cstdint>

namespace h2tap {

__device__ __forceinline__ uint64_t l2_policy_evict_last() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(p));
    return p;
}
__device__ __forceinline__ uint64_t l2_policy_evict_first() {
    uint64_t p;
    asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(p));
    return p;
}
// 16-byte store / load with an L2 cache policy
__device__ __forceinline__ void st16_policy(void *ptr, unsigned long long a, unsigned long long b,
                                            uint64_t pol) {
    asm volatile("st.global.L2::cache_hint.v2.u64 [%0], {%1, %2}, %3;"
                 :: "l"(ptr), "l"(a), "l"(b), "l"(pol) : "memory");
}
__device__ __forceinline__ void ld16_policy(const void *ptr, unsigned long long &a,
                                            unsigned long long &b, uint64_t pol) {
    asm volatile("ld.global.L2::cache_hint.v2.u64 {%0, %1}, [%2], %3;"
                 : "=l"(a), "=l"(b) : "l"(ptr), "l"(pol));
}

}  // namespace h2tap
