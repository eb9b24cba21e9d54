// join_index.cuh — device side of the (w, d, id) -> row join index, shared by
// the Q18 kernels (join_kernels.cu) and the NEXT-2 CH queries (ch_kernels.cu). Product code only.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

#include "kernels.cuh"

namespace h2tap {
namespace jx {

__device__ __forceinline__ unsigned long long fmix64(unsigned long long k) {
    k ^= k >> 33; k *= 0xff51afd7ed558ccdull; k ^= k >> 33; k *= 0xc4ceb9fe1a85ec53ull; k ^= k >> 33;
    return k;
}

// (w, d, id) -> 64-bit key, injective on the supported domain (R16).
__device__ __forceinline__ bool pack_key(int w, int d, int id, unsigned long long &k) {
    k = ((unsigned long long)(unsigned)w << 40) | ((unsigned long long)(unsigned)d << 32) |
        (unsigned long long)(unsigned)id;
    return ((unsigned)w < (1u << 23)) & ((unsigned)d < 256u) & (id >= 0);
}

// Dense slot of (w, d, id) in the index's box, or false when outside it.
__device__ __forceinline__ bool dense_slot(const JoinIndex &j, int w, int d, int id,
                                          unsigned long long &slot) {
    const unsigned dw = (unsigned)(w - j.w0), dd = (unsigned)(d - j.d0), dk = (unsigned)(id - j.k0);
    slot = ((unsigned long long)dw * j.nd + dd) * j.nk + dk;
    return (dw < j.nw) & (dd < j.nd) & (dk < j.nk);
}

// Insert; returns false on a key outside the supported domain. Duplicates set `dupbit`.
__device__ __forceinline__ bool jx_insert(const JoinIndex &j, int w, int d, int id, unsigned int row,
                                          unsigned int *err, unsigned int dupbit) {
    if (j.dense) {
        unsigned long long s;
        if (!dense_slot(j, w, d, id, s)) return false;  // stats must cover every build row
        if (atomicCAS(j.slots + s, kNoRow, row) != kNoRow) atomicOr(err, dupbit);
        return true;
    }
    unsigned long long key;
    if (!pack_key(w, d, id, key)) return false;
    unsigned long long h = fmix64(key) & j.mask;
    while (true) {
        const unsigned long long prev = atomicCAS(&j.ht[h].key, kEmpty, key);
        if (prev == kEmpty) { j.ht[h].row = row; return true; }
        if (prev == key) { atomicOr(err, dupbit); return true; }
        h = (h + 1) & j.mask;
    }
}

// The build side is stored in key order with no gap (verified by the init kernel): row == slot.
__device__ __forceinline__ bool jx_identity(const JoinIndex &j) {
    return j.dense && j.may_ident && __ldg(j.viol) == 0u;
}

// `ident` = jx_identity(j), read once per kernel by callers in a hot loop (the verdict is a global
// load: one L1 round trip per lookup otherwise, and an L2 one when a kernel's shared memory leaves
// L1 little room)
__device__ __forceinline__ unsigned int jx_lookup(const JoinIndex &j, int w, int d, int id, bool ident) {
    if (j.dense) {
        unsigned long long s;
        if (!dense_slot(j, w, d, id, s)) return kNoRow;  // outside the build box: no match
        H2TAP_CHECK(s < j.range);
        if (ident) return (unsigned int)s;                // clustered build side: positional
        return __ldcg(j.slots + s);
    }
    unsigned long long key;
    if (!pack_key(w, d, id, key)) return kNoRow;  // no build key can lie outside the domain
    unsigned long long h = fmix64(key) & j.mask;
    while (true) {
        const ulonglong2 s = __ldcg(reinterpret_cast<const ulonglong2 *>(j.ht + h));
        if (s.x == key) return (unsigned int)s.y;
        if (s.x == kEmpty) return kNoRow;
        h = (h + 1) & j.mask;
    }
}

__device__ __forceinline__ unsigned int jx_lookup(const JoinIndex &j, int w, int d, int id) {
    return jx_lookup(j, w, d, id, jx_identity(j));
}

__host__ __device__ __forceinline__ uint64_t jx_words(const JoinIndex &j) {  // 16-byte units
    return j.dense ? (j.range + 3) / 4 : j.mask + 1;
}
__device__ __forceinline__ void jx_clear(const JoinIndex &j, uint64_t i) {
    if (j.dense) reinterpret_cast<uint4 *>(j.slots)[i] = make_uint4(kNoRow, kNoRow, kNoRow, kNoRow);
    else reinterpret_cast<ulonglong2 *>(j.ht)[i] = make_ulonglong2(kEmpty, 0ull);
}

}  // namespace jx
}  // namespace h2tap
