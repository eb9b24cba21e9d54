// probe_device.cuh — the K4 probe's warp step, shared by the probe kernels
// (join_kernels.cu) and the batch's shared scan (scan_kernels.cu): each lane holds 4 consecutive
// order_line rows; runs of equal (w, d, o) are summed in the lane and across lanes (segmented
// shuffle scan), and every run end probes the orders index once and adds (sum, count) to
// acc[orders row] with two atomics. A run split over two warp steps is flushed twice (two
// atomic adds to the same accumulator): any partition into 128-row warp steps is correct.
#pragma once
#include <cstdint>

#include "join_index.cuh"
#include "kernels.cuh"

namespace h2tap {
namespace pd {
using namespace jx;
constexpr unsigned kPdFull = 0xffffffffu;

struct Key3 { int w, d, o; };
__device__ __forceinline__ bool eq3(const Key3 &a, const Key3 &b) {
    return (a.w == b.w) & (a.d == b.d) & (a.o == b.o);
}

// kFilter (CH Q3): only orders rows marked by the new_order ⋈ orders ⋈ customer kernel
// accumulate; the others skip their atomics.
// The marks are read from a bitmap (n_orders / 8 bytes: L2-resident), not from acc[].pad.
template <bool kFilter>
__device__ __forceinline__ unsigned int keep_row(const Q18Scratch &s, unsigned int row) {
    if (!kFilter || row == kNoRow) return row;
    return (__ldcg(s.qbits + (row >> 5)) >> (row & 31)) & 1u ? row : kNoRow;
}

template <bool kFilter>
__device__ __forceinline__ void flush_run(const Q18Scratch &s, const Key3 &k, long long sum,
                                          unsigned int cnt, bool ident) {
    const unsigned int row = keep_row<kFilter>(s, jx_lookup(s.jo, k.w, k.d, k.o, ident));
    if (row != kNoRow) {
        atomicAdd(reinterpret_cast<unsigned long long *>(&s.acc[row].sum), (unsigned long long)sum);
        atomicAdd(&s.acc[row].cnt, cnt);
    }
}

// One warp step over 128 consecutive rows, 4 per lane (k, a in registers; `valid` per lane;
// `ident` = jx_identity(s.jo), read once by the caller):
// in-lane runs, cross-lane segmented scan, one probe + two atomics per run (see above).
template <bool kFilter>
__device__ __forceinline__ void probe_lane_group(const Q18Scratch &s, const Key3 (&k)[4],
                                                 const long long (&a)[4], bool valid, int lane,
                                                 bool ident) {
        // in-lane runs: b[j] = row j starts a run; s[j], c[j] = running sum / count of its run
        bool b1 = !eq3(k[1], k[0]), b2 = !eq3(k[2], k[1]), b3 = !eq3(k[3], k[2]);
        long long s0 = a[0], s1 = (b1 ? 0 : s0) + a[1], s2 = (b2 ? 0 : s1) + a[2], s3 = (b3 ? 0 : s2) + a[3];
        unsigned c0 = 1, c1 = (b1 ? 0 : c0) + 1, c2 = (b2 ? 0 : c1) + 1, c3 = (b3 ? 0 : c2) + 1;
        const bool multi = b1 | b2 | b3;
        // does my first run continue the previous lane's last run?
        const int pw = __shfl_up_sync(kPdFull, k[3].w, 1), pd = __shfl_up_sync(kPdFull, k[3].d, 1),
                  po = __shfl_up_sync(kPdFull, k[3].o, 1);
        const bool pvalid = __shfl_up_sync(kPdFull, valid, 1);
        const bool cont = lane > 0 && valid && pvalid && pw == k[0].w && pd == k[0].d && po == k[0].o;
        const bool next_cont = __shfl_down_sync(kPdFull, cont, 1) && lane < 31;
        // segmented inclusive scan of the lanes' last partial runs (segment starts where a lane
        // does not continue, or where its last run starts inside the lane)
        const bool start = !cont || multi;
        const unsigned starts = __ballot_sync(kPdFull, start);
        const int seg = 31 - __clz(starts & (0xffffffffu >> (31 - lane)));
        long long is = s3;
        unsigned ic = c3;
#pragma unroll
        for (int off = 1; off < 32; off <<= 1) {
            const long long ts = __shfl_up_sync(kPdFull, is, off);
            const unsigned tc = __shfl_up_sync(kPdFull, ic, off);
            if (lane - off >= seg) { is += ts; ic += tc; }
        }
        // carry into my first run = inclusive value of the previous lane (if I continue it)
        long long carry_s = __shfl_up_sync(kPdFull, is, 1);
        unsigned carry_c = __shfl_up_sync(kPdFull, ic, 1);
        if (!cont) { carry_s = 0; carry_c = 0; }
        if (!valid) return;
        // runs ending inside the lane (rows 0..2; the first run also gets the carry) and the
        // lane's last run unless the next lane continues it: all lookups are issued first
        // (independent loads in flight together), then the atomics
        const bool f[4] = {b1, b2, b3, !next_cont};
        const long long fs[4] = {s0 + carry_s, s1 + (b1 ? 0 : carry_s), s2 + ((b1 | b2) ? 0 : carry_s), is};
        const unsigned fc[4] = {c0 + carry_c, c1 + (b1 ? 0 : carry_c), c2 + ((b1 | b2) ? 0 : carry_c), ic};
        // one probe + two atomics per run end, looping over this lane's run ends only (a lane
        // holds at most one end inside plus the flush of its last run: the warp iterates 1-2
        // times instead of executing four predicated probes)
        unsigned em = (unsigned)f[0] | ((unsigned)f[1] << 1) | ((unsigned)f[2] << 2) | ((unsigned)f[3] << 3);
        while (em) {
            const int j = __ffs(em) - 1;
            em &= em - 1;
            const Key3 kj = j == 0 ? k[0] : j == 1 ? k[1] : j == 2 ? k[2] : k[3];
            const long long sj = j == 0 ? fs[0] : j == 1 ? fs[1] : j == 2 ? fs[2] : fs[3];
            const unsigned cj = j == 0 ? fc[0] : j == 1 ? fc[1] : j == 2 ? fc[2] : fc[3];
            const unsigned int row = keep_row<kFilter>(s, jx_lookup(s.jo, kj.w, kj.d, kj.o, ident));
            if (row != kNoRow) {
                atomicAdd(reinterpret_cast<unsigned long long *>(&s.acc[row].sum), (unsigned long long)sj);
                atomicAdd(&s.acc[row].cnt, cj);
            }
        }
}


}  // namespace pd
}  // namespace h2tap
