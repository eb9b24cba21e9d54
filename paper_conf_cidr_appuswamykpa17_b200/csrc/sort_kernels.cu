// sort_kernels.cu — a8 finalize for CH Q18: ORDER BY amount_sum DESC, o_entry_d ASC, then the
// (o_w_id, o_d_id, o_id) tie-break that makes the order total (R11).
//
// The three sort fields are mapped to unsigned integers whose widths come from the result's
// min/max (HAVING kernel statistics) and the snapshot's zone maps: a = max - amount_sum (DESC),
// e = o_entry_d - min, r = (w, d, o) offsets as concatenated fixed-width fields. a|e|r is the
// exact composite key.
//  * main path: a bucket sort (partition by the top key bits, then a sub-bucket partition and
//    rank counting per bucket in shared memory) of 128-bit carry records that hold the whole
//    result row when it fits, else of (top 64 bits of a|e|r, row id) pairs.
//    For the pairs: if a|e|r fits 64 bits the keys are
//    distinct and the order is exact; otherwise runs of equal 64-bit prefixes are ordered by the
//    full tuple (tie-fix; runs are a handful of rows on realistic data).
//  * exact fallback (a run > 32 rows or a bucket > shared memory): one stable LSD radix sort of
//    (key, row) pairs per field, r then e then a. Radix pass = per-tile digit histogram ->
//    per-digit scan -> stable scatter; keys travel with their row ids.
#include <algorithm>
#include <cstdint>
#include <cstdlib>
#include <cuda_runtime.h>

#include "cache_hints.cuh"
#include "join_index.cuh"
#include "kernels.cuh"
#include "peer.cuh"

// per-bucket emit geometry (A/B via scripts/build_variants.py): carry-record capacity of the small
// instance, its blocks per SM, and the row-id path's capacity (both share its shared memory)
#ifndef OB_CAP
#define OB_CAP 1536
#endif
#ifndef EMIT_BPS
#define EMIT_BPS 6
#endif
#ifndef ROW_CAP
#define ROW_CAP 1024
#endif

namespace h2tap {
namespace {

constexpr unsigned kFull = 0xffffffffu;
constexpr int kT = kSortThreads;         // 256
constexpr int kI = kSortItems;           // 16
constexpr int kWarps = kT / 32;
constexpr int kWarpTile = 32 * kI;       // 512

// ------------------------------------------------------------- radix pass --
__global__ void __launch_bounds__(kT)
hist_kernel(const unsigned long long *__restrict__ key, uint64_t n, int shift,
            unsigned int *__restrict__ counts, uint64_t ntiles) {
    __shared__ unsigned int h[256];
    for (int i = threadIdx.x; i < 256; i += kT) h[i] = 0;
    __syncthreads();
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const uint64_t base = (uint64_t)blockIdx.x * kSortTile + (uint64_t)warp * kWarpTile + lane;
    unsigned int dg[kI];
#pragma unroll
    for (int i = 0; i < kI; ++i) {
        const uint64_t j = base + i * 32;
        dg[i] = j < n ? (unsigned int)(__ldcg(key + j) >> shift) & 0xffu : 256u + lane;  // unique dummy
    }
#pragma unroll
    for (int i = 0; i < kI; ++i) {
        const unsigned int peers = __match_any_sync(kFull, dg[i]);
        if (dg[i] < 256u && lane == __ffs(peers) - 1) atomicAdd(&h[dg[i]], (unsigned int)__popc(peers));
    }
    __syncthreads();
    for (int d = threadIdx.x; d < 256; d += kT) counts[(uint64_t)d * ntiles + blockIdx.x] = h[d];
}

// One block per digit: exclusive scan of that digit's per-tile counts, total -> totals[d].
__global__ void __launch_bounds__(256) digit_scan_kernel(unsigned int *__restrict__ counts,
                                                         uint64_t ntiles,
                                                         unsigned int *__restrict__ totals) {
    __shared__ unsigned int wsum[8];
    unsigned int *row = counts + (uint64_t)blockIdx.x * ntiles;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    unsigned int carry = 0;
    for (uint64_t r0 = 0; r0 < ntiles; r0 += 256) {
        const uint64_t i = r0 + threadIdx.x;
        const unsigned int v = i < ntiles ? row[i] : 0u;
        unsigned int x = v;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const unsigned int t = __shfl_up_sync(kFull, x, o);
            if (lane >= o) x += t;
        }
        if (lane == 31) wsum[warp] = x;
        __syncthreads();
        unsigned int before = 0, all = 0;
#pragma unroll
        for (int w = 0; w < 8; ++w) {
            before += w < warp ? wsum[w] : 0u;
            all += wsum[w];
        }
        if (i < ntiles) row[i] = carry + before + x - v;
        carry += all;
        __syncthreads();
    }
    if (threadIdx.x == 0) totals[blockIdx.x] = carry;
}

__global__ void __launch_bounds__(kT)
scatter_kernel(const unsigned long long *__restrict__ kin, const unsigned int *__restrict__ vin,
               unsigned long long *__restrict__ kout, unsigned int *__restrict__ vout, uint64_t n,
               int shift, const unsigned int *__restrict__ counts, uint64_t ntiles,
               const unsigned int *__restrict__ totals) {
    __shared__ unsigned int wc[kWarps][256];  // per-warp digit counts -> running offsets
    __shared__ unsigned int dbase[256];
    __shared__ unsigned int ws[kWarps];
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    for (int i = threadIdx.x; i < kWarps * 256; i += kT) (&wc[0][0])[i] = 0;
    {   // exclusive scan of the 256 digit totals (every block recomputes it: 256 values)
        const unsigned int v = totals[threadIdx.x];
        unsigned int x = v;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const unsigned int t = __shfl_up_sync(kFull, x, o);
            if (lane >= o) x += t;
        }
        if (lane == 31) ws[warp] = x;
        __syncthreads();
        unsigned int before = 0;
        for (int w = 0; w < warp; ++w) before += ws[w];
        dbase[threadIdx.x] = before + x - v;
    }
    const uint64_t base = (uint64_t)blockIdx.x * kSortTile + (uint64_t)warp * kWarpTile + lane;
    unsigned long long k[kI];
    unsigned int v[kI], dg[kI];
#pragma unroll
    for (int i = 0; i < kI; ++i) {
        const uint64_t j = base + i * 32;
        if (j < n) {
            k[i] = __ldcs(kin + j);
            v[i] = __ldcs(vin + j);
            dg[i] = (unsigned int)(k[i] >> shift) & 0xffu;
        } else {
            k[i] = 0; v[i] = 0; dg[i] = 256u + lane;
        }
    }
    __syncthreads();
    unsigned int peers[kI];
#pragma unroll
    for (int i = 0; i < kI; ++i) {  // per-warp histogram (leaders only; __syncwarp orders RAW)
        peers[i] = __match_any_sync(kFull, dg[i]);
        if (dg[i] < 256u && lane == __ffs(peers[i]) - 1) wc[warp][dg[i]] += __popc(peers[i]);
        __syncwarp();
    }
    __syncthreads();
    {   // running offset of warp w for digit d = global digit base + tile offset + warps < w
        const int d = threadIdx.x;
        unsigned int run = dbase[d] + counts[(uint64_t)d * ntiles + blockIdx.x];
#pragma unroll
        for (int w = 0; w < kWarps; ++w) {
            const unsigned int c = wc[w][d];
            wc[w][d] = run;
            run += c;
        }
    }
    __syncthreads();
    const unsigned lt = (1u << lane) - 1u;
#pragma unroll
    for (int i = 0; i < kI; ++i) {  // stable scatter in (warp, item, lane) = index order
        if (dg[i] < 256u) {
            const unsigned int pos = wc[warp][dg[i]] + __popc(peers[i] & lt);
            kout[pos] = k[i];
            vout[pos] = v[i];
        }
        __syncwarp();
        if (dg[i] < 256u && lane == __ffs(peers[i]) - 1) wc[warp][dg[i]] += __popc(peers[i]);
        __syncwarp();
    }
}

// ------------------------------------------------------------ Q18 keys --
__device__ __forceinline__ unsigned long long field_a(long long amount, const Q18SortSpec &sp) {
    return (unsigned long long)sp.amt_max - (unsigned long long)amount;  // DESC
}
__device__ __forceinline__ unsigned long long field_e(const Q18Row &r, const Q18SortSpec &sp) {
    return (unsigned long long)r.o_entry_d - (unsigned long long)sp.ent_min;
}
__device__ __forceinline__ unsigned long long field_r(const Q18Row &r, const Q18SortSpec &sp) {
    // (w, d, o) as concatenated fixed-width fields: lexicographic order = integer order, and
    // the carry decode is shifts and masks (no division)
    const unsigned long long w = (unsigned)(r.o_w_id - sp.w_min);
    const unsigned long long d = (unsigned)(r.o_d_id - sp.d_min);
    const unsigned long long o = (unsigned)(r.o_id - sp.o_min);
    return (w << (sp.bits_d + sp.bits_o)) | (d << sp.bits_o) | o;
}

// top `prefix_bits` bits of the concatenation (a | e | r) with widths (bits_a, bits_e, bits_r)
__device__ __forceinline__ unsigned long long prefix_key(const Q18Row &r, long long amount,
                                                         const Q18SortSpec &sp) {
    const unsigned long long f[3] = {field_a(amount, sp), field_e(r, sp), field_r(r, sp)};
    const int b[3] = {sp.bits_a, sp.bits_e, sp.bits_r};
    unsigned long long p = 0;
    int room = sp.prefix_bits;
#pragma unroll
    for (int i = 0; i < 3; ++i) {
        const int take = b[i] < room ? b[i] : room;
        if (take > 0) {
            p = (take == 64 ? 0ull : (p << take)) | (f[i] >> (b[i] - take));
            room -= take;
        }
    }
    return p;
}

// full ORDER BY comparison: amount_sum DESC, o_entry_d, o_w_id, o_d_id, o_id
__device__ __forceinline__ bool row_less(const Q18Row &x, long long ax, const Q18Row &y, long long ay) {
    if (ax != ay) return ax > ay;
    if (x.o_entry_d != y.o_entry_d) return x.o_entry_d < y.o_entry_d;
    if (x.o_w_id != y.o_w_id) return x.o_w_id < y.o_w_id;
    if (x.o_d_id != y.o_d_id) return x.o_d_id < y.o_d_id;
    return x.o_id < y.o_id;
}

// ---- carry records: 128 bits = (top 64 key bits, low key bits | payload).
// The key K = a|e|r is unique per result row (r encodes the orders PK), so
// comparing (hi, lo) as one 128-bit integer is the exact ORDER BY; the payload
// (c_last, c_id, o_ol_cnt as offsets from their minima) rides in the lowest bits.
// Built with 64-bit shifts only: PTX shl / shr clamp shift amounts >= 64 to a zero result, so
// every field placement is branch-free (an unsigned "negative" amount is >= 64 too). With
// K = a << (R + E) | e << R | r held as (khi, klo), the record is (K >> L, (K mod 2^L) << P | pay)
// (L = bits_low, P = payload bits). The u128 formulation it replaced spent ~2x the instructions on
// variable 128-bit shifts: HAVING 45 -> 40 us, emit 64 -> 56 us measured.
__device__ __forceinline__ unsigned long long shl_c(unsigned long long x, unsigned s) {
    unsigned long long r;
    asm("shl.b64 %0, %1, %2;" : "=l"(r) : "l"(x), "r"(s));
    return r;
}
__device__ __forceinline__ unsigned long long shr_c(unsigned long long x, unsigned s) {
    unsigned long long r;
    asm("shr.u64 %0, %1, %2;" : "=l"(r) : "l"(x), "r"(s));
    return r;
}
__device__ __forceinline__ unsigned long long mask_c(unsigned b) { return shr_c(~0ull, 64u - b); }  // b in [0, 64]

__device__ __forceinline__ ulonglong2 carry_record(const Q18Row &r, long long amount, const Q18SortSpec &sp) {
    const unsigned R = (unsigned)sp.bits_r, pa = R + (unsigned)sp.bits_e, L = (unsigned)sp.bits_low;
    const unsigned P = (unsigned)(sp.bits_cl + sp.bits_ci + sp.bits_n);
    const unsigned long long a = field_a(amount, sp), e = field_e(r, sp), f = field_r(r, sp);
    const unsigned long long klo = shl_c(a, pa) | shl_c(e, R) | f;  // (R <= 62: e and r start in klo)
    const unsigned long long khi = shl_c(a, pa - 64u) | shr_c(a, 64u - pa) | shr_c(e, 64u - R);
    const unsigned long long pay =
        (((unsigned long long)((unsigned)r.c_last - (unsigned)sp.cl_min) << sp.bits_ci |
          (unsigned long long)((unsigned)r.c_id - (unsigned)sp.ci_min)) << sp.bits_n) |
        (unsigned long long)((unsigned)r.o_ol_cnt - (unsigned)sp.n_min);
    return make_ulonglong2(shl_c(khi, 64u - L) | shr_c(klo, L), shl_c(klo & mask_c(L), P) | pay);
}

struct CarryRow { long long amount, o_entry_d; int c_last, c_id, o_id, o_ol_cnt, o_w_id, o_d_id; };
__device__ __forceinline__ CarryRow carry_decode(unsigned long long hi, unsigned long long lo,
                                                 const Q18SortSpec &sp) {
    const unsigned R = (unsigned)sp.bits_r, E = (unsigned)sp.bits_e, pa = R + E, L = (unsigned)sp.bits_low;
    const unsigned bn = (unsigned)sp.bits_n, bci = (unsigned)sp.bits_ci, bo = (unsigned)sp.bits_o,
                   bd = (unsigned)sp.bits_d;
    const unsigned P = (unsigned)sp.bits_cl + bci + bn;
    const unsigned long long klo = shl_c(hi, L) | shr_c(lo, P), khi = shr_c(hi, 64u - L);
    const unsigned long long fr = klo & mask_c(R);
    const unsigned long long fe = (shr_c(klo, R) | shl_c(khi, 64u - R)) & mask_c(E);
    const unsigned long long fa = shr_c(klo, pa) | shl_c(khi, 64u - pa) | shr_c(khi, pa - 64u);
    CarryRow c;
    c.amount = (long long)((unsigned long long)sp.amt_max - fa);
    c.o_entry_d = (long long)((unsigned long long)sp.ent_min + fe);
    c.o_id = (int)((unsigned)sp.o_min + (unsigned)(fr & mask_c(bo)));
    c.o_d_id = (int)((unsigned)sp.d_min + (unsigned)(shr_c(fr, bo) & mask_c(bd)));
    c.o_w_id = (int)((unsigned)sp.w_min + (unsigned)shr_c(fr, bo + bd));
    c.o_ol_cnt = (int)((unsigned)sp.n_min + (unsigned)(lo & mask_c(bn)));
    c.c_id = (int)((unsigned)sp.ci_min + (unsigned)(shr_c(lo, bn) & mask_c(bci)));
    c.c_last = (int)((unsigned)sp.cl_min + (unsigned)(shr_c(lo, bn + bci) & mask_c((unsigned)sp.bits_cl)));
    return c;
}

constexpr int kMaxRun = 32;

__global__ void field_keys_kernel(const Q18Row *__restrict__ rows, const long long *__restrict__ amt,
                                  const unsigned int *__restrict__ vals, uint64_t n, int field,
                                  const Q18Plan *__restrict__ plan, unsigned long long *__restrict__ k) {
    const Q18SortSpec sp = plan->spec;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        const unsigned int x = vals[i];
        const Q18Row r = rows[x];
        switch (field) {  // 0 r, 1 e, 2 a; 3 o, 4 d, 5 w (r split per column when wide_r)
            case 0: k[i] = field_r(r, sp); break;
            case 1: k[i] = field_e(r, sp); break;
            case 2: k[i] = field_a(amt[x], sp); break;
            case 3: k[i] = (unsigned)(r.o_id - sp.o_min); break;
            case 4: k[i] = (unsigned)(r.o_d_id - sp.d_min); break;
            default: k[i] = (unsigned)(r.o_w_id - sp.w_min); break;
        }
    }
}

__global__ void iota_kernel(unsigned int *v, uint64_t n) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
        v[i] = (unsigned int)i;
}

// Gather one 32-byte row (one sector) per output position, write the SoA columns coalesced;
// amount_sum comes from the sorted prefix key (contiguous) instead of a second random gather.
__global__ void permute_kernel(const Q18Row *__restrict__ rows, const long long *__restrict__ amt,
                               const unsigned int *__restrict__ perm,
                               const unsigned long long *__restrict__ keys,
                               const Q18Plan *__restrict__ plan, Q18Cols dst) {
    const uint64_t n = plan->n;
    const Q18SortSpec sp = plan->spec;
    if (n <= 1) { perm = nullptr; keys = nullptr; }  // nothing was sorted
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    const int ashift = sp.prefix_bits - sp.bits_a;
    const uint64_t drop = l2_policy_evict_first();  // last read of the result rows
    for (uint64_t j = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; j < n; j += stride) {
        const unsigned int i = perm ? perm[j] : (unsigned int)j;
        Q18Row r;
        {
            unsigned long long *w64 = reinterpret_cast<unsigned long long *>(&r);
            ld16_policy(rows + i, w64[0], w64[1], drop);
            ld16_policy(reinterpret_cast<const char *>(rows + i) + 16, w64[2], w64[3], drop);
        }
        long long amount;
        if (keys) {
            const unsigned long long a = sp.bits_a ? (__ldcs(keys + j) >> ashift) : 0ull;
            amount = (long long)((unsigned long long)sp.amt_max - a);
        } else {
            amount = amt[i];
        }
        dst.c_last[j] = r.c_last;
        dst.c_id[j] = r.c_id;
        dst.o_id[j] = r.o_id;
        dst.o_entry_d[j] = r.o_entry_d;
        dst.o_ol_cnt[j] = r.o_ol_cnt;
        dst.amount_sum[j] = amount;
        dst.o_w_id[j] = r.o_w_id;
        dst.o_d_id[j] = r.o_d_id;
    }
}

__device__ __forceinline__ int bitwidth_dev(unsigned long long x) { return x ? 64 - __clzll(x) : 0; }

// The plan from the statistics: `n_spec` rows decide whether there is anything to order (one
// GPU: > 1 rows, the single-row case takes the row-id path; distributed: >= 1 row anywhere, the
// spec must be filled on every rank so that a lone row's carry record decodes).
__device__ Q18Plan make_q18_plan_vals(const Q18Stats &st, const Q18Zone &z, unsigned long long n_local,
                                      bool fill_spec, int bucket_bits, int allow_carry, unsigned int *flag) {
    Q18Plan p{};
    p.n = n_local;
    p.bucket_bits = bucket_bits;
    Q18SortSpec &sp = p.spec;
    if (fill_spec) {
        sp.amt_max = st.amt_max;
        sp.ent_min = st.ent_min;
        sp.w_min = z.w_min; sp.d_min = z.d_min; sp.o_min = z.o_min;
        sp.bits_w = bitwidth_dev((unsigned)z.w_max - (unsigned)z.w_min);
        sp.bits_d = bitwidth_dev((unsigned)z.d_max - (unsigned)z.d_min);
        sp.bits_o = bitwidth_dev((unsigned)z.o_max - (unsigned)z.o_min);
        sp.bits_a = bitwidth_dev((unsigned long long)st.amt_max - (unsigned long long)st.amt_min);
        sp.bits_e = bitwidth_dev((unsigned long long)st.ent_max - (unsigned long long)st.ent_min);
        // (the join-key domain, w < 2^23, d < 2^8, o >= 0, keeps this <= 62; guard anyway)
        sp.wide_r = sp.bits_w + sp.bits_d + sp.bits_o > 62;
        if (sp.wide_r && flag) atomicOr(flag, 4u);  // the engine redoes the ORDER BY per column
        sp.bits_r = sp.wide_r ? 62 : sp.bits_w + sp.bits_d + sp.bits_o;
        const int B = sp.bits_a + sp.bits_e + sp.bits_r;
        sp.prefix_bits = B <= 64 ? B : 64;
        sp.bits_low = B - sp.prefix_bits;
        sp.cl_min = z.cl_min; sp.ci_min = z.ci_min; sp.n_min = z.n_min;
        sp.bits_cl = bitwidth_dev((unsigned)z.cl_max - (unsigned)z.cl_min);
        sp.bits_ci = bitwidth_dev((unsigned)z.ci_max - (unsigned)z.ci_min);
        sp.bits_n = bitwidth_dev((unsigned)z.n_max - (unsigned)z.n_min);
        sp.carry = allow_carry && !sp.wide_r && sp.bits_low + sp.bits_cl + sp.bits_ci + sp.bits_n <= 64;
        p.tiefix = B > 64 && !sp.carry;  // carry records compare all key bits: no tie-fix
        p.shift = sp.prefix_bits > bucket_bits ? sp.prefix_bits - bucket_bits : 0;
    }
    return p;
}

__device__ Q18Plan make_q18_plan(const Q18Stats *__restrict__ stats, const Q18Zone &z,
                                 const unsigned long long *nout, int bucket_bits, int allow_carry,
                                 unsigned int *flag) {
    const unsigned long long n = *nout;
    return make_q18_plan_vals(*stats, z, n, n > 1, bucket_bits, allow_carry, flag);
}

// One thread: the ORDER BY plan from the HAVING statistics (amount_sum, o_entry_d) and the
// snapshot's zone maps (w, d, o; carry payload): widths of a, e, r, the prefix width, and
// whether the 128-bit carry record holds the whole row. (The v2 ORDER BY computes it inside
// its histogram kernel instead: one launch less.)
__global__ void q18_plan_kernel(const Q18Stats *__restrict__ stats, Q18Zone z,
                                const unsigned long long *nout, int bucket_bits, int allow_carry,
                                Q18Plan *plan, unsigned int *flag) {
    pdl_wait();
    pdl_trigger();
    *plan = make_q18_plan(stats, z, nout, bucket_bits, allow_carry, flag);
}

unsigned grid_cap(uint64_t work, int threads, int num_sms, int per_sm) {
    uint64_t want = (work + threads - 1) / threads;
    uint64_t cap = (uint64_t)num_sms * per_sm;
    if (want > cap) want = cap;
    return want ? (unsigned)want : 1u;
}

}  // namespace

void launch_q18_plan(const Q18Stats *stats, const Q18Zone &zone, const unsigned long long *nout,
                     int bucket_bits, bool allow_carry, Q18Plan *plan, unsigned int *flag,
                     cudaStream_t st) {
    launch_pdl(q18_plan_kernel, 1, 1, 0, st, stats, zone, nout, bucket_bits, allow_carry ? 1 : 0, plan, flag);
    count_launches(1);
}

int radix_sort_pairs(uint64_t n, int bits, const SortPairs &s, int num_sms, cudaStream_t st) {
    (void)num_sms;
    const uint64_t ntiles = sort_tiles(n);
    int cur = 0;
    for (int shift = 0; shift < bits; shift += 8) {
        hist_kernel<<<(unsigned)ntiles, kT, 0, st>>>(s.k[cur], n, shift, s.counts, ntiles);
        count_launches(1);
        digit_scan_kernel<<<256, 256, 0, st>>>(s.counts, ntiles, s.totals);
        count_launches(1);
        scatter_kernel<<<(unsigned)ntiles, kT, 0, st>>>(s.k[cur], s.v[cur], s.k[cur ^ 1], s.v[cur ^ 1],
                                                         n, shift, s.counts, ntiles, s.totals);
        count_launches(1);
        cur ^= 1;
    }
    return cur;
}

void launch_q18_field_keys(const Q18Row *rows, const long long *amt, const unsigned int *vals,
                           uint64_t n, int field, const Q18Plan *plan, unsigned long long *keys,
                           int num_sms, cudaStream_t st) {
    field_keys_kernel<<<grid_cap(n, 256, num_sms, 8), 256, 0, st>>>(rows, amt, vals, n, field, plan, keys);
    count_launches(1);
}

void launch_iota(unsigned int *v, uint64_t n, int num_sms, cudaStream_t st) {
    iota_kernel<<<grid_cap(n, 256, num_sms, 8), 256, 0, st>>>(v, n);
    count_launches(1);
}

void launch_q18_permute(const Q18Row *rows, const long long *amt, const unsigned int *perm,
                        const unsigned long long *keys, const Q18Plan *plan, uint64_t n_max,
                        const Q18Cols &dst, int num_sms, cudaStream_t st) {
    permute_kernel<<<grid_cap(n_max, 256, num_sms, 8), 256, 0, st>>>(rows, amt, perm, keys, plan, dst);
    count_launches(1);
}

}  // namespace h2tap

// ============================================================ bucket sort ===
// Main ORDER BY path, three kernels:
//  1. keys+hist: the 64-bit prefix key of every result row, the row id, a shared-memory
//     histogram of the top key bits; the last block to finish scans the bucket counts;
//  2. scatter: rows into buckets (per-block range reservation, shared cursors);
//  3. local sort + emit: each bucket in shared memory — second partition into ~8-row sub-buckets
//     and rank counting, then runs of equal prefixes ordered by the full tuple (tie-fix), then
//     the rows are gathered and written straight into the result columns at their final
//     positions (amount_sum decoded from the key).
// A bucket > 8192 rows or a tie run > 32 rows sets *flag; the engine then redoes the ORDER BY
// exactly with the LSD fallback above.
namespace h2tap {
namespace {

constexpr int kBkThreads = 256;
constexpr int kBkItems = 16;                       // rows per thread in the scatter
constexpr int kLsCapSmall = 2048;                  // rows per bucket: v1 small instance
constexpr int kLsCapLarge = 8192;                  // rows per bucket: large-bucket kernel
#ifndef LS_SUB_MAX
#define LS_SUB_MAX 512
#endif
constexpr int kLsSubMax = LS_SUB_MAX;              // max sub-buckets per bucket (4 per emit thread)
constexpr int kEmThreads = 128;                    // per-bucket sort / emit block (8 blocks/SM)

// 1. keys + histogram (+ bucket scan by the last block)
__global__ void __launch_bounds__(kBkThreads)
q18_keys_hist_kernel(const Q18Row *__restrict__ rows, const long long *__restrict__ amt,
                     const Q18Plan *__restrict__ plan, unsigned long long *__restrict__ k,
                     unsigned int *__restrict__ v, int nb, unsigned int *__restrict__ count,
                     unsigned int *__restrict__ offset, unsigned int *__restrict__ cursor,
                     unsigned int *ticket) {
    extern __shared__ unsigned int h[];
    __shared__ bool last;
    __shared__ unsigned int wsum[kBkThreads / 32];
    const uint64_t n = plan->n;
    const Q18SortSpec sp = plan->spec;
    const int shift = plan->shift;
    for (int i = threadIdx.x; i < nb; i += kBkThreads) h[i] = 0;
    __syncthreads();
    const uint64_t stride = (uint64_t)gridDim.x * kBkThreads;
    constexpr int U = 4;  // independent row loads in flight per thread
    for (uint64_t i0 = (uint64_t)blockIdx.x * kBkThreads + threadIdx.x; i0 < n; i0 += U * stride) {
        Q18Row r[U];
        long long a[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t i = i0 + u * stride;
            if (i < n) { r[u] = rows[i]; a[u] = amt[i]; }
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t i = i0 + u * stride;
            if (i >= n) break;
            const unsigned long long kk = prefix_key(r[u], a[u], sp);
            k[i] = kk;
            v[i] = (unsigned int)i;
            atomicAdd(&h[(unsigned int)(kk >> shift)], 1u);
        }
    }
    __syncthreads();
    for (int i = threadIdx.x; i < nb; i += kBkThreads)
        if (h[i]) atomicAdd(count + i, h[i]);
    __threadfence();
    __syncthreads();
    if (threadIdx.x == 0) last = atomicAdd(ticket, 1u) == gridDim.x - 1;
    __syncthreads();
    if (!last) return;
    __threadfence();
    // exclusive scan of the nb bucket counts: each thread owns nb/256 contiguous counts
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int per = (nb + kBkThreads - 1) / kBkThreads;
    const int b0 = threadIdx.x * per;
    unsigned int t = 0;
    for (int q = 0; q < per && b0 + q < nb; ++q) t += __ldcg(count + b0 + q);
    unsigned int x = t;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
        const unsigned int y = __shfl_up_sync(kFull, x, o);
        if (lane >= o) x += y;
    }
    if (lane == 31) wsum[warp] = x;
    __syncthreads();
    unsigned int run = x - t;
    for (int w = 0; w < warp; ++w) run += wsum[w];
    for (int q = 0; q < per && b0 + q < nb; ++q) {
        const unsigned int c = __ldcg(count + b0 + q);
        offset[b0 + q] = run;
        cursor[b0 + q] = run;
        run += c;
    }
    if (threadIdx.x == kBkThreads - 1) offset[nb] = run;
    if (threadIdx.x == 0) *ticket = 0;  // self-reset for the next launch
}

// 2. scatter into buckets: a block's shared histogram reserves one global range per bucket
__global__ void __launch_bounds__(kBkThreads)
bucket_scatter_kernel(const unsigned long long *__restrict__ kin, const unsigned int *__restrict__ vin,
                      unsigned long long *__restrict__ kout, unsigned int *__restrict__ vout,
                      const Q18Plan *__restrict__ plan, int nb, unsigned int *__restrict__ cursor) {
    const uint64_t n = plan->n;
    const int shift = plan->shift;
    if ((uint64_t)blockIdx.x * kBkThreads * kBkItems >= n) return;  // grid sized for an upper bound
    extern __shared__ unsigned int h[];  // [nb] local counts -> local cursors
    for (int i = threadIdx.x; i < nb; i += kBkThreads) h[i] = 0;
    const uint64_t base = (uint64_t)blockIdx.x * kBkThreads * kBkItems;
    unsigned long long kv[kBkItems];
    unsigned int b[kBkItems], val[kBkItems];
#pragma unroll
    for (int i = 0; i < kBkItems; ++i) {
        const uint64_t j = base + (uint64_t)i * kBkThreads + threadIdx.x;
        kv[i] = j < n ? __ldcs(kin + j) : 0ull;
        val[i] = j < n ? __ldcs(vin + j) : 0u;
        b[i] = j < n ? (unsigned int)(kv[i] >> shift) : 0xffffffffu;
    }
    __syncthreads();
#pragma unroll
    for (int i = 0; i < kBkItems; ++i)
        if (b[i] != 0xffffffffu) atomicAdd(&h[b[i]], 1u);
    __syncthreads();
#pragma unroll 8
    for (int i = threadIdx.x; i < nb; i += kBkThreads)  // independent atomics: keep 8 in flight
        if (h[i]) h[i] = atomicAdd(cursor + i, h[i]);  // base of this block's range in bucket i
    __syncthreads();
    unsigned int pos[kBkItems];
#pragma unroll
    for (int i = 0; i < kBkItems; ++i)
        pos[i] = b[i] != 0xffffffffu ? atomicAdd(&h[b[i]], 1u) : 0u;
#pragma unroll
    for (int i = 0; i < kBkItems; ++i) {
        if (b[i] == 0xffffffffu) continue;
        kout[pos[i]] = kv[i];
        vout[pos[i]] = val[i];
    }
}

template <int kLsCap> struct LsSmem {
    unsigned long long k1[kLsCap], k2[kLsCap];
    unsigned int v1[kLsCap], v2[kLsCap];
    unsigned int sub[kLsSubMax + 1];   // sub-bucket counts -> offsets
    unsigned int cur[kLsSubMax];       // sub-bucket cursors
    // 16-byte aligned on its own: the compiler reads wsum[] with one 128-bit shared load, which
    // from an unaligned start also covered the last cur[] entry — racecheck reported that benign
    // over-read as a read/write hazard against the scan's cur[] stores
    alignas(16) unsigned int wsum[kEmThreads / 32];
};

// carry mode: the records stay where they were loaded and the sort moves 16-bit record ids
// (1 536 rows: 35 KB, 6 blocks of 128 threads per SM)
template <int kCap, int kSub = kLsSubMax, int kT = kEmThreads> struct LcSmem {
    ulonglong2 rec[kCap];             // the bucket's records, load order
    unsigned short idx[kCap];         // record ids grouped by sub-bucket
    unsigned short srt[kCap];         // record ids in sorted order
    unsigned int sub[kSub + 1];
    unsigned int cur[kSub];
    // 16-byte aligned on its own: the compiler reads wsum[] with one 128-bit shared load, which
    // from an unaligned start also covered the last cur[] entry — racecheck reported that benign
    // over-read as a read/write hazard against the scan's cur[] stores
    alignas(16) unsigned int wsum[kT / 32];
};
static_assert(kLsCapLarge <= 65536, "16-bit record ids");
constexpr int kLcCapLarge = 8192;  // carry records per bucket in the large instance (~172 KB)

// Per-bucket sort of carry records (same sub-bucket + rank scheme as the row-id body below,
// 128-bit compares, no tie-fix) and the emit: every output column is decoded from the record,
// so the only global traffic is the bucket's records in and the result columns out. The next
// bucket's first kPre * 256 records are loaded into registers while the current one is
// decoded and stored, and its sub-bucket counters are cleared then too (one barrier less).
constexpr unsigned int kFlagHoles = 16u;    // direct ORDER BY: a counted row found no customer (the
                                            // host re-runs the v2 path; the emits skip their work)
constexpr int kPre = 3;
// kT threads per block, at most kSub sub-buckets per bucket (a power of two).
template <int kCap, int kMin, int kSub = kLsSubMax, int kT = kEmThreads>
__device__ __forceinline__ void carry_sort_emit(const ulonglong2 *__restrict__ kv,
                                                const unsigned int *__restrict__ offset, int nb,
                                                const Q18Plan *__restrict__ plan, const Q18Cols &dst,
                                                unsigned int *flag, unsigned int *big, unsigned char *smem,
                                                int sub_log2) {
    LcSmem<kCap, kSub, kT> &S = *reinterpret_cast<LcSmem<kCap, kSub, kT> *>(smem);
    constexpr int kQ = (kSub + kT - 1) / kT;  // sub-bucket counts scanned per thread
    constexpr int kSubBits = kSub >= 4096 ? 12 : kSub >= 2048 ? 11 : kSub >= 1024 ? 10 : 9;
    const int shift = plan->shift;
    const Q18SortSpec sp = plan->spec;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int nwork = kMin > 0 ? (int)*(volatile unsigned int *)big : nb;
    // bucket `wi` of this block: its range and the first kPre records of this thread
    unsigned int lo = 0, m = 0;
    ulonglong2 pre[kPre];
    auto fetch = [&](int wi) {
        lo = m = 0;
        if (wi >= nwork) return;
        const int b = kMin > 0 ? (int)big[1 + wi] : wi;
        lo = offset[b];
        m = offset[b + 1] - lo;
        if (m == 0) return;
        if (m > (unsigned)kCap) {
            if (threadIdx.x == 0) {
                if (kMin > 0) atomicOr(flag, 2u);                 // too big even for shared memory
                else big[1 + atomicAdd(big, 1u)] = (unsigned)b;   // hand over to the large instance
            }
            m = 0;
            return;
        }
#pragma unroll
        for (int u = 0; u < kPre; ++u) {
            const unsigned int i = threadIdx.x + u * kT;
            if (i < m) pre[u] = __ldcg(kv + lo + i);
        }
    };
    for (unsigned int i = threadIdx.x; i <= kSub; i += kT) S.sub[i] = 0;
    fetch(blockIdx.x);
    __syncthreads();
    for (int wi = blockIdx.x; wi < nwork; wi += gridDim.x) {
        if (m == 0) {  // empty or handed over (uniform across the block)
            fetch(wi + gridDim.x);
            continue;
        }
        // sub-bucket bits: the smallest sb with (m >> (sb + sub_log2)) == 0, at most 10
        int sb = 32 - __clz(m) - sub_log2;
        sb = sb < 0 ? 0 : sb > kSubBits ? kSubBits : sb;  // ns <= kSub
        if (sb > shift) sb = shift;
        const int ssh = shift - sb;
        const unsigned int ns = 1u << sb, smask = ns - 1u;
#pragma unroll
        for (int u = 0; u < kPre; ++u) {
            const unsigned int i = threadIdx.x + u * kT;
            if (i < m) {
                S.rec[i] = pre[u];
                atomicAdd(&S.sub[(unsigned int)(pre[u].x >> ssh) & smask], 1u);
            }
        }
        for (unsigned int i = threadIdx.x + kPre * kT; i < m; i += kT) {  // rest
            const ulonglong2 r = __ldcg(kv + lo + i);
            S.rec[i] = r;
            atomicAdd(&S.sub[(unsigned int)(r.x >> ssh) & smask], 1u);
        }
        __syncthreads();
        {   // exclusive scan of ns (<= kSub) sub-bucket counts: kQ per thread
            unsigned int c[kQ], t = 0;
#pragma unroll
            for (int q = 0; q < kQ; ++q) {
                const unsigned int i = threadIdx.x * kQ + q;
                c[q] = i < ns ? S.sub[i] : 0u;
                t += c[q];
            }
            unsigned int x = t;
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                const unsigned int y = __shfl_up_sync(kFull, x, o);
                if (lane >= o) x += y;
            }
            if (lane == 31) S.wsum[warp] = x;
            __syncthreads();
            unsigned int before = 0;
            for (int w = 0; w < warp; ++w) before += S.wsum[w];
            unsigned int run = before + x - t;
#pragma unroll
            for (int q = 0; q < kQ; ++q) {
                const unsigned int i = threadIdx.x * kQ + q;
                if (i < ns) { S.sub[i] = run; S.cur[i] = run; }
                run += c[q];
            }
            if (threadIdx.x == kT - 1) S.sub[ns] = run;
        }
        __syncthreads();
        for (unsigned int i = threadIdx.x; i < m; i += kT) {
            const unsigned long long kk = S.rec[i].x;
            const unsigned int p = atomicAdd(&S.cur[(unsigned int)(kk >> ssh) & smask], 1u);
            H2TAP_CHECK(p < m);
            S.idx[p] = (unsigned short)i;
        }
        __syncthreads();
        for (unsigned int i = threadIdx.x; i < m; i += kT) {  // rank -> sorted order
            const unsigned int me = S.idx[i];
            const ulonglong2 r = S.rec[me];
            const unsigned int sbk = (unsigned int)(r.x >> ssh) & smask;
            const unsigned int s0 = S.sub[sbk], s1 = S.sub[sbk + 1];
            unsigned int rank = s0;
            if (s1 - s0 > 1) {  // (a sub-bucket of one row: its rank is its offset)
                for (unsigned int j = s0; j < s1; ++j) {
                    const ulonglong2 o = S.rec[S.idx[j]];
                    rank += (o.x < r.x) | ((o.x == r.x) & ((o.y < r.y) | ((o.y == r.y) & (j < i))));
                }
            }
            H2TAP_CHECK(rank < m && me < m);
            S.srt[rank] = (unsigned short)me;
        }
        __syncthreads();
        const unsigned int cur_lo = lo, cur_m = m;
        fetch(wi + gridDim.x);  // next bucket's records in flight during the stores below
        for (unsigned int i = threadIdx.x; i <= ns; i += kT) S.sub[i] = 0;
        // decode + coalesced stores, two adjacent output rows per thread (8-byte stores of the
        // int32 columns, 16-byte of the int64 ones); an odd first / last row goes alone
        auto store1 = [&](unsigned int i) {
            const ulonglong2 r = S.rec[S.srt[i]];
            const CarryRow c = carry_decode(r.x, r.y, sp);
            const uint64_t j = cur_lo + i;
            dst.c_last[j] = c.c_last;
            dst.c_id[j] = c.c_id;
            dst.o_id[j] = c.o_id;
            dst.o_entry_d[j] = c.o_entry_d;
            dst.o_ol_cnt[j] = c.o_ol_cnt;
            dst.amount_sum[j] = c.amount;
            dst.o_w_id[j] = c.o_w_id;
            dst.o_d_id[j] = c.o_d_id;
        };
        const unsigned int head = cur_lo & 1u;  // output row cur_lo + i is even for i = head
        const unsigned int npair = (cur_m - head) >> 1;
        for (unsigned int p = threadIdx.x; p < npair; p += kT) {
            const unsigned int i = head + 2 * p;
            const ulonglong2 ra = S.rec[S.srt[i]], rb = S.rec[S.srt[i + 1]];
            const CarryRow a = carry_decode(ra.x, ra.y, sp);
            const CarryRow b = carry_decode(rb.x, rb.y, sp);
            const uint64_t j = cur_lo + i;
            *reinterpret_cast<int2 *>(dst.c_last + j) = make_int2(a.c_last, b.c_last);
            *reinterpret_cast<int2 *>(dst.c_id + j) = make_int2(a.c_id, b.c_id);
            *reinterpret_cast<int2 *>(dst.o_id + j) = make_int2(a.o_id, b.o_id);
            *reinterpret_cast<longlong2 *>(dst.o_entry_d + j) = make_longlong2(a.o_entry_d, b.o_entry_d);
            *reinterpret_cast<int2 *>(dst.o_ol_cnt + j) = make_int2(a.o_ol_cnt, b.o_ol_cnt);
            *reinterpret_cast<longlong2 *>(dst.amount_sum + j) = make_longlong2(a.amount, b.amount);
            *reinterpret_cast<int2 *>(dst.o_w_id + j) = make_int2(a.o_w_id, b.o_w_id);
            *reinterpret_cast<int2 *>(dst.o_d_id + j) = make_int2(a.o_d_id, b.o_d_id);
        }
        if (threadIdx.x == kT - 1 && head) store1(0);
        if (threadIdx.x == kT - 2 && ((cur_m - head) & 1u)) store1(cur_m - 1);
        __syncthreads();
    }
}

// 3. One block per bucket: partition by the next `sb` key bits into sub-buckets, rank every row
// inside its sub-bucket, order equal-prefix runs by the full tuple, and write the result columns
// at their final positions. The small instance walks every bucket and queues buckets above its
// capacity in big[1..]; the large instance walks only that queue.
// kPairs: k holds interleaved 16-byte (key, row id) pairs (v2 scatter), v is unused.
template <int kLsCap, int kMin, bool kPairs = false>
__global__ void __launch_bounds__(kEmThreads, EMIT_BPS)
bucket_local_emit_kernel(const unsigned long long *__restrict__ k, const unsigned int *__restrict__ v,
                         const unsigned int *__restrict__ offset, int nb,
                         const Q18Plan *__restrict__ plan, const Q18Row *__restrict__ rows,
                         const long long *__restrict__ amt, Q18Cols dst, unsigned int *flag,
                         unsigned int *big, int sub_log2 = 3, PeerArgs pa = PeerArgs{}) {
    pdl_wait();
    pdl_trigger();
    if (flag && (*reinterpret_cast<volatile unsigned int *>(flag) & kFlagHoles)) return;  // re-run on v2
    extern __shared__ __align__(16) unsigned char smem_raw[];
    if (pa.world > 1) {  // distributed ORDER BY: this rank's buckets, exchanged into its heap
        // (their arrival was awaited by the one-thread peer_wait launched before this grid)
        const unsigned long long xs = plan->xseq;
        if (plan->err & (kPeerErrHeap | kPeerErrOutCap | kPeerErrNoCarry | kPeerErrTimeout)) return;
        k = reinterpret_cast<const unsigned long long *>(peer::heap(pa, pa.rank, (int)(xs & 1)));
        nb = (int)plan->nb_mine;  // offset = the receive offsets of those buckets
    }
    if (kPairs && plan->spec.carry) {  // uniform: the whole ORDER BY runs on carry records
        carry_sort_emit<(kMin > 0 ? kLcCapLarge : kLsCap), kMin>(
            reinterpret_cast<const ulonglong2 *>(k), offset, nb, plan, dst, flag, big, smem_raw, sub_log2);
        return;
    }
    // row-id path: the v2 small instance holds 1 024 rows (LsSmem<1024> fits the 35 KB of the
    // carry layout, so both run 6 blocks per SM); larger buckets go to the large instance
    if (rows == nullptr) return;  // v3 / distributed: carry records only (row path re-run by the host)
    constexpr int kRowCap = (kPairs && kMin == 0) ? ROW_CAP : kLsCap;
    LsSmem<kRowCap> &S = *reinterpret_cast<LsSmem<kRowCap> *>(smem_raw);
    const int shift = plan->shift;
    const Q18SortSpec sp = plan->spec;
    const bool tiefix = plan->tiefix != 0;
    const int ashift = sp.prefix_bits - sp.bits_a;
    const uint64_t drop = l2_policy_evict_first();  // last read of the result rows
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int nwork = kMin > 0 ? (int)*(volatile unsigned int *)big : nb;
    for (int wi = blockIdx.x; wi < nwork; wi += gridDim.x) {
        const int b = kMin > 0 ? (int)big[1 + wi] : wi;
        const unsigned int lo = offset[b], m = offset[b + 1] - lo;
        if (m == 0) continue;
        if (m > (unsigned)kRowCap) {
            if (threadIdx.x == 0) {
                if (kMin > 0) atomicOr(flag, 2u);                 // too big even for shared memory
                else big[1 + atomicAdd(big, 1u)] = (unsigned)b;   // hand over to the large instance
            }
            continue;
        }
        if (m == 1) {
            if (threadIdx.x == 0) {
                if (kPairs) { S.k1[0] = k[2ull * lo]; S.v1[0] = (unsigned int)k[2ull * lo + 1]; }
                else { S.k1[0] = k[lo]; S.v1[0] = v[lo]; }
            }
        } else {
            // sub-bucket bits: ~8 rows per sub-bucket, at most kLsSubMax sub-buckets
            int sb = 0;
            while (sb < 9 && (m >> (sb + 3)) > 0) ++sb;
            if (sb > shift) sb = shift;
            const int ssh = shift - sb;
            const unsigned int ns = 1u << sb, smask = ns - 1u;
            for (unsigned int i = threadIdx.x; i < ns; i += kEmThreads) S.sub[i] = 0;
            __syncthreads();
            for (unsigned int i0 = threadIdx.x; i0 < m; i0 += 2 * kEmThreads) {  // 2 loads in flight
                unsigned long long kk[2];
                unsigned int vv[2];
#pragma unroll
                for (int u = 0; u < 2; ++u) {
                    const unsigned int i = i0 + u * kEmThreads;
                    if (i < m) {
                        if (kPairs) {
                            const ulonglong2 kv = __ldcs(reinterpret_cast<const ulonglong2 *>(k) + lo + i);
                            kk[u] = kv.x;
                            vv[u] = (unsigned int)kv.y;
                        } else {
                            kk[u] = __ldcs(k + lo + i);
                            vv[u] = __ldcs(v + lo + i);
                        }
                    }
                }
#pragma unroll
                for (int u = 0; u < 2; ++u) {
                    const unsigned int i = i0 + u * kEmThreads;
                    if (i >= m) break;
                    S.k1[i] = kk[u];
                    S.v1[i] = vv[u];
                    atomicAdd(&S.sub[(unsigned int)(kk[u] >> ssh) & smask], 1u);
                }
            }
            __syncthreads();
            {   // exclusive scan of ns (<= 1024) sub-bucket counts: 4 per thread
                unsigned int c[4], t = 0;
#pragma unroll
                for (int q = 0; q < 4; ++q) {
                    const unsigned int i = threadIdx.x * 4 + q;
                    c[q] = i < ns ? S.sub[i] : 0u;
                    t += c[q];
                }
                unsigned int x = t;
#pragma unroll
                for (int o = 1; o < 32; o <<= 1) {
                    const unsigned int y = __shfl_up_sync(kFull, x, o);
                    if (lane >= o) x += y;
                }
                if (lane == 31) S.wsum[warp] = x;
                __syncthreads();
                unsigned int before = 0;
                for (int w = 0; w < warp; ++w) before += S.wsum[w];
                unsigned int run = before + x - t;
#pragma unroll
                for (int q = 0; q < 4; ++q) {
                    const unsigned int i = threadIdx.x * 4 + q;
                    if (i < ns) { S.sub[i] = run; S.cur[i] = run; }
                    run += c[q];
                }
                if (threadIdx.x == kEmThreads - 1) S.sub[ns] = run;
            }
            __syncthreads();
            for (unsigned int i = threadIdx.x; i < m; i += kEmThreads) {
                const unsigned long long kk = S.k1[i];
                const unsigned int p = atomicAdd(&S.cur[(unsigned int)(kk >> ssh) & smask], 1u);
                S.k2[p] = kk;
                S.v2[p] = S.v1[i];
            }
            __syncthreads();
            for (unsigned int i = threadIdx.x; i < m; i += kEmThreads) {  // rank -> sorted smem
                const unsigned long long kk = S.k2[i];
                const unsigned int sbk = (unsigned int)(kk >> ssh) & smask;
                const unsigned int s0 = S.sub[sbk], s1 = S.sub[sbk + 1];
                unsigned int rank = s0;
                for (unsigned int j = s0; j < s1; ++j) {
                    const unsigned long long kj = S.k2[j];
                    rank += (kj < kk) | ((kj == kk) & (j < i));
                }
                S.k1[rank] = kk;
                S.v1[rank] = S.v2[i];
            }
            __syncthreads();
            if (tiefix) {  // runs of equal 64-bit prefixes never cross buckets
                for (unsigned int i = threadIdx.x; i < m; i += kEmThreads) {
                    const unsigned long long ki = S.k1[i];
                    if (i > 0 && S.k1[i - 1] == ki) continue;          // not a run head
                    if (i + 1 >= m || S.k1[i + 1] != ki) continue;     // run of one
                    unsigned int j = i + 1;
                    while (j < m && S.k1[j] == ki && j - i <= (unsigned)kMaxRun) ++j;
                    if (j - i > (unsigned)kMaxRun) { atomicOr(flag, 1u); continue; }
                    for (unsigned int t = i + 1; t < j; ++t) {  // insertion sort by the full tuple
                        const unsigned int x = S.v1[t];
                        const Q18Row rx = rows[x];
                        const long long ax = amt[x];
                        int u = (int)t - 1;
                        while (u >= (int)i && row_less(rx, ax, rows[S.v1[u]], amt[S.v1[u]])) {
                            S.v1[u + 1] = S.v1[u];
                            --u;
                        }
                        S.v1[u + 1] = x;
                    }
                }
                __syncthreads();
            }
        }
        __syncthreads();
        for (unsigned int i0 = threadIdx.x; i0 < m; i0 += 2 * kEmThreads) {  // emit: 2 gathers in flight
            Q18Row row[2];
#pragma unroll
            for (int u = 0; u < 2; ++u) {
                const unsigned int i = i0 + u * kEmThreads;
                if (i < m) {
                    const unsigned int r = S.v1[i];
                    unsigned long long *w64 = reinterpret_cast<unsigned long long *>(&row[u]);
                    ld16_policy(rows + r, w64[0], w64[1], drop);
                    ld16_policy(reinterpret_cast<const char *>(rows + r) + 16, w64[2], w64[3], drop);
                }
            }
#pragma unroll
            for (int u = 0; u < 2; ++u) {
                const unsigned int i = i0 + u * kEmThreads;
                if (i >= m) break;
                const unsigned long long a = sp.bits_a ? (S.k1[i] >> ashift) : 0ull;
                const uint64_t j = lo + i;
                dst.c_last[j] = row[u].c_last;
                dst.c_id[j] = row[u].c_id;
                dst.o_id[j] = row[u].o_id;
                dst.o_entry_d[j] = row[u].o_entry_d;
                dst.o_ol_cnt[j] = row[u].o_ol_cnt;
                dst.amount_sum[j] = m == 1 && plan->n <= 1 ? amt[S.v1[i]]
                                                           : (long long)((unsigned long long)sp.amt_max - a);
                dst.o_w_id[j] = row[u].o_w_id;
                dst.o_d_id[j] = row[u].o_d_id;
            }
        }
        __syncthreads();
    }
}

// Buckets above the small instance's capacity, carry records only (v3 / distributed): 512 threads
// and up to 4 096 sub-buckets per 8 192-record bucket in one 192 KB block per SM (the 128-thread
// instance left 4 warps per SM for exactly the buckets that need the most work).
constexpr int kLgThreads = 512;
constexpr int kLgSub = 4096;
constexpr size_t kLgSmem = sizeof(LcSmem<kLcCapLarge, kLgSub, kLgThreads>);
__global__ void __launch_bounds__(kLgThreads, 1)
carry_large_emit_kernel(const unsigned long long *__restrict__ k, const unsigned int *__restrict__ offset, int nb,
                        const Q18Plan *__restrict__ plan, Q18Cols dst, unsigned int *flag, unsigned int *big,
                        int sub_log2, PeerArgs pa) {
    pdl_wait();
    pdl_trigger();
    if (flag && (*reinterpret_cast<volatile unsigned int *>(flag) & kFlagHoles)) return;  // re-run on v2
    extern __shared__ __align__(16) unsigned char smem_raw[];
    if (pa.world > 1) {  // distributed ORDER BY: this rank's buckets in its heap (as the emit above)
        const unsigned long long xs = plan->xseq;
        if (plan->err & (kPeerErrHeap | kPeerErrOutCap | kPeerErrNoCarry | kPeerErrTimeout)) return;
        k = reinterpret_cast<const unsigned long long *>(peer::heap(pa, pa.rank, (int)(xs & 1)));
        nb = (int)plan->nb_mine;
    }
    if (!plan->spec.carry) return;
    carry_sort_emit<kLcCapLarge, 1, kLgSub, kLgThreads>(reinterpret_cast<const ulonglong2 *>(k), offset, nb, plan,
                                                      dst, flag, big, smem_raw, sub_log2);
}

// ============================================== bucket sort v2 (default) ===
// The v1 path above spends most of its time in global atomics (the histogram flush and the
// per-block range reservation: ~one per row each) and in one shared-memory sort per ~360-row
// bucket (eight block barriers per bucket, latency-bound). v2:
//  1. ob_hist:    block b owns rows [b*T, (b+1)*T); shared histogram of the bucket ids (only
//                 amount_sum is read when the bucket bits lie inside field a) -> matrix row b;
//  2. ob_scan:    per bucket, exclusive scan down the [G][nb] matrix column (staged through
//                 shared memory); the last block scans the bucket totals into bucket offsets;
//  3. ob_scatter: block b seeds shared cursors with offset[j] + matrix[b][j] — no global atomics —
//                 recomputes every key from the row and writes the 16-byte (key, row id) pair at
//                 its position (one scattered store per row);
//  4. v1's per-bucket shared-memory sort + tie-fix + emit on the (key, row id) pairs.
// Measured and rejected: carrying the 32-byte rows through the scatter (the
// scattered 40 B/row writes cost more than the random gather they save) and sorting chunks of
// whole buckets per block (fewer barriers, but 2 blocks/SM left the gathers latency-bound).
constexpr int kObThreads = 1024;   // hist / scatter: 2 blocks of 32 warps per SM
constexpr int kObCap = OB_CAP;  // per-bucket sort capacity (carry: 35 KB, 6 blocks of 128 threads/SM);
                                     // 4 096 (2 blocks/SM) with ~730-row buckets measured slower
// dynamic shared memory of the v2 emit instances: row-id or carry layout, whichever is larger
constexpr size_t kObSmem = sizeof(LsSmem<ROW_CAP>) > sizeof(LcSmem<kObCap>) ? sizeof(LsSmem<ROW_CAP>)
                                                                            : sizeof(LcSmem<kObCap>);
constexpr size_t kObSmemLarge = sizeof(LsSmem<kLsCapLarge>) > sizeof(LcSmem<kLcCapLarge>)
                                    ? sizeof(LsSmem<kLsCapLarge>) : sizeof(LcSmem<kLcCapLarge>);

__device__ __forceinline__ unsigned int ob_bucket(const Q18Row *rows, const long long *amt, uint64_t i,
                                                  const Q18SortSpec &sp, int shift, bool amt_only) {
    if (amt_only) {  // the bucket bits are the top bits of field a
        const unsigned long long a = field_a(amt[i], sp);
        return (unsigned int)(a >> (shift - (sp.prefix_bits - sp.bits_a)));
    }
    return (unsigned int)(prefix_key(rows[i], amt[i], sp) >> shift);
}

__device__ __forceinline__ void ob_range(uint64_t n, uint64_t &r0, uint64_t &r1) {
    const uint64_t T = (n + gridDim.x - 1) / gridDim.x;
    r0 = (uint64_t)blockIdx.x * T;
    r1 = r0 + T < n ? r0 + T : n;
    if (r0 > n) r0 = n;
}

__global__ void __launch_bounds__(kObThreads)
ob_hist_kernel(const Q18Row *__restrict__ rows, const long long *__restrict__ amt,
               Q18Plan *__restrict__ plan, int nb, unsigned int *__restrict__ mat,
               unsigned int *__restrict__ big, int make_plan, Q18PlanArgs pa, int bucket_bits,
               unsigned int *flag) {
    pdl_wait();
    pdl_trigger();
    extern __shared__ unsigned int h[];
    __shared__ Q18Plan P;
    if (blockIdx.x == 0 && threadIdx.x == 0) *big = 0;  // work-list count of the emit kernels
    if (make_plan) {  // every block derives the plan (a few dozen instructions); block 0 stores it
        if (threadIdx.x == 0) {
            P = make_q18_plan(pa.stats, pa.zone, pa.nout, bucket_bits, pa.allow_carry,
                              blockIdx.x == 0 ? flag : nullptr);
            if (blockIdx.x == 0) *plan = P;
        }
    } else if (threadIdx.x == 0) {
        P = *plan;
    }
    __syncthreads();
    const uint64_t n = P.n;
    const Q18SortSpec sp = P.spec;
    const int shift = P.shift;
    if (P.dist) nb = 1 << P.bucket_bits;  // distributed: from the global row count (<= launch nb)
    const bool amt_only = sp.bits_a > 0 && shift >= sp.prefix_bits - sp.bits_a;
    for (int i = threadIdx.x; i < nb; i += kObThreads) h[i] = 0;
    __syncthreads();
    uint64_t r0, r1;
    ob_range(n, r0, r1);
    constexpr int U = 8;
    for (uint64_t i0 = r0 + threadIdx.x; i0 < r1; i0 += U * kObThreads) {
        unsigned int b[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t i = i0 + (uint64_t)u * kObThreads;
            b[u] = i < r1 ? ob_bucket(rows, amt, i, sp, shift, amt_only) : 0xffffffffu;
        }
#pragma unroll
        for (int u = 0; u < U; ++u)
            if (b[u] != 0xffffffffu) atomicAdd(&h[b[u]], 1u);
    }
    __syncthreads();
    unsigned int *row = mat + (uint64_t)blockIdx.x * nb;
    for (int i = threadIdx.x; i < nb; i += kObThreads) row[i] = h[i];
}

// Column scans of the [G][nb] matrix: a block owns 32 buckets (lane); the [G][32] tile is staged
// in shared memory with independent coalesced loads, scanned per column, written back. The last
// block scans the bucket totals into bucket offsets.
constexpr int kScanWarps = 32;
__global__ void __launch_bounds__(32 * kScanWarps)
ob_scan_kernel(unsigned int *__restrict__ mat, int G, int nb, unsigned int *__restrict__ count,
               unsigned int *__restrict__ offset, unsigned int *ticket, const Q18Plan *__restrict__ plan,
               ulonglong2 *__restrict__ touch = nullptr, uint64_t touch_n = 0) {
    pdl_wait();
    pdl_trigger();
    const unsigned nscan = (unsigned)(nb + 31) / 32;  // the column-scan blocks (launch nb)
    if (plan && plan->dist) nb = 1 << plan->bucket_bits;  // (grid sized for the launch nb)
    if (blockIdx.x >= nscan) {  // v3: blocks past the scan write the scatter's target lines into
        // L2 (evict_last) while the latency-bound scan runs on the first nscan blocks
        const uint64_t keep = l2_policy_evict_last();
        const uint64_t stride = (uint64_t)(gridDim.x - nscan) * blockDim.x;
        for (uint64_t i = (uint64_t)(blockIdx.x - nscan) * blockDim.x + threadIdx.x; i < touch_n; i += stride)
            st16_policy(touch + i, 0ull, 0ull, keep);
        return;
    }
    extern __shared__ unsigned int tile[];  // [G][32]; the last block reuses it for nb totals
    __shared__ bool last;
    __shared__ unsigned int tot[kScanWarps][32];
    __shared__ unsigned int wsum[kScanWarps];
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int j = blockIdx.x * 32 + lane;
#pragma unroll 8
    for (int b = warp; b < G; b += kScanWarps) tile[b * 32 + lane] = j < nb ? __ldcs(mat + (uint64_t)b * nb + j) : 0u;
    __syncthreads();
    const int C = (G + kScanWarps - 1) / kScanWarps;
    const int b0 = warp * C, b1 = min(G, b0 + C);
    unsigned int sum = 0;
    for (int b = b0; b < b1; ++b) sum += tile[b * 32 + lane];
    tot[warp][lane] = sum;
    __syncthreads();
    unsigned int run = 0;
    for (int w = 0; w < warp; ++w) run += tot[w][lane];
    if (warp == kScanWarps - 1 && j < nb) count[j] = run + sum;
    for (int b = b0; b < b1; ++b) {
        const unsigned int c = tile[b * 32 + lane];
        tile[b * 32 + lane] = run;
        run += c;
    }
    __syncthreads();
    if (j < nb) {
#pragma unroll 8
        for (int b = warp; b < G; b += kScanWarps) mat[(uint64_t)b * nb + j] = tile[b * 32 + lane];
    }
    __threadfence();
    __syncthreads();
    if (threadIdx.x == 0) last = atomicAdd(ticket, 1u) == nscan - 1;
    __syncthreads();
    if (!last) return;
    __threadfence();
    // last block: stage the bucket totals in shared memory (all loads independent, many in
    // flight), then an exclusive scan, warp-cooperatively (lane i reads element base + i: no bank
    // conflicts), each warp over a contiguous range
    unsigned int *sc = tile;  // reuse: nb entries (dynamic smem >= 4 * nb)
#pragma unroll 8
    for (int i = threadIdx.x; i < nb; i += 32 * kScanWarps) sc[i] = __ldcg(count + i);
    __syncthreads();
    const int span = (nb + kScanWarps - 1) / kScanWarps;
    const int w0 = warp * span, w1 = min(nb, w0 + span);
    unsigned int wtot = 0;
    for (int base = w0; base < w1; base += 32) {
        const int i = base + lane;
        wtot += __reduce_add_sync(kFull, i < w1 ? sc[i] : 0u);
    }
    if (lane == 0) wsum[warp] = wtot;
    __syncthreads();
    unsigned int acc = 0;
    for (int w = 0; w < warp; ++w) acc += wsum[w];
    for (int base = w0; base < w1; base += 32) {
        const int i = base + lane;
        const unsigned int c = i < w1 ? sc[i] : 0u;
        unsigned int x = c;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const unsigned int y = __shfl_up_sync(kFull, x, o);
            if (lane >= o) x += y;
        }
        if (i < w1) offset[i] = acc + x - c;
        acc += __shfl_sync(kFull, x, 31);
    }
    if (warp == kScanWarps - 1 && lane == 0) offset[nb] = acc;
    if (threadIdx.x == 0) *ticket = 0;  // self-reset
}

__global__ void __launch_bounds__(kObThreads)
ob_scatter_kernel(const Q18Row *__restrict__ rows, const long long *__restrict__ amt,
                  const Q18Plan *__restrict__ plan, int nb, const unsigned int *__restrict__ mat,
                  const unsigned int *__restrict__ offset, unsigned long long *__restrict__ kvout) {
    pdl_wait();
    pdl_trigger();
    extern __shared__ unsigned int cur[];
    const uint64_t n = plan->n;
    const Q18SortSpec sp = plan->spec;
    const int shift = plan->shift;
    if (plan->dist) nb = 1 << plan->bucket_bits;
    const unsigned int *row = mat + (uint64_t)blockIdx.x * nb;
    for (int i = threadIdx.x; i < nb; i += kObThreads) cur[i] = offset[i] + row[i];
    __syncthreads();
    uint64_t r0, r1;
    ob_range(n, r0, r1);
    constexpr int U = 4;
    for (uint64_t i0 = r0 + threadIdx.x; i0 < r1; i0 += U * kObThreads) {
        Q18Row r[U];
        long long a[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t i = i0 + (uint64_t)u * kObThreads;
            if (i < r1) {
                const ulonglong2 *src = reinterpret_cast<const ulonglong2 *>(rows + i);
                ulonglong2 *d = reinterpret_cast<ulonglong2 *>(&r[u]);
                d[0] = src[0];  // (rows stay cached: the emit gathers them again)
                d[1] = src[1];
                a[u] = __ldcs(amt + i);
            }
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t i = i0 + (uint64_t)u * kObThreads;
            if (i >= r1) break;
            const ulonglong2 rec = sp.carry ? carry_record(r[u], a[u], sp)
                                            : make_ulonglong2(prefix_key(r[u], a[u], sp), (unsigned long long)i);
            const unsigned int p = atomicAdd(&cur[(unsigned int)(rec.x >> shift)], 1u);
            reinterpret_cast<ulonglong2 *>(kvout)[p] = rec;
        }
    }
}

}  // namespace

void q18_bucket_order(const Q18Row *rows, const long long *amt, const Q18Plan *plan, uint64_t n_max,
                      int bucket_bits, const BucketSort &s, const Q18Cols &dst, unsigned int *flag,
                      int num_sms, cudaStream_t st, PhaseMarks *marks) {
    auto begin = [&](const char *nm) { if (marks) marks->begin(nm); };
    auto end = [&] { if (marks) marks->end(); };
    if (bucket_bits > kBucketMaxBits) bucket_bits = kBucketMaxBits;
    const int nb = 1 << bucket_bits;
    cudaMemsetAsync(s.count, 0, sizeof(unsigned int) * (nb + 1), st);
    cudaMemsetAsync(s.big, 0, sizeof(unsigned int), st);
    const uint64_t n1 = n_max ? n_max : 1;
    uint64_t hb = (n1 + kBkThreads * 8 - 1) / (kBkThreads * 8);
    if (hb > (uint64_t)num_sms * 4) hb = (uint64_t)num_sms * 4;
    begin("q18_sort_keys_hist");
    q18_keys_hist_kernel<<<(unsigned)hb, kBkThreads, nb * 4, st>>>(rows, amt, plan, s.k[0], s.v[0], nb,
                                                                  s.count, s.offset, s.cursor, s.ticket);
    count_launches(1);
    end();
    begin("q18_bucket_scatter");
    const uint64_t per = (uint64_t)kBkThreads * kBkItems;
    const uint64_t sb = (n1 + per - 1) / per;
    bucket_scatter_kernel<<<(unsigned)sb, kBkThreads, nb * 4, st>>>(s.k[0], s.v[0], s.k[1], s.v[1], plan,
                                                                   nb, s.cursor);
    count_launches(1);
    end();
    begin("q18_bucket_sort_emit");
    unsigned lb = (unsigned)nb < (unsigned)num_sms * 3 ? (unsigned)nb : (unsigned)num_sms * 3;
    bucket_local_emit_kernel<kLsCapSmall, 0><<<lb, kEmThreads, sizeof(LsSmem<kLsCapSmall>), st>>>(
        s.k[1], s.v[1], s.offset, nb, plan, rows, amt, dst, flag, s.big);
    count_launches(1);
    end();
    // buckets above the small capacity (skewed keys): one block per SM, ~200 KB shared memory
    begin("q18_bucket_sort_emit_large");
    bucket_local_emit_kernel<kLsCapLarge, kLsCapSmall><<<(unsigned)num_sms, kEmThreads,
                                                          sizeof(LsSmem<kLsCapLarge>), st>>>(
        s.k[1], s.v[1], s.offset, nb, plan, rows, amt, dst, flag, s.big);
    count_launches(1);
    end();
}

}  // namespace h2tap

namespace h2tap {

int ob_grid(int num_sms) {  // row partitions of the v2 ORDER BY front (H2TAP_OB_PER_SM, 1..2)
    static const int per = [] {
        const char *v = std::getenv("H2TAP_OB_PER_SM");
        return v ? std::max(1, std::min(2, std::atoi(v))) : 2;
    }();
    return per * num_sms;
}
int ob_bucket_bits(uint64_t n_max) {  // ~256-512 rows per bucket
    int bb = 1;
    while (bb < kBucketMaxBits && (n_max >> (bb + 9)) > 0) ++bb;
    return bb;
}

void q18_bucket_order_v2(const Q18Row *rows, const long long *amt, Q18Plan *plan, uint64_t n_max,
                         int bucket_bits, const BucketSort &s, const Q18Cols &dst, unsigned int *flag,
                         int num_sms, cudaStream_t st, PhaseMarks *marks, const Q18PlanArgs *plan_args) {
    auto begin = [&](const char *nm) { if (marks) marks->begin(nm); };
    auto end = [&] { if (marks) marks->end(); };
    if (bucket_bits > kBucketMaxBits) bucket_bits = kBucketMaxBits;
    const int nb = 1 << bucket_bits;
    const int G = ob_grid(num_sms);
    (void)n_max;
    // carry sort: ~2^sub_log2 rows per sub-bucket (rank loop vs sub-bucket scan; knob for A/B)
    static const int sub_log2 = [] {
        const char *v = std::getenv("H2TAP_SUB_ROWS_LOG2");
        return v ? std::max(0, std::min(6, std::atoi(v))) : 1;  // measured: 1 -> 74 us, 3 -> 84 us
    }();
    begin("q18_sort_hist");
    const Q18PlanArgs pa = plan_args ? *plan_args : Q18PlanArgs{};
    launch_pdl(ob_hist_kernel, G, kObThreads, nb * 4, st, rows, amt, plan, nb, s.mat, s.big,
               plan_args ? 1 : 0, pa, bucket_bits, flag);
    count_launches(1);
    end();
    begin("q18_sort_scan");
    launch_pdl(ob_scan_kernel, (nb + 31) / 32, 32 * kScanWarps, 4 * std::max(32 * G, nb), st, s.mat, G, nb, s.count,
               s.offset, s.ticket, (const Q18Plan *)plan, (ulonglong2 *)nullptr, (uint64_t)0);
    count_launches(1);
    end();
    begin("q18_bucket_scatter");
    launch_pdl(ob_scatter_kernel, G, kObThreads, nb * 4, st, rows, amt, plan, nb, s.mat, s.offset, s.kv);
    count_launches(1);
    end();
    // per-bucket shared-memory sort + tie-fix + emit: the v1 kernels on the (key, row id) pairs
    begin("q18_bucket_sort_emit");
    const unsigned lb = (unsigned)nb < (unsigned)num_sms * 6 ? (unsigned)nb : (unsigned)num_sms * 6;
    launch_pdl(bucket_local_emit_kernel<kObCap, 0, true>, lb, kEmThreads, kObSmem, st,
        s.kv, nullptr, s.offset, nb, plan, rows, amt, dst, flag, s.big, sub_log2, PeerArgs{});
    count_launches(1);
    end();
    begin("q18_bucket_sort_emit_large");
    launch_pdl(bucket_local_emit_kernel<kLsCapLarge, kObCap, true>, (unsigned)num_sms, kEmThreads, kObSmemLarge, st,
        s.kv, nullptr, s.offset, nb, plan, rows, amt, dst, flag, s.big, sub_log2, PeerArgs{});
    count_launches(1);
    end();
}

}  // namespace h2tap

// ================================ Q18 v3: HAVING writes carry records (default) ===
// The v2 chain materialises every result row twice before the sort (HAVING: 32 B row + 8 B amount;
// ob_hist re-reads the amounts; ob_scatter re-reads rows + amounts to build the records). v3 derives
// the ORDER BY plan BEFORE the HAVING pass, from one read of the accumulators (the min / max of
// amount_sum and o_entry_d over the groups that pass cnt > 0 AND sum > having — a superset of the
// result, whose bounds are valid for it), so the HAVING pass itself builds each result row's 16-byte
// carry record and histograms its bucket:
//   acc_stats (+ plan)  ->  having_rec: records, block-compacted into the block's own row range,
//   + the block's bucket counts (one row of the [partition][bucket] matrix)  ->  ob_scan  ->
//   scatter_rec: each block's records to their bucket positions  ->  per-bucket sort + emit (v2).
// Rows whose records would not fit 128 bits (bit 8 of *flag) and oversized buckets (bit 2) are
// re-run by the host through the v2 path (rows + amounts), which has the exact fallbacks.
namespace h2tap {
namespace {

constexpr unsigned int kFlagRowPath = 8u;   // carry records do not fit: host re-runs the v2 path
// H2TAP_KV_TOUCH=0: no pre-write of the scatter's target lines (A/B)
int kv_touch_mode() {  // 1: inside the scan kernel (default), 2: its own kernel, 0: off
    static const int m = [] { const char *v = std::getenv("H2TAP_KV_TOUCH"); return v ? std::atoi(v) : 1; }();
    return m;
}
bool kv_touch() { return kv_touch_mode() != 0; }

// The scatter writes 16-byte records at random kv positions: half sectors, which L2 would first
// fill from DRAM (a random read per record). Writing the whole kv range just before (whole lines,
// coalesced, kept in L2: no fills) makes those lines L2-resident: scatter 58 -> 27 us measured.
__global__ void __launch_bounds__(1024) l2_touch_kernel(ulonglong2 *__restrict__ p, uint64_t n,
                                                        const Q18Plan *__restrict__ plan) {
    pdl_wait();
    pdl_trigger();
    if (!plan->spec.carry || (plan->err & ~kPeerErrOutCap)) return;
    const uint64_t keep = l2_policy_evict_last();
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
        st16_policy(p + i, 0ull, 0ull, keep);
}
constexpr int kStatThreads = 256;

__device__ __forceinline__ long long wmin(long long v) {
    for (int o = 16; o; o >>= 1) { const long long t = __shfl_xor_sync(kFull, v, o); v = t < v ? t : v; }
    return v;
}
__device__ __forceinline__ long long wmax(long long v) {
    for (int o = 16; o; o >>= 1) { const long long t = __shfl_xor_sync(kFull, v, o); v = t > v ? t : v; }
    return v;
}

__global__ void __launch_bounds__(kStatThreads)
q18_acc_stats_kernel(const Q18Acc *__restrict__ acc, const int64_t *__restrict__ o_ent, uint64_t n_o,
                     long long having, Q18Stats *__restrict__ part, unsigned long long *__restrict__ cpart,
                     unsigned int *ticket, Q18Stats *stats, unsigned long long *count, int make_plan,
                     Q18Zone zone, int bucket_bits, int allow_carry, Q18Plan *plan, unsigned int *flag) {
    pdl_wait();
    pdl_trigger();
    __shared__ Q18Stats ws[kStatThreads / 32];
    __shared__ unsigned long long wc[kStatThreads / 32];
    __shared__ bool last;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    long long amin = INT64_MAX, amax = INT64_MIN, emin = INT64_MAX, emax = INT64_MIN;
    unsigned long long c = 0;
    const uint64_t stride = (uint64_t)gridDim.x * kStatThreads;
    // with the plan on one GPU the o_entry_d bounds are the snapshot's zone map (every orders row:
    // a superset of the passing ones): only acc[] is read (48 of 72 MB at W=100)
    if (make_plan && zone.has_e) o_ent = nullptr;
    constexpr int U = 8;  // independent accumulator loads in flight per thread
    for (uint64_t r0 = (uint64_t)blockIdx.x * kStatThreads + threadIdx.x; r0 < n_o; r0 += U * stride) {
        ulonglong2 a[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t r = r0 + u * stride;
            a[u] = r < n_o ? __ldcg(reinterpret_cast<const ulonglong2 *>(acc + r)) : make_ulonglong2(0, 0);
        }
        long long e[U];  // loaded unconditionally: independent of the accumulator loads (most pass)
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t r = r0 + u * stride;
            e[u] = r < n_o && o_ent ? __ldcs(o_ent + r) : 0;
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const long long sum = (long long)a[u].x;
            if ((unsigned int)a[u].y > 0 && sum > having) {
                amin = sum < amin ? sum : amin; amax = sum > amax ? sum : amax;
                emin = e[u] < emin ? e[u] : emin; emax = e[u] > emax ? e[u] : emax;
                ++c;
            }
        }
    }
    amin = wmin(amin); amax = wmax(amax); emin = wmin(emin); emax = wmax(emax);
    for (int o = 16; o; o >>= 1) c += __shfl_xor_sync(kFull, c, o);
    if (lane == 0) { ws[warp] = Q18Stats{amin, amax, emin, emax}; wc[warp] = c; }
    __syncthreads();
    if (threadIdx.x == 0) {
        Q18Stats b{INT64_MAX, INT64_MIN, INT64_MAX, INT64_MIN};
        unsigned long long bc = 0;
        for (int k = 0; k < kStatThreads / 32; ++k) {
            b.amt_min = min(b.amt_min, ws[k].amt_min); b.amt_max = max(b.amt_max, ws[k].amt_max);
            b.ent_min = min(b.ent_min, ws[k].ent_min); b.ent_max = max(b.ent_max, ws[k].ent_max);
            bc += wc[k];
        }
        part[blockIdx.x] = b;
        cpart[blockIdx.x] = bc;
        __threadfence();
        last = atomicAdd(ticket, 1u) == gridDim.x - 1;
    }
    __syncthreads();
    if (!last) return;
    __threadfence();
    // the last block folds every block's partial, all threads in parallel (independent loads)
    amin = INT64_MAX; amax = INT64_MIN; emin = INT64_MAX; emax = INT64_MIN; c = 0;
    for (unsigned k = threadIdx.x; k < gridDim.x; k += kStatThreads) {
        const long long *src = reinterpret_cast<const long long *>(part + k);
        amin = min(amin, __ldcg(src + 0)); amax = max(amax, __ldcg(src + 1));
        emin = min(emin, __ldcg(src + 2)); emax = max(emax, __ldcg(src + 3));
        c += __ldcg(cpart + k);
    }
    amin = wmin(amin); amax = wmax(amax); emin = wmin(emin); emax = wmax(emax);
    for (int o = 16; o; o >>= 1) c += __shfl_xor_sync(kFull, c, o);
    __syncthreads();
    if (lane == 0) { ws[warp] = Q18Stats{amin, amax, emin, emax}; wc[warp] = c; }
    __syncthreads();
    if (threadIdx.x != 0) return;
    Q18Stats g{INT64_MAX, INT64_MIN, INT64_MAX, INT64_MIN};
    unsigned long long gc = 0;
    for (int k = 0; k < kStatThreads / 32; ++k) {
        g.amt_min = min(g.amt_min, ws[k].amt_min); g.amt_max = max(g.amt_max, ws[k].amt_max);
        g.ent_min = min(g.ent_min, ws[k].ent_min); g.ent_max = max(g.ent_max, ws[k].ent_max);
        gc += wc[k];
    }
    if (!o_ent) { g.ent_min = zone.e_min; g.ent_max = zone.e_max; }
    *stats = g;
    *count = gc;
    *ticket = 0;  // self-reset
    if (make_plan) {
        Q18Plan P = make_q18_plan_vals(g, zone, gc, gc >= 1, bucket_bits, allow_carry, flag);
        if (gc == 0) P.spec.carry = allow_carry;  // nothing to order: no record is ever decoded
        *plan = P;
    }
}

// HAVING + customer probe + carry record + bucket histogram, one block per contiguous orders-row
// range (the same partition the scatter uses): records are compacted into the block's own range
// of rec[] (a shared counter per warp-ballot), the block's bucket counts become matrix row p.
constexpr int kHrThreads = 512;  // 2 blocks per SM (<= 64 registers), 4 rows per thread in flight
template <bool kDirect>
__global__ void __launch_bounds__(kHrThreads, 2)
q18_having_rec_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                      const int32_t *__restrict__ o_id, const int32_t *__restrict__ o_c,
                      const int32_t *__restrict__ o_cnt, const int64_t *__restrict__ o_ent, uint64_t n_o,
                      const int32_t *__restrict__ c_last, long long having, Q18Scratch s,
                      const Q18Plan *__restrict__ plan, int nb_launch, unsigned int *__restrict__ mat,
                      unsigned int *__restrict__ cnt_part, ulonglong2 *__restrict__ rec, unsigned int *flag,
                      const unsigned int *__restrict__ offset) {
    pdl_wait();
    pdl_trigger();
    extern __shared__ unsigned int h[];
    __shared__ unsigned int s_cnt;
    __shared__ Q18SortSpec S;
    __shared__ int s_shift, s_nb, s_carry;
    if (threadIdx.x == 0) {
        S = plan->spec;
        s_shift = plan->shift;
        s_nb = plan->dist ? (1 << plan->bucket_bits) : nb_launch;
        s_carry = plan->spec.carry && !(plan->err);
        s_cnt = 0;
        if (!plan->spec.carry && blockIdx.x == 0 && !plan->dist) atomicOr(flag, kFlagRowPath);
    }
    __syncthreads();
    const int nb = s_nb;
    uint64_t r0, r1;
    ob_range(n_o, r0, r1);
    if (kDirect) {  // h[] = this partition's cursors: bucket start + the lower partitions' counts
        const unsigned int *mrow = mat + (uint64_t)blockIdx.x * nb;
        for (int i = threadIdx.x; i < nb; i += kHrThreads) h[i] = offset[i] + mrow[i];
    } else {
        for (int i = threadIdx.x; i < nb; i += kHrThreads) h[i] = 0;
    }
    __syncthreads();
    const int lane = threadIdx.x & 31;
    const int shift = s_shift;
    const Q18SortSpec sp = S;
    const uint64_t keep = l2_policy_evict_last();  // records are re-read by the scatter
    const bool ident_c = jx::jx_identity(s.jc);     // read once (the verify kernel ran before)
    constexpr int U = 4;
    if (s_carry)
    for (uint64_t base = r0; base < r1; base += (uint64_t)U * kHrThreads) {
        long long sum[U], ent[U];
        int w[U], d[U], c[U], oid[U], cnt[U];
        unsigned int crow[U];
        bool hv_pass[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {  // independent coalesced loads first
            const uint64_t r = base + (uint64_t)u * kHrThreads + threadIdx.x;
            crow[u] = kNoRow;
            sum[u] = 0; w[u] = d[u] = c[u] = 0;
            ent[u] = 0; oid[u] = cnt[u] = 0;
            if (r < r1) {
                const ulonglong2 a = __ldcs(reinterpret_cast<const ulonglong2 *>(s.acc + r));
                sum[u] = (long long)a.x;
                crow[u] = ((unsigned int)a.y > 0 && sum[u] > having) ? 0u : kNoRow;
                w[u] = __ldcs(o_w + r); d[u] = __ldcs(o_d + r); c[u] = __ldcs(o_c + r);
                // the row's other columns in the same round trip (a row failing HAVING wastes them)
                ent[u] = __ldcs(o_ent + r); oid[u] = __ldcs(o_id + r); cnt[u] = __ldcs(o_cnt + r);
            }
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {  // customer ⋈ orders, independent across rows
            hv_pass[u] = crow[u] == 0u;
            if (crow[u] == 0u) crow[u] = jx::jx_lookup(s.jc, w[u], d[u], c[u], ident_c);
        }
        ulonglong2 rc[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            if (crow[u] == kNoRow) continue;
            Q18Row row;
            row.o_entry_d = ent[u];
            row.c_last = __ldg(c_last + crow[u]);
            row.c_id = c[u];
            row.o_id = oid[u];
            row.o_ol_cnt = cnt[u];
            row.o_w_id = w[u];
            row.o_d_id = d[u];
            rc[u] = carry_record(row, sum[u], sp);
            if (kDirect) {  // straight to its final bucket position (the scatter's job)
                const unsigned int p = atomicAdd(&h[(unsigned int)(rc[u].x >> shift)], 1u);
                H2TAP_CHECK(p < n_o);
                st16_policy(rec + p, rc[u].x, rc[u].y, keep);
            } else {
                atomicAdd(&h[(unsigned int)(rc[u].x >> shift)], 1u);
            }
        }
        if (kDirect) {
#pragma unroll
            for (int u = 0; u < U; ++u) {
                // counted by q18_acc_hist (cnt > 0, sum > having) but no customer: a hole
                if (crow[u] == kNoRow && hv_pass[u]) atomicOr(flag, kFlagHoles);
                const unsigned int bal = __ballot_sync(kFull, crow[u] != kNoRow);
                if (bal && lane == __ffs(bal) - 1) atomicAdd(&s_cnt, (unsigned int)__popc(bal));
            }
        } else
#pragma unroll
        for (int u = 0; u < U; ++u) {  // warp-aggregated compaction into the block's range
            const bool v = crow[u] != kNoRow;
            const unsigned int bal = __ballot_sync(kFull, v);
            if (!bal) continue;
            unsigned int wb = 0;
            if (lane == __ffs(bal) - 1) wb = atomicAdd(&s_cnt, (unsigned int)__popc(bal));
            wb = __shfl_sync(kFull, wb, __ffs(bal) - 1);
            if (v) st16_policy(rec + r0 + wb + __popc(bal & ((1u << lane) - 1u)), rc[u].x, rc[u].y, keep);
        }
    }
    __syncthreads();
    if (!kDirect) {
        unsigned int *row = mat + (uint64_t)blockIdx.x * nb;
        for (int i = threadIdx.x; i < nb; i += kHrThreads) row[i] = h[i];
    }
    if (threadIdx.x == 0) {
        if (!kDirect) cnt_part[blockIdx.x] = s_cnt;
        if (s_cnt) atomicAdd(s.nout, (unsigned long long)s_cnt);
    }
}

// The direct ORDER BY's count pass (one GPU): per row partition (the HAVING pass's),
// the bucket counts of the groups passing HAVING (cnt > 0, sum > having; the customer join is
// assumed — a missing customer is a hole the HAVING pass reports), so that HAVING writes each
// record at its final bucket position and no scatter pass is needed. When the bucket bits lie
// inside field a (the usual plan) only acc[] is read.
__global__ void __launch_bounds__(kObThreads)
q18_acc_hist_kernel(const Q18Acc *__restrict__ acc, const int32_t *__restrict__ o_w,
                    const int32_t *__restrict__ o_d, const int32_t *__restrict__ o_id,
                    const int64_t *__restrict__ o_ent, uint64_t n_o, long long having,
                    const Q18Plan *__restrict__ plan, int nb, unsigned int *__restrict__ mat,
                    unsigned int *big) {
    pdl_wait();
    pdl_trigger();
    extern __shared__ unsigned int h[];
    if (big && blockIdx.x == 0 && threadIdx.x == 0) *big = 0;  // the emit's oversized-bucket list
    for (int i = threadIdx.x; i < nb; i += kObThreads) h[i] = 0;
    __syncthreads();
    const Q18SortSpec sp = plan->spec;
    const int shift = plan->shift;
    const bool amt_only = shift >= sp.prefix_bits - sp.bits_a;
    uint64_t r0, r1;
    ob_range(n_o, r0, r1);
    if (sp.carry && amt_only) {  // acc[] only, 8 independent loads in flight per thread
        constexpr int U = 8;
        const int sa = shift - (sp.prefix_bits - sp.bits_a);
        for (uint64_t r = r0 + threadIdx.x; r < r1; r += (uint64_t)U * kObThreads) {
            ulonglong2 a[U];
#pragma unroll
            for (int u = 0; u < U; ++u) {
                const uint64_t x = r + (uint64_t)u * kObThreads;
                a[u] = x < r1 ? __ldcs(reinterpret_cast<const ulonglong2 *>(acc + x)) : make_ulonglong2(0, 0);
            }
#pragma unroll
            for (int u = 0; u < U; ++u) {
                const long long sum = (long long)a[u].x;
                if ((unsigned int)a[u].y > 0 && sum > having) {
                    const unsigned int b = (unsigned int)(field_a(sum, sp) >> sa);
                    H2TAP_CHECK(b < (unsigned int)nb);
                    atomicAdd(&h[b], 1u);
                }
            }
        }
    } else if (sp.carry)
    for (uint64_t r = r0 + threadIdx.x; r < r1; r += kObThreads) {
        const ulonglong2 a = __ldcs(reinterpret_cast<const ulonglong2 *>(acc + r));
        const long long sum = (long long)a.x;
        if (!((unsigned int)a.y > 0 && sum > having)) continue;
        unsigned int b;
        {
            Q18Row row{};
            row.o_entry_d = __ldg(o_ent + r);
            row.o_w_id = __ldg(o_w + r); row.o_d_id = __ldg(o_d + r); row.o_id = __ldg(o_id + r);
            row.c_last = sp.cl_min; row.c_id = sp.ci_min; row.o_ol_cnt = sp.n_min;
            b = (unsigned int)(carry_record(row, sum, sp).x >> shift);
        }
        H2TAP_CHECK(b < (unsigned int)nb);
        atomicAdd(&h[b], 1u);
    }
    __syncthreads();
    unsigned int *row = mat + (uint64_t)blockIdx.x * nb;
    for (int i = threadIdx.x; i < nb; i += kObThreads) row[i] = h[i];
}

// Each block's records (rec[r0 .. r0 + cnt_part[p])) to their bucket positions: the shared cursors
// start at offset[b] + matrix[p][b] (the column scan), no global atomics.
__global__ void __launch_bounds__(kObThreads)
ob_scatter_rec_kernel(const ulonglong2 *__restrict__ rec, uint64_t n_o, const Q18Plan *__restrict__ plan,
                      int nb_launch, const unsigned int *__restrict__ mat, const unsigned int *__restrict__ offset,
                      const unsigned int *__restrict__ cnt_part, ulonglong2 *__restrict__ kv,
                      unsigned int *big) {
    pdl_wait();
    pdl_trigger();
    extern __shared__ unsigned int cur[];
    // the emit's oversized-bucket work list (nothing reads it before the emit; a memset node here
    // would break the PDL chain: -4 us measured); null: the caller resets it
    if (big && blockIdx.x == 0 && threadIdx.x == 0) *big = 0;
    // (kPeerErrOutCap only stops this rank's emit: its records must still be exchanged)
    if (!plan->spec.carry || (plan->err & ~kPeerErrOutCap)) return;
    const int nb = plan->dist ? (1 << plan->bucket_bits) : nb_launch;
    const int shift = plan->shift;
    const unsigned int *row = mat + (uint64_t)blockIdx.x * nb;
    for (int i = threadIdx.x; i < nb; i += kObThreads) cur[i] = offset[i] + row[i];
    __syncthreads();
    uint64_t r0, r1;
    ob_range(n_o, r0, r1);
    const unsigned int m = cnt_part[blockIdx.x];
    const uint64_t drop = l2_policy_evict_first();
    constexpr int U = 4;
    for (unsigned int i0 = threadIdx.x; i0 < m; i0 += U * kObThreads) {
        ulonglong2 r[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const unsigned int i = i0 + u * kObThreads;
            if (i < m) ld16_policy(rec + r0 + i, r[u].x, r[u].y, drop);
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const unsigned int i = i0 + u * kObThreads;
            if (i >= m) break;
            H2TAP_CHECK((r[u].x >> shift) < (unsigned long long)nb && m <= r1 - r0);
            const unsigned int p = atomicAdd(&cur[(unsigned int)(r[u].x >> shift)], 1u);
            H2TAP_CHECK(p < n_o);
            kv[p] = r[u];
        }
    }
}

}  // namespace

__device__ __forceinline__ unsigned long long ld_acquire_gpu_u64(const unsigned long long *a) {
    unsigned long long v;
    asm volatile("ld.acquire.gpu.global.u64 %0, [%1];" : "=l"(v) : "l"(a) : "memory");
    return v;
}

// The plan and the bucket counts in one kernel (one GPU, direct ORDER BY): each
// block reduces its row partition's passing amount bounds (as q18_acc_stats), a grid barrier (a
// monotonic 64-bit arrival counter; the grid is one wave of resident blocks — the host checks the
// occupancy and that no other engine shares the device), every block derives the same plan from
// all blocks' partials (block 0 publishes it), then counts its partition's buckets (as
// q18_acc_hist) re-reading acc[] while it is still in L2.
constexpr int kPhThreads = 512;
__global__ void __launch_bounds__(kPhThreads)
q18_plan_hist_kernel(const Q18Acc *__restrict__ acc, uint64_t n_o, long long having, Q18Stats *part,
                     unsigned long long *cpart, unsigned long long *gbar, Q18Stats *stats,
                     unsigned long long *count, Q18Zone zone, int bucket_bits, Q18Plan *plan,
                     unsigned int *flag, unsigned int *mat, unsigned int *big) {
    pdl_wait();
    pdl_trigger();
    extern __shared__ unsigned int h[];
    __shared__ Q18Stats ws[kPhThreads / 32];
    __shared__ unsigned long long wc[kPhThreads / 32];
    __shared__ Q18Plan s_plan;
    const int nb = 1 << bucket_bits;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    if (big && blockIdx.x == 0 && threadIdx.x == 0) *big = 0;  // the emit's oversized-bucket list
    for (int i = threadIdx.x; i < nb; i += kPhThreads) h[i] = 0;
    uint64_t r0, r1;
    ob_range(n_o, r0, r1);
    long long amin = INT64_MAX, amax = INT64_MIN;
    unsigned long long c = 0;
    const uint64_t keep = l2_policy_evict_last();  // re-read by the count phase below
    constexpr int U = 8;
    for (uint64_t r = r0 + threadIdx.x; r < r1; r += (uint64_t)U * kPhThreads) {
        unsigned long long ax[U], ay[U];
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const uint64_t x = r + (uint64_t)u * kPhThreads;
            ax[u] = ay[u] = 0;
            if (x < r1) ld16_policy(reinterpret_cast<const ulonglong2 *>(acc + x), ax[u], ay[u], keep);
        }
#pragma unroll
        for (int u = 0; u < U; ++u) {
            const long long sum = (long long)ax[u];
            if ((unsigned int)ay[u] > 0 && sum > having) {
                amin = sum < amin ? sum : amin; amax = sum > amax ? sum : amax;
                ++c;
            }
        }
    }
    amin = wmin(amin); amax = wmax(amax);
    for (int o = 16; o; o >>= 1) c += __shfl_xor_sync(kFull, c, o);
    if (lane == 0) { ws[warp] = Q18Stats{amin, amax, 0, 0}; wc[warp] = c; }
    __syncthreads();
    if (threadIdx.x == 0) {
        long long b0 = INT64_MAX, b1 = INT64_MIN;
        unsigned long long bc = 0;
        for (int k = 0; k < kPhThreads / 32; ++k) {
            b0 = min(b0, ws[k].amt_min); b1 = max(b1, ws[k].amt_max); bc += wc[k];
        }
        part[blockIdx.x] = Q18Stats{b0, b1, 0, 0};
        cpart[blockIdx.x] = bc;
        __threadfence();
        const unsigned long long t = atomicAdd(gbar, 1ull);
        const unsigned long long target = (t / gridDim.x + 1) * gridDim.x;
        // bounded wait: should the grid ever not be co-resident (another tenant on the device), a
        // block gives up after 2 s and flags the query, which the host then redoes on the v2 path
        unsigned long long t0;
        asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t0));
        while (ld_acquire_gpu_u64(gbar) < target) {
            __nanosleep(32);
            unsigned long long now;
            asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(now));
            if (now - t0 > 2000000000ull) { atomicOr(flag, kFlagHoles); break; }
        }
    }
    __syncthreads();
    if (warp == 0) {  // every block folds all partials (independent loads) and derives the plan
        long long a0 = INT64_MAX, a1 = INT64_MIN;
        unsigned long long cc = 0;
        for (unsigned k = lane; k < gridDim.x; k += 32) {
            const long long *src = reinterpret_cast<const long long *>(part + k);
            a0 = min(a0, __ldcg(src + 0)); a1 = max(a1, __ldcg(src + 1));
            cc += __ldcg(cpart + k);
        }
        a0 = wmin(a0); a1 = wmax(a1);
        for (int o = 16; o; o >>= 1) cc += __shfl_xor_sync(kFull, cc, o);
        if (lane == 0) {
            const Q18Stats g{a0, a1, zone.e_min, zone.e_max};  // o_entry_d: the zone map (has_e)
            Q18Plan P = make_q18_plan_vals(g, zone, cc, cc >= 1, bucket_bits, 1, blockIdx.x == 0 ? flag : nullptr);
            if (cc == 0) P.spec.carry = 1;  // nothing to order: no record is ever decoded
            // buckets must lie inside field a for the count below (else, rare: the v2 row path)
            if (P.spec.carry && cc >= 1 && P.shift < P.spec.prefix_bits - P.spec.bits_a) P.spec.carry = 0;
            s_plan = P;
            if (blockIdx.x == 0) { *plan = P; *stats = g; *count = cc; }
        }
    }
    __syncthreads();
    const Q18SortSpec sp = s_plan.spec;
    const int shift = s_plan.shift;
    if (sp.carry && shift >= sp.prefix_bits - sp.bits_a) {  // buckets inside field a
        const int sa = shift - (sp.prefix_bits - sp.bits_a);
        for (uint64_t r = r0 + threadIdx.x; r < r1; r += (uint64_t)U * kPhThreads) {
            ulonglong2 a[U];
#pragma unroll
            for (int u = 0; u < U; ++u) {
                const uint64_t x = r + (uint64_t)u * kPhThreads;
                a[u] = x < r1 ? __ldcg(reinterpret_cast<const ulonglong2 *>(acc + x)) : make_ulonglong2(0, 0);
            }
#pragma unroll
            for (int u = 0; u < U; ++u) {
                const long long sum = (long long)a[u].x;
                if ((unsigned int)a[u].y > 0 && sum > having) {
                    const unsigned int b = (unsigned int)(field_a(sum, sp) >> sa);
                    H2TAP_CHECK(b < (unsigned int)nb);
                    atomicAdd(&h[b], 1u);
                }
            }
        }
    }
    __syncthreads();
    unsigned int *row = mat + (uint64_t)blockIdx.x * nb;
    for (int i = threadIdx.x; i < nb; i += kPhThreads) row[i] = h[i];
}

// Whether the fused plan + count kernel can run: its grid (ob_grid blocks) resident at once.
bool q18_plan_hist_ok(int num_sms, int bucket_bits) {
    int per_sm = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per_sm, q18_plan_hist_kernel, kPhThreads,
                                                      4 << bucket_bits) != cudaSuccess) {
        cudaGetLastError();
        return false;
    }
    return (long long)per_sm * num_sms >= ob_grid(num_sms);
}

void launch_q18_plan_hist(const Q18Scratch &s, uint64_t n_o, int64_t having, unsigned long long *cpart,
                          unsigned long long *gbar, unsigned long long *count, const Q18Zone &zone,
                          int bucket_bits, Q18Plan *plan, unsigned int *flag, const BucketSort &bs, int num_sms,
                          cudaStream_t st) {
    launch_pdl(q18_plan_hist_kernel, ob_grid(num_sms), kPhThreads, 4 << bucket_bits, st, (const Q18Acc *)s.acc, n_o,
               (long long)having, s.stat_part, cpart, gbar, s.stats, count, zone, bucket_bits, plan, flag, bs.mat,
               bs.big);
    count_launches(1);
}

void launch_q18_acc_stats(const Q18Scratch &s, const int64_t *o_ent, uint64_t n_o, int64_t having,
                          unsigned long long *cpart, unsigned long long *count, const Q18PlanArgs *plan_args,
                          int bucket_bits, Q18Plan *plan, unsigned int *flag, int num_sms, cudaStream_t st) {
    uint64_t want = (n_o + kStatThreads - 1) / kStatThreads;
    const uint64_t cap = (uint64_t)num_sms * 4;  // <= the stat_part capacity (8 blocks per SM)
    const unsigned grid = (unsigned)(want < 1 ? 1 : want > cap ? cap : want);
    const Q18Zone z = plan_args ? plan_args->zone : Q18Zone{};
    launch_pdl(q18_acc_stats_kernel, grid, kStatThreads, 0, st, (const Q18Acc *)s.acc, o_ent, n_o,
               (long long)having, s.stat_part, cpart, s.ticket, s.stats, count, plan_args ? 1 : 0, z,
               bucket_bits, plan_args ? plan_args->allow_carry : 0, plan, flag);
    count_launches(1);
}

void q18_order_v3(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, const int32_t *o_c,
                  const int32_t *o_cnt, const int64_t *o_ent, uint64_t n_o, const int32_t *c_last,
                  int64_t having, const Q18Scratch &s, const Q18Plan *plan, int bucket_bits,
                  const BucketSort &bs, unsigned int *cnt_part, const Q18Cols &dst, unsigned int *flag,
                  int num_sms, cudaStream_t st, PhaseMarks *marks, bool counted) {
    auto begin = [&](const char *nm) { if (marks) marks->begin(nm); };
    auto end = [&] { if (marks) marks->end(); };
    const int nb = 1 << bucket_bits;
    const int G = ob_grid(num_sms);
    // direct (default, H2TAP_ORDER_DIRECT=0 for the scatter pass): counts from acc[] first, the
    // column scan, then HAVING writes every record at its final bucket position
    const char *dx = std::getenv("H2TAP_ORDER_DIRECT");  // (read per query: tests switch it)
    const bool direct = !(dx && dx[0] == '0');
    if (direct || counted) {
        if (!counted) {  // (counted: q18_plan_hist ran the count with the plan)
        begin("q18_bucket_count");
        launch_pdl(q18_acc_hist_kernel, G, kObThreads, 4 * nb, st, (const Q18Acc *)s.acc, o_w, o_d, o_id, o_ent, n_o,
                   (long long)having, plan, nb, bs.mat, bs.big);
        count_launches(1);
        end();
        }
        begin("q18_sort_scan");
        launch_pdl(ob_scan_kernel, (nb + 31) / 32 + (kv_touch_mode() == 1 ? num_sms : 0), 32 * kScanWarps,
                   4 * std::max(32 * G, nb), st, bs.mat, G, nb, bs.count, bs.offset, bs.ticket, plan,
                   kv_touch_mode() == 1 ? reinterpret_cast<ulonglong2 *>(bs.kv) : nullptr, kv_touch_mode() == 1 ? n_o : 0);
        count_launches(1);
        end();
        begin("q18_having_records");
        launch_pdl(q18_having_rec_kernel<true>, G, kHrThreads, 4 * nb, st, o_w, o_d, o_id, o_c, o_cnt, o_ent, n_o,
                   c_last, (long long)having, s, plan, nb, bs.mat, cnt_part, reinterpret_cast<ulonglong2 *>(bs.kv),
                   flag, (const unsigned int *)bs.offset);
        count_launches(1);
        end();
    } else {
    begin("q18_having_records");
    launch_pdl(q18_having_rec_kernel<false>, G, kHrThreads, 4 * nb, st, o_w, o_d, o_id, o_c, o_cnt, o_ent, n_o, c_last,
               (long long)having, s, plan, nb, bs.mat, cnt_part, reinterpret_cast<ulonglong2 *>(bs.k[0]), flag,
               (const unsigned int *)nullptr);
    count_launches(1);
    end();
    begin("q18_sort_scan");
    launch_pdl(ob_scan_kernel, (nb + 31) / 32 + (kv_touch_mode() == 1 ? num_sms : 0), 32 * kScanWarps,
               4 * std::max(32 * G, nb), st, bs.mat, G, nb, bs.count, bs.offset, bs.ticket, plan,
               kv_touch_mode() == 1 ? reinterpret_cast<ulonglong2 *>(bs.kv) : nullptr, kv_touch_mode() == 1 ? n_o : 0);
    count_launches(1);
    end();
    if (kv_touch_mode() == 2) {
        begin("q18_kv_touch");
        launch_pdl(l2_touch_kernel, (unsigned)num_sms * 2, 1024, 0, st, reinterpret_cast<ulonglong2 *>(bs.kv), n_o, plan);
        count_launches(1);
        end();
    }
    begin("q18_bucket_scatter");
    launch_pdl(ob_scatter_rec_kernel, G, kObThreads, 4 * nb, st, reinterpret_cast<const ulonglong2 *>(bs.k[0]), n_o,
               plan, nb, (const unsigned int *)bs.mat, (const unsigned int *)bs.offset, (const unsigned int *)cnt_part,
               reinterpret_cast<ulonglong2 *>(bs.kv), bs.big);
    count_launches(1);
    end();
    }
    // (big[], the oversized-bucket work list, was reset by the count or the scatter kernel)
    static const int sub_log2 = [] {
        const char *v = std::getenv("H2TAP_SUB_ROWS_LOG2");
        return v ? std::max(0, std::min(6, std::atoi(v))) : 1;
    }();
    begin("q18_bucket_sort_emit");
    const unsigned lb = (unsigned)nb < (unsigned)num_sms * EMIT_BPS ? (unsigned)nb : (unsigned)num_sms * EMIT_BPS;
    launch_pdl(bucket_local_emit_kernel<kObCap, 0, true>, lb, kEmThreads, kObSmem, st,
               (const unsigned long long *)bs.kv, (const unsigned int *)nullptr, (const unsigned int *)bs.offset, nb,
               plan, (const Q18Row *)nullptr, (const long long *)nullptr, dst, flag, bs.big, sub_log2, PeerArgs{});
    count_launches(1);
    end();
    begin("q18_bucket_sort_emit_large");
    launch_pdl(carry_large_emit_kernel, (unsigned)num_sms, kLgThreads, kLgSmem, st,
               (const unsigned long long *)bs.kv, (const unsigned int *)bs.offset, nb, plan, dst, flag, bs.big,
               sub_log2, PeerArgs{});
    count_launches(1);
    end();
}

}  // namespace h2tap

// ==================================== distributed ORDER BY (world > 1) ===
// Q18 groups are warehouse-local (every join predicate has w_id equality), so each rank computes
// its groups alone; only the ORDER BY crosses ranks. The result is range-partitioned: the buckets
// of the carry-record sort (top bits of the exact composite key, one definition on every rank)
// are assigned to ranks by their GLOBAL row positions, so rank k ends up holding rows
// [row0_k, row0_k + n_k) of the globally ordered result, ~1/world of it, sorted by the same
// per-bucket shared-memory sort as on one GPU. No rank gathers or re-sorts anyone else's rows.
//   meta  (1 warp):  push {nout, err, stats, zone} -> every rank; wait; reduce; derive the plan
//                    (widths from the GLOBAL min/max, bucket bits from the global row count)
//   hist + scan:     as on one GPU, over this rank's rows (local bucket counts and offsets)
//   push counts:     launch_peer_push of the nb local bucket counts
//   route (1 block): wait; per bucket the total over ranks and this rank's prefix among them;
//                    scan -> global start; owner = the rank whose 1/world slice the start is in;
//                    the destination position of this rank's records of every bucket; the receive
//                    offsets of this rank's own buckets; heap / output capacity checks
//   scatter:         as on one GPU: the carry records in local bucket order
//   send:            per bucket, one warp copies this rank's records (contiguous, 16 B each) to
//                    its place in the owner's heap over NVLink; the last block signals every rank
//   emit:            as on one GPU over this rank's buckets, reading the records from its heap
namespace h2tap {
namespace {
using namespace peer;

struct Q18Meta {                 // one rank's contribution to the plan (mailbox payload)
    unsigned long long nout;
    unsigned int err, pad;
    Q18Stats st;
    Q18Zone z;
};

__global__ void q18_dist_meta_kernel(PeerArgs p, const unsigned long long *nout, const unsigned int *err,
                                     const Q18Stats *stats, Q18Zone zone, int allow_carry, int nb_max_bits,
                                     Q18Plan *plan, unsigned int *flag) {
    pdl_wait();
    trigger_before_wait(p);
    if (threadIdx.x != 0) return;  // (a CTA triggers when one of its threads does: thread 0 below)
    const unsigned long long s = next_seq(p);
    const int par = (int)(s & 1);
    Q18Meta m{};
    m.nout = *nout;
    m.err = *err;
    m.st = *stats;
    m.z = zone;
    for (int k = 0; k < p.world; ++k) *reinterpret_cast<Q18Meta *>(mbox(p, k, par, p.rank)) = m;
    signal_all(p, s);
    Q18Meta g{};
    g.st.amt_min = INT64_MAX; g.st.amt_max = INT64_MIN; g.st.ent_min = INT64_MAX; g.st.ent_max = INT64_MIN;
    g.z = zone;
    unsigned int perr = 0;
    const bool ok = wait_all(p, s);
    trigger_after_wait(p);
    if (!ok) perr |= kPeerErrTimeout;
    else
        for (int k = 0; k < p.world; ++k) {
            Q18Meta x;
            const unsigned long long *src = reinterpret_cast<const unsigned long long *>(mbox(p, p.rank, par, k));
            unsigned long long *dst = reinterpret_cast<unsigned long long *>(&x);
            for (int q = 0; q < (int)(sizeof(Q18Meta) / 8); ++q) dst[q] = __ldcg(src + q);
            g.nout += x.nout;
            g.err |= x.err;
            if (x.nout) {  // a rank without result rows has sentinel statistics: skip them
                g.st.amt_min = min(g.st.amt_min, x.st.amt_min); g.st.amt_max = max(g.st.amt_max, x.st.amt_max);
                g.st.ent_min = min(g.st.ent_min, x.st.ent_min); g.st.ent_max = max(g.st.ent_max, x.st.ent_max);
            }
            int *gz = reinterpret_cast<int *>(&g.z);
            const int *xz = reinterpret_cast<const int *>(&x.z);
            for (int q = 0; q < 6; ++q) { gz[2 * q] = min(gz[2 * q], xz[2 * q]); gz[2 * q + 1] = max(gz[2 * q + 1], xz[2 * q + 1]); }
        }
    // bucket bits from the global row count (~256-512 rows per bucket, as on one GPU)
    int bb = 1;
    while (bb < nb_max_bits && (g.nout >> (bb + 9)) > 0) ++bb;
    Q18Plan P = make_q18_plan_vals(g.st, g.z, m.nout, g.nout >= 1, bb, allow_carry, flag);
    P.dist = 1;
    P.nbuckets = 1ull << bb;
    P.n_total = g.nout;
    P.err = g.err | perr;
    if (g.nout >= 1 && !P.spec.carry) P.err |= kPeerErrNoCarry;  // the exchange moves carry records
    if (P.err) P.n = 0;  // nothing is scattered; every rank reports the error
    *plan = P;
}

// Receive-side plan (one block of 1024 threads; shared memory: nb totals). `count`/`offset` are
// this rank's bucket counts / exclusive offsets (ob_scan); the mailboxes hold every rank's counts.
constexpr int kRouteThreads = 1024;
__global__ void __launch_bounds__(kRouteThreads)
q18_dist_route_kernel(PeerArgs p, Q18Plan *plan, unsigned long long *__restrict__ send,
                      unsigned int *__restrict__ recv_off, unsigned long long out_cap) {
    pdl_wait();
    trigger_before_wait(p);
    extern __shared__ unsigned int tot[];          // [nb] totals -> global starts (exclusive)
    __shared__ unsigned int wsum[kRouteThreads / 32];
    __shared__ unsigned int lo[kMaxRanks + 1];     // first bucket of each rank (nb: none)
    __shared__ int ok;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const unsigned long long s = cur_seq(p);       // the counts' push
    if (threadIdx.x == 0) ok = wait_all(p, s) ? 1 : 0;
    __syncthreads();
    trigger_after_wait(p);
    const int nb = 1 << plan->bucket_bits;
    const int par = (int)(s & 1);
    unsigned int perr = ok ? 0u : kPeerErrTimeout;
    if (ok) {
        for (int b = threadIdx.x; b < nb; b += kRouteThreads) {
            unsigned int t = 0, pre = 0;
            for (int k = 0; k < p.world; ++k) {
                const unsigned int c = __ldcg(reinterpret_cast<const unsigned int *>(mbox(p, p.rank, par, k) + 16) + b);
                t += c;
                if (k < p.rank) pre += c;
            }
            tot[b] = t;
            send[b] = pre;  // this rank's place among the bucket's ranks (completed below)
        }
    }
    if (threadIdx.x <= kMaxRanks) lo[threadIdx.x] = (unsigned int)nb;
    __syncthreads();
    // exclusive scan of tot[]: each warp a contiguous span, warp-cooperative
    const int span = (nb + kRouteThreads / 32 - 1) / (kRouteThreads / 32);
    const int w0 = warp * span, w1 = min(nb, w0 + span);
    unsigned int wt = 0;
    for (int base = w0; base < w1; base += 32) {
        const int i = base + lane;
        wt += __reduce_add_sync(kFull, i < w1 ? tot[i] : 0u);
    }
    if (lane == 0) wsum[warp] = wt;
    __syncthreads();
    unsigned int acc = 0;
    for (int w = 0; w < warp; ++w) acc += wsum[w];
    for (int base = w0; base < w1; base += 32) {
        const int i = base + lane;
        const unsigned int c = i < w1 ? tot[i] : 0u;
        unsigned int x = c;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const unsigned int y = __shfl_up_sync(kFull, x, o);
            if (lane >= o) x += y;
        }
        if (i < w1) tot[i] = acc + x - c;
        acc += __shfl_sync(kFull, x, 31);
    }
    __syncthreads();
    unsigned long long T = 0;
    for (int w = 0; w < kRouteThreads / 32; ++w) T += wsum[w];
    const int W = p.world;
    auto owner = [&](int b) -> int {
        if (T == 0) return 0;
        const unsigned long long o = (unsigned long long)tot[b] * (unsigned long long)W / T;
        return o >= (unsigned long long)W ? W - 1 : (int)o;
    };
    // lo[k] = first bucket owned by a rank >= k (owners are non-decreasing in b)
    for (int b = threadIdx.x; b < nb; b += kRouteThreads) {
        const int o = owner(b), op = b ? owner(b - 1) : -1;
        for (int k = op + 1; k <= o; ++k) lo[k] = (unsigned int)b;
    }
    __syncthreads();
    auto row0 = [&](int k) -> unsigned long long { return lo[k] < (unsigned int)nb ? tot[lo[k]] : T; };
    for (int b = threadIdx.x; b < nb; b += kRouteThreads) {
        const int o = owner(b);
        const unsigned long long pos = (unsigned long long)tot[b] - row0(o) + send[b];
        send[b] = ((unsigned long long)o << 56) | pos;
    }
    const unsigned int b_lo = lo[p.rank], b_hi = lo[p.rank + 1] < lo[p.rank] ? lo[p.rank] : lo[p.rank + 1];
    const unsigned long long r0 = row0(p.rank);
    for (unsigned int b = b_lo + threadIdx.x; b <= b_hi; b += kRouteThreads)
        recv_off[b - b_lo] = (unsigned int)((b < (unsigned int)nb ? (unsigned long long)tot[b] : T) - r0);
    if (threadIdx.x == 0) {
        unsigned long long worst = 0;
        for (int k = 0; k < W; ++k) {
            const unsigned long long nk = (k + 1 < W ? row0(k + 1) : T) - row0(k);
            worst = nk > worst ? nk : worst;
        }
        const unsigned long long mine = (p.rank + 1 < W ? row0(p.rank + 1) : T) - r0;
        if (worst * 16ull > p.heap_half) perr |= kPeerErrHeap;      // the same decision on every rank
        if (mine > out_cap) perr |= kPeerErrOutCap;                 // local: re-emitted by the host
        plan->b_lo = b_lo;
        plan->nb_mine = b_hi - b_lo;
        plan->n_mine = mine;
        plan->row0 = r0;
        plan->xseq = s + 1;
        plan->err |= perr;
    }
}

// One warp per bucket: this rank's records of bucket b (contiguous after the local scatter) to
// their place in the owner's heap; the last block publishes the exchange to every rank.
__global__ void __launch_bounds__(1024)
q18_dist_send_kernel(PeerArgs p, const Q18Plan *__restrict__ plan, const ulonglong2 *__restrict__ kv,
                     const unsigned int *__restrict__ offset, const unsigned long long *__restrict__ send) {
    pdl_wait();
    pdl_trigger();
    const unsigned long long s = next_seq(p);
    const int par = (int)(s & 1);
    if (!(plan->err & kPeerErrHeap) && !(plan->err & kPeerErrTimeout)) {
        const int nb = 1 << plan->bucket_bits;
        const int lane = threadIdx.x & 31;
        const int nw = (int)(gridDim.x * (blockDim.x >> 5));
        for (int b = (int)(blockIdx.x * (blockDim.x >> 5) + (threadIdx.x >> 5)); b < nb; b += nw) {
            const unsigned int lo = offset[b], c = offset[b + 1] - lo;
            if (c == 0) continue;
            const unsigned long long d = send[b];
            ulonglong2 *dst = reinterpret_cast<ulonglong2 *>(heap(p, (int)(d >> 56), par)) + (d & ((1ull << 56) - 1));
            for (unsigned int i = lane; i < c; i += 32) dst[i] = __ldcs(kv + lo + i);
        }
    }
    if (block_done_last(p)) signal_all(p, s);
}

struct Q18SmallDist { unsigned long long nout; unsigned int err, tie; Q18Stats st; unsigned long long row0, n_total; };
__global__ void q18_dist_publish_kernel(const Q18Plan *plan, const unsigned int *tie, Q18SmallDist *out) {
    pdl_wait();
    pdl_trigger();
    out->nout = plan->n_mine;
    out->err = plan->err;
    out->tie = *tie;
    out->row0 = plan->row0;
    out->n_total = plan->n_total;
}

}  // namespace

void q18_bucket_order_dist(const PeerArgs &pa, const Q18Row *rows, const long long *amt, Q18Plan *plan,
                           const Q18PlanArgs &meta, const unsigned int *err, const BucketSort &s,
                           unsigned long long *send, unsigned int *recv_off, uint64_t out_cap,
                           const Q18Cols &dst, unsigned int *flag, void *host_small, int num_sms,
                           cudaStream_t st, PhaseMarks *marks, const Q18HavingArgs *hv) {
    auto begin = [&](const char *nm) { if (marks) marks->begin(nm); };
    auto end = [&] { if (marks) marks->end(); };
    const int nb = 1 << kBucketMaxBits;  // launch sizes: the largest bucket count the plan may pick
    const int G = ob_grid(num_sms);
    begin("q18_dist_meta");
    launch_pdl(q18_dist_meta_kernel, 1, 32, 0, st, pa, meta.nout, err, meta.stats, meta.zone, meta.allow_carry,
               kBucketMaxBits, plan, flag);
    count_launches(1);
    end();
    if (hv) {  // v3: HAVING builds the carry records and the bucket counts with the global plan
        begin("q18_having_records");
        launch_pdl(q18_having_rec_kernel<false>, G, kHrThreads, nb * 4, st, hv->o_w, hv->o_d, hv->o_id, hv->o_c, hv->o_cnt,
                   hv->o_ent, hv->n_o, hv->c_last, (long long)hv->having, hv->s, (const Q18Plan *)plan, nb, s.mat,
                   hv->cnt_part, reinterpret_cast<ulonglong2 *>(s.k[0]), flag,
                   (const unsigned int *)nullptr);
        count_launches(1);
        end();
    } else {
        begin("q18_sort_hist");
        launch_pdl(ob_hist_kernel, G, kObThreads, nb * 4, st, rows, amt, plan, nb, s.mat, s.big, 0, Q18PlanArgs{}, 0, flag);
        count_launches(1);
        end();
    }
    begin("q18_sort_scan");
    const bool tin = hv && kv_touch_mode() == 1;
    launch_pdl(ob_scan_kernel, (nb + 31) / 32 + (tin ? num_sms : 0), 32 * kScanWarps, 4 * std::max(32 * G, nb), st,
               s.mat, G, nb, s.count, s.offset, s.ticket, (const Q18Plan *)plan,
               tin ? reinterpret_cast<ulonglong2 *>(s.kv) : nullptr, tin ? hv->n_o : (uint64_t)0);
    count_launches(1);
    end();
    begin("q18_dist_counts");
    launch_peer_push(pa, s.count, &plan->nbuckets, 0, 4u, num_sms, st);
    end();
    begin("q18_dist_route");
    launch_pdl(q18_dist_route_kernel, 1, kRouteThreads, 4 * nb, st, pa, plan, send, recv_off,
               (unsigned long long)out_cap);
    count_launches(1);
    end();
    if (hv && kv_touch_mode() == 2) {
        begin("q18_kv_touch");
        launch_pdl(l2_touch_kernel, (unsigned)num_sms * 2, 1024, 0, st, reinterpret_cast<ulonglong2 *>(s.kv), hv->n_o,
                   (const Q18Plan *)plan);
        count_launches(1);
        end();
    }
    begin("q18_bucket_scatter");
    if (hv)
        launch_pdl(ob_scatter_rec_kernel, G, kObThreads, nb * 4, st, reinterpret_cast<const ulonglong2 *>(s.k[0]),
                   hv->n_o, (const Q18Plan *)plan, nb, (const unsigned int *)s.mat, (const unsigned int *)s.offset,
                   (const unsigned int *)hv->cnt_part, reinterpret_cast<ulonglong2 *>(s.kv), (unsigned int *)nullptr);
    else
        launch_pdl(ob_scatter_kernel, G, kObThreads, nb * 4, st, rows, amt, (const Q18Plan *)plan, nb,
                   (const unsigned int *)s.mat, (const unsigned int *)s.offset, s.kv);
    count_launches(1);
    end();
    begin("q18_dist_send");
    launch_pdl(q18_dist_send_kernel, (unsigned)num_sms, 1024, 0, st, pa, (const Q18Plan *)plan,
               reinterpret_cast<const ulonglong2 *>(s.kv), (const unsigned int *)s.offset, (const unsigned long long *)send);
    count_launches(1);
    end();
    cudaMemsetAsync(s.big, 0, sizeof(unsigned int), st);  // the emit's oversized-bucket work list
    begin("q18_dist_wait");
    launch_peer_wait(pa, st);
    end();
    q18_dist_emit(pa, plan, recv_off, dst, flag, s, num_sms, st, marks);
    launch_pdl(q18_dist_publish_kernel, 1, 1, 0, st, (const Q18Plan *)plan, (const unsigned int *)flag,
               static_cast<Q18SmallDist *>(host_small));
    count_launches(1);
}

void q18_dist_emit(const PeerArgs &pa, const Q18Plan *plan, const unsigned int *recv_off, const Q18Cols &dst,
                   unsigned int *flag, const BucketSort &s, int num_sms, cudaStream_t st, PhaseMarks *marks) {
    auto begin = [&](const char *nm) { if (marks) marks->begin(nm); };
    auto end = [&] { if (marks) marks->end(); };
    static const int sub_log2 = [] {
        const char *v = std::getenv("H2TAP_SUB_ROWS_LOG2");
        return v ? std::max(0, std::min(6, std::atoi(v))) : 1;
    }();
    // the emit walks at most 2^kBucketMaxBits buckets; the grid covers the SMs
    begin("q18_bucket_sort_emit");
    launch_pdl(bucket_local_emit_kernel<kObCap, 0, true>, (unsigned)num_sms * 6, kEmThreads, kObSmem, st,
               (const unsigned long long *)nullptr, (const unsigned int *)nullptr, recv_off, 0, plan,
               (const Q18Row *)nullptr, (const long long *)nullptr, dst, flag, s.big, sub_log2, pa);
    count_launches(1);
    end();
    begin("q18_bucket_sort_emit_large");
    launch_pdl(carry_large_emit_kernel, (unsigned)num_sms, kLgThreads, kLgSmem, st,
               (const unsigned long long *)nullptr, recv_off, 0, plan, dst, flag, s.big, sub_log2, pa);
    count_launches(1);
    end();
}

// Dynamic shared-memory limits of every ORDER BY kernel, set once per device (h2tap_open).
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

cudaError_t set_attributes_sort(int num_sms) {
    static const void *const kKernels[] = {
        (const void *)bucket_local_emit_kernel<kLsCapLarge, kLsCapSmall>,
        (const void *)bucket_local_emit_kernel<kLsCapLarge, kObCap, true>,
        (const void *)bucket_local_emit_kernel<kLsCapSmall, 0>,
        (const void *)bucket_local_emit_kernel<kObCap, 0, true>,
        (const void *)bucket_scatter_kernel,
        (const void *)digit_scan_kernel,
        (const void *)field_keys_kernel,
        (const void *)hist_kernel,
        (const void *)iota_kernel,
        (const void *)ob_hist_kernel,
        (const void *)ob_scan_kernel,
        (const void *)ob_scatter_kernel,
        (const void *)permute_kernel,
        (const void *)q18_dist_meta_kernel,
        (const void *)q18_dist_publish_kernel,
        (const void *)q18_dist_route_kernel,
        (const void *)q18_dist_send_kernel,
        (const void *)q18_keys_hist_kernel,
        (const void *)q18_plan_kernel,
        (const void *)scatter_kernel,
        (const void *)q18_acc_stats_kernel,
        (const void *)q18_having_rec_kernel<false>,
        (const void *)q18_having_rec_kernel<true>,
        (const void *)q18_acc_hist_kernel,
        (const void *)ob_scatter_rec_kernel,
        (const void *)l2_touch_kernel,
        (const void *)carry_large_emit_kernel};
    const cudaError_t le = force_load(kKernels, sizeof kKernels / sizeof kKernels[0]);
    if (le != cudaSuccess) return le;

    const int G = ob_grid(num_sms);
    const struct { const void *f; int bytes; } a[] = {
        {(const void *)bucket_local_emit_kernel<kLsCapSmall, 0>, (int)sizeof(LsSmem<kLsCapSmall>)},
        {(const void *)bucket_local_emit_kernel<kLsCapLarge, kLsCapSmall>, (int)sizeof(LsSmem<kLsCapLarge>)},
        {(const void *)q18_keys_hist_kernel, 4 << kBucketMaxBits},
        {(const void *)bucket_scatter_kernel, 4 << kBucketMaxBits},
        {(const void *)bucket_local_emit_kernel<kObCap, 0, true>, (int)kObSmem},
        {(const void *)bucket_local_emit_kernel<kLsCapLarge, kObCap, true>, (int)kObSmemLarge},
        {(const void *)ob_hist_kernel, 4 << kBucketMaxBits},
        {(const void *)ob_scatter_kernel, 4 << kBucketMaxBits},
        {(const void *)ob_scan_kernel, 4 * std::max(32 * G, 1 << kBucketMaxBits)},
        {(const void *)q18_dist_route_kernel, 4 << kBucketMaxBits},
        {(const void *)q18_having_rec_kernel<false>, 4 << kBucketMaxBits},
        {(const void *)q18_having_rec_kernel<true>, 4 << kBucketMaxBits},
        {(const void *)q18_acc_hist_kernel, 4 << kBucketMaxBits},
        {(const void *)carry_large_emit_kernel, (int)kLgSmem},
        {(const void *)ob_scatter_rec_kernel, 4 << kBucketMaxBits},
    };
    for (const auto &x : a) {
        const cudaError_t e = cudaFuncSetAttribute(x.f, cudaFuncAttributeMaxDynamicSharedMemorySize, x.bytes);
        if (e != cudaSuccess) return e;
    }
    return cudaSuccess;
}

}  // namespace h2tap
