// sort_kernels.cu — a8 finalize for CH Q18: ORDER BY amount_sum DESC, o_entry_d ASC, then the
// (o_w_id, o_d_id, o_id) tie-break that makes the order total (R11).
//
// The three sort fields are mapped to unsigned integers whose widths come from the result's
// min/max (HAVING kernel statistics): a = max - amount_sum (DESC), e = o_entry_d - min,
// r = dense rank of (w, d, o). Their concatenation a|e|r is the exact composite key.
//  * main path: sort (top 64 bits of a|e|r, row id) pairs with a bucket sort (partition by the
//    top key bits, bitonic sort per bucket in shared memory). If a|e|r fits 64 bits the keys are
//    distinct and the order is exact; otherwise runs of equal 64-bit prefixes are ordered by the
//    full tuple (tie-fix; runs are a handful of rows on realistic data).
//  * exact fallback (a run > 32 rows or a bucket > shared memory): one stable LSD radix sort of
//    (key, row) pairs per field, r then e then a. Radix pass = per-tile digit histogram ->
//    per-digit scan -> stable scatter; keys travel with their row ids.
#include <cstdint>
#include <cuda_runtime.h>

#include "kernels.cuh"

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
__device__ __forceinline__ unsigned long long field_a(const Q18Row &r, const Q18SortSpec &sp) {
    return (unsigned long long)sp.amt_max - (unsigned long long)r.amount_sum;  // DESC
}
__device__ __forceinline__ unsigned long long field_e(const Q18Row &r, const Q18SortSpec &sp) {
    return (unsigned long long)r.o_entry_d - (unsigned long long)sp.ent_min;
}
__device__ __forceinline__ unsigned long long field_r(const Q18Row &r, const Q18SortSpec &sp) {
    const unsigned long long w = (unsigned)(r.o_w_id - sp.w_min);
    const unsigned long long d = (unsigned)(r.o_d_id - sp.d_min);
    const unsigned long long o = (unsigned)(r.o_id - sp.o_min);
    return (w * (unsigned long long)sp.nd + d) * (unsigned long long)sp.no + o;
}

// top `prefix_bits` bits of the concatenation (a | e | r) with widths (bits_a, bits_e, bits_r)
__device__ __forceinline__ unsigned long long prefix_key(const Q18Row &r, const Q18SortSpec &sp) {
    const unsigned long long f[3] = {field_a(r, sp), field_e(r, sp), field_r(r, sp)};
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

__global__ void sort_keys_kernel(const Q18Row *__restrict__ rows, uint64_t n, Q18SortSpec sp,
                                 unsigned long long *__restrict__ k, unsigned int *__restrict__ v) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        k[i] = prefix_key(rows[i], sp);
        v[i] = (unsigned int)i;
    }
}

// full ORDER BY comparison: amount_sum DESC, o_entry_d, o_w_id, o_d_id, o_id
__device__ __forceinline__ bool row_less(const Q18Row &x, const Q18Row &y) {
    if (x.amount_sum != y.amount_sum) return x.amount_sum > y.amount_sum;
    if (x.o_entry_d != y.o_entry_d) return x.o_entry_d < y.o_entry_d;
    if (x.o_w_id != y.o_w_id) return x.o_w_id < y.o_w_id;
    if (x.o_d_id != y.o_d_id) return x.o_d_id < y.o_d_id;
    return x.o_id < y.o_id;
}

constexpr int kMaxRun = 32;

__global__ void tiefix_kernel(const Q18Row *__restrict__ rows, const unsigned long long *__restrict__ k,
                              unsigned int *__restrict__ v, uint64_t n, unsigned int *flag) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        const unsigned long long ki = k[i];
        if (i > 0 && k[i - 1] == ki) continue;         // not the head of a run
        if (i + 1 >= n || k[i + 1] != ki) continue;    // run of one
        uint64_t j = i + 1;
        while (j < n && k[j] == ki && j - i <= kMaxRun) ++j;
        if (j - i > kMaxRun) { atomicOr(flag, 1u); continue; }
        unsigned int idx[kMaxRun];
        const int len = (int)(j - i);
        for (int t = 0; t < len; ++t) idx[t] = v[i + t];
        for (int t = 1; t < len; ++t) {  // insertion sort by the full tuple
            const unsigned int x = idx[t];
            const Q18Row rx = rows[x];
            int u = t - 1;
            while (u >= 0 && row_less(rx, rows[idx[u]])) { idx[u + 1] = idx[u]; --u; }
            idx[u + 1] = x;
        }
        for (int t = 0; t < len; ++t) v[i + t] = idx[t];
    }
}

__global__ void field_keys_kernel(const Q18Row *__restrict__ rows, const unsigned int *__restrict__ vals,
                                  uint64_t n, int field, Q18SortSpec sp,
                                  unsigned long long *__restrict__ k) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
        const Q18Row r = rows[vals[i]];
        k[i] = field == 0 ? field_r(r, sp) : field == 1 ? field_e(r, sp) : field_a(r, sp);
    }
}

__global__ void iota_kernel(unsigned int *v, uint64_t n) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
        v[i] = (unsigned int)i;
}

// Gather one 40-byte row per output position, write the eight SoA columns coalesced.
__global__ void permute_kernel(const Q18Row *__restrict__ rows, const unsigned int *__restrict__ perm,
                               uint64_t n, Q18Cols dst) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t j = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; j < n; j += stride) {
        const Q18Row r = rows[perm ? perm[j] : j];
        dst.c_last[j] = r.c_last;
        dst.c_id[j] = r.c_id;
        dst.o_id[j] = r.o_id;
        dst.o_entry_d[j] = r.o_entry_d;
        dst.o_ol_cnt[j] = r.o_ol_cnt;
        dst.amount_sum[j] = r.amount_sum;
        dst.o_w_id[j] = r.o_w_id;
        dst.o_d_id[j] = r.o_d_id;
    }
}

unsigned grid_cap(uint64_t work, int threads, int num_sms, int per_sm) {
    uint64_t want = (work + threads - 1) / threads;
    uint64_t cap = (uint64_t)num_sms * per_sm;
    if (want > cap) want = cap;
    return want ? (unsigned)want : 1u;
}

}  // namespace

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

void launch_q18_sort_keys(const Q18Row *rows, uint64_t n, const Q18SortSpec &spec,
                          const SortPairs &s, int num_sms, cudaStream_t st) {
    sort_keys_kernel<<<grid_cap(n, 256, num_sms, 8), 256, 0, st>>>(rows, n, spec, s.k[0], s.v[0]);
    count_launches(1);
}

void launch_q18_tiefix(const Q18Row *rows, const unsigned long long *keys, unsigned int *vals,
                       uint64_t n, unsigned int *flag, int num_sms, cudaStream_t st) {
    tiefix_kernel<<<grid_cap(n, 256, num_sms, 8), 256, 0, st>>>(rows, keys, vals, n, flag);
    count_launches(1);
}

void launch_q18_field_keys(const Q18Row *rows, const unsigned int *vals, uint64_t n, int field,
                           const Q18SortSpec &spec, unsigned long long *keys, int num_sms,
                           cudaStream_t st) {
    field_keys_kernel<<<grid_cap(n, 256, num_sms, 8), 256, 0, st>>>(rows, vals, n, field, spec, keys);
    count_launches(1);
}

void launch_iota(unsigned int *v, uint64_t n, int num_sms, cudaStream_t st) {
    iota_kernel<<<grid_cap(n, 256, num_sms, 8), 256, 0, st>>>(v, n);
    count_launches(1);
}

void launch_q18_permute(const Q18Row *rows, const unsigned int *perm, uint64_t n,
                        const Q18Cols &dst, int num_sms, cudaStream_t st) {
    permute_kernel<<<grid_cap(n, 256, num_sms, 8), 256, 0, st>>>(rows, perm, n, dst);
    count_launches(1);
}

}  // namespace h2tap

// ============================================================ bucket sort ===
// Main ORDER BY path: the result (a few million 12-byte pairs) fits in L2, so
// one partition pass by the top key bits plus a shared-memory sort per bucket replaces the
// 6 LSD passes. Buckets are not stable internally; equal full prefixes are ordered afterwards by
// the tie-fix kernel (which sorts runs of equal prefix by the full tuple) — so the result is the
// same total order as the LSD path.
namespace h2tap {
namespace {

constexpr int kBkThreads = 256;
constexpr int kBkSmemBins = 8192;  // max buckets counted in shared memory per block

__global__ void __launch_bounds__(kBkThreads)
bucket_hist_kernel(const unsigned long long *__restrict__ key, uint64_t n, int shift, int nb,
                   unsigned int *__restrict__ count) {
    extern __shared__ unsigned int h[];
    for (int i = threadIdx.x; i < nb; i += kBkThreads) h[i] = 0;
    __syncthreads();
    const uint64_t stride = (uint64_t)gridDim.x * kBkThreads;
    for (uint64_t i = (uint64_t)blockIdx.x * kBkThreads + threadIdx.x; i < n; i += stride)
        atomicAdd(&h[(unsigned int)(__ldcg(key + i) >> shift)], 1u);
    __syncthreads();
    for (int i = threadIdx.x; i < nb; i += kBkThreads)
        if (h[i]) atomicAdd(count + i, h[i]);
}

// exclusive scan of nb bucket counts -> offset[] and cursor[]; max bucket size -> count[nb]
__global__ void __launch_bounds__(1024) bucket_scan_kernel(unsigned int *__restrict__ count, int nb,
                                                           unsigned int *__restrict__ offset,
                                                           unsigned int *__restrict__ cursor) {
    __shared__ unsigned int wsum[32];
    __shared__ unsigned int carry_s;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    unsigned int carry = 0, mx = 0;
    for (int r0 = 0; r0 < nb; r0 += 1024) {
        const int i = r0 + threadIdx.x;
        const unsigned int v = i < nb ? count[i] : 0u;
        mx = max(mx, v);
        unsigned int x = v;
#pragma unroll
        for (int o = 1; o < 32; o <<= 1) {
            const unsigned int t = __shfl_up_sync(kFull, x, o);
            if (lane >= o) x += t;
        }
        if (lane == 31) wsum[warp] = x;
        __syncthreads();
        if (warp == 0) {
            unsigned int y = wsum[lane];
#pragma unroll
            for (int o = 1; o < 32; o <<= 1) {
                const unsigned int t = __shfl_up_sync(kFull, y, o);
                if (lane >= o) y += t;
            }
            wsum[lane] = y;
            if (lane == 31) carry_s = y;
        }
        __syncthreads();
        const unsigned int ex = carry + (warp ? wsum[warp - 1] : 0u) + x - v;
        if (i < nb) { offset[i] = ex; cursor[i] = ex; }
        carry += carry_s;
        __syncthreads();
    }
    mx = __reduce_max_sync(kFull, mx);
    if (lane == 0) wsum[warp] = mx;
    __syncthreads();
    if (threadIdx.x == 0) {
        unsigned int m = 0;
        for (int w = 0; w < 32; ++w) m = max(m, wsum[w]);
        offset[nb] = carry;
        count[nb] = m;
    }
}

// scatter into buckets: per-block shared histogram reserves one global range per bucket
__global__ void __launch_bounds__(kBkThreads)
bucket_scatter_kernel(const unsigned long long *__restrict__ kin, const unsigned int *__restrict__ vin,
                      unsigned long long *__restrict__ kout, unsigned int *__restrict__ vout, uint64_t n,
                      int shift, int nb, unsigned int *__restrict__ cursor, uint64_t per_block) {
    extern __shared__ unsigned int h[];  // [nb] local counts -> local cursors
    for (int i = threadIdx.x; i < nb; i += kBkThreads) h[i] = 0;
    __syncthreads();
    const uint64_t lo = (uint64_t)blockIdx.x * per_block;
    const uint64_t hi = lo + per_block < n ? lo + per_block : n;
    for (uint64_t i = lo + threadIdx.x; i < hi; i += kBkThreads)
        atomicAdd(&h[(unsigned int)(__ldcg(kin + i) >> shift)], 1u);
    __syncthreads();
    for (int i = threadIdx.x; i < nb; i += kBkThreads)
        if (h[i]) h[i] = atomicAdd(cursor + i, h[i]);  // base of this block's range in bucket i
    __syncthreads();
    for (uint64_t i = lo + threadIdx.x; i < hi; i += kBkThreads) {
        const unsigned long long k = __ldcg(kin + i);
        const unsigned int p = atomicAdd(&h[(unsigned int)(k >> shift)], 1u);
        kout[p] = k;
        vout[p] = __ldcg(vin + i);
    }
}

// one block per bucket: load into shared memory, bitonic sort by key, write back
__global__ void __launch_bounds__(kBkThreads)
bucket_local_sort_kernel(unsigned long long *__restrict__ k, unsigned int *__restrict__ v,
                         const unsigned int *__restrict__ offset, int nb, unsigned int *flag) {
    extern __shared__ unsigned long long sk[];  // [kBucketCap] keys, then [kBucketCap] values
    unsigned int *sv = reinterpret_cast<unsigned int *>(sk + kBucketCap);
    for (int b = blockIdx.x; b < nb; b += gridDim.x) {
        const unsigned int lo = offset[b], cnt = offset[b + 1] - lo;
        if (cnt <= 1) continue;
        if (cnt > (unsigned)kBucketCap) {
            if (threadIdx.x == 0) atomicOr(flag, 2u);
            continue;
        }
        unsigned int m = 2;
        while (m < cnt) m <<= 1;
        for (unsigned int i = threadIdx.x; i < m; i += kBkThreads) {
            sk[i] = i < cnt ? k[lo + i] : ~0ull;
            sv[i] = i < cnt ? v[lo + i] : 0u;
        }
        __syncthreads();
        for (unsigned int size = 2; size <= m; size <<= 1) {
            for (unsigned int stride = size >> 1; stride > 0; stride >>= 1) {
                for (unsigned int t = threadIdx.x; t < m / 2; t += kBkThreads) {
                    const unsigned int i = 2 * t - (t & (stride - 1));
                    const unsigned int j = i + stride;
                    const bool up = (i & size) == 0;
                    const unsigned long long a = sk[i], c = sk[j];
                    if ((a > c) == up) {
                        sk[i] = c; sk[j] = a;
                        const unsigned int tv = sv[i]; sv[i] = sv[j]; sv[j] = tv;
                    }
                }
                __syncthreads();
            }
        }
        for (unsigned int i = threadIdx.x; i < cnt; i += kBkThreads) {
            k[lo + i] = sk[i];
            v[lo + i] = sv[i];
        }
        __syncthreads();
    }
}

}  // namespace

void bucket_sort_pairs(uint64_t n, int bits, int bucket_bits, const BucketSort &s, unsigned int *flag,
                       int num_sms, cudaStream_t st) {
    if (bucket_bits > bits) bucket_bits = bits;
    if (bucket_bits > 13) bucket_bits = 13;  // shared histogram of <= 8192 bins
    const int nb = 1 << bucket_bits;
    const int shift = bits - bucket_bits;
    static bool init = false;
    if (!init) {
        cudaFuncSetAttribute(bucket_local_sort_kernel, cudaFuncAttributeMaxDynamicSharedMemorySize,
                             kBucketCap * 12);
        init = true;
    }
    cudaMemsetAsync(s.count, 0, sizeof(unsigned int) * (nb + 1), st);
    uint64_t hb = (n + kBkThreads * 16 - 1) / (kBkThreads * 16);
    if (hb > (uint64_t)num_sms * 4) hb = (uint64_t)num_sms * 4;
    if (!hb) hb = 1;
    bucket_hist_kernel<<<(unsigned)hb, kBkThreads, nb * 4, st>>>(s.k[0], n, shift, nb, s.count);
    count_launches(1);
    bucket_scan_kernel<<<1, 1024, 0, st>>>(s.count, nb, s.offset, s.cursor);
    count_launches(1);
    const uint64_t per_block = 16384;
    const uint64_t sb = (n + per_block - 1) / per_block;
    bucket_scatter_kernel<<<(unsigned)(sb ? sb : 1), kBkThreads, nb * 4, st>>>(
        s.k[0], s.v[0], s.k[1], s.v[1], n, shift, nb, s.cursor, per_block);
    count_launches(1);
    unsigned lb = (unsigned)nb < (unsigned)num_sms * 16 ? (unsigned)nb : (unsigned)num_sms * 16;
    bucket_local_sort_kernel<<<lb, kBkThreads, kBucketCap * 12, st>>>(s.k[1], s.v[1], s.offset, nb, flag);
    count_launches(1);
}

}  // namespace h2tap
