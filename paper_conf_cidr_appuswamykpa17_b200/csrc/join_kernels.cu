// join_kernels.cu — K3 hash build, K4 probe + group-join aggregation, K5 HAVING + compaction +
// customer probe + gather, for CH Q18 (customer ⋈ orders ⋈ order_line, GROUP BY, HAVING) on sm_100a.
//
// The paper gives no join algorithm (hash joins on accelerators appear only as related work,
// PAPER.md L1224-1227); its runtime hands kernels the snapshot's column pointers (L568-570).
// Design: open-addressing hash tables with 16-byte slots {packed key, row},
// linear probing, capacity a power of two >= 2n, insert by 64-bit atomicCAS. Q18's GROUP BY
// key (o_id, o_w_id, o_d_id, c_id, c_last, o_entry_d, o_ol_cnt) is functionally determined by
// the orders primary key once orders and customer PKs are unique (checked: EDUPKEY), so the
// group-by collapses onto the orders row: acc[orders row] += (amount, 1).
#include <cstdint>
#include <cuda_runtime.h>

#include "kernels.cuh"

namespace h2tap {
namespace {

constexpr unsigned kFull = 0xffffffffu;
constexpr unsigned int kNone = 0xffffffffu;

__device__ __forceinline__ unsigned long long fmix64(unsigned long long k) {
    k ^= k >> 33; k *= 0xff51afd7ed558ccdull; k ^= k >> 33; k *= 0xc4ceb9fe1a85ec53ull; k ^= k >> 33;
    return k;
}

// (w, d, id) -> 64-bit key, order-preserving on the supported domain (R16).
__device__ __forceinline__ bool pack_key(int w, int d, int id, unsigned long long &k) {
    k = ((unsigned long long)(unsigned)w << 40) | ((unsigned long long)(unsigned)d << 32) |
        (unsigned long long)(unsigned)id;
    return ((unsigned)w < (1u << 23)) & ((unsigned)d < 256u) & (id >= 0);
}

__device__ __forceinline__ void ht_insert(HtSlot *ht, unsigned long long mask, unsigned long long key,
                                          unsigned int row, unsigned int *err, unsigned int dupbit) {
    unsigned long long h = fmix64(key) & mask;
    while (true) {
        const unsigned long long prev = atomicCAS(&ht[h].key, kEmpty, key);
        if (prev == kEmpty) { ht[h].row = row; return; }
        if (prev == key) { atomicOr(err, dupbit); return; }
        h = (h + 1) & mask;
    }
}

__device__ __forceinline__ unsigned int ht_probe(const HtSlot *ht, unsigned long long mask,
                                                 unsigned long long key) {
    unsigned long long h = fmix64(key) & mask;
    while (true) {
        const ulonglong2 s = __ldcg(reinterpret_cast<const ulonglong2 *>(ht + h));
        if (s.x == key) return (unsigned int)s.y;
        if (s.x == kEmpty) return kNone;
        h = (h + 1) & mask;
    }
}

// ------------------------------------------------------------------- init --
__global__ void q18_init_kernel(Q18Scratch s, uint64_t n_orders) {
    const uint64_t total = s.cap_o + s.cap_c + n_orders;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    const ulonglong2 empty = make_ulonglong2(kEmpty, 0ull), zero = make_ulonglong2(0ull, 0ull);
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < total; i += stride) {
        if (i < s.cap_o) reinterpret_cast<ulonglong2 *>(s.ht_o)[i] = empty;
        else if (i < s.cap_o + s.cap_c) reinterpret_cast<ulonglong2 *>(s.ht_c)[i - s.cap_o] = empty;
        else reinterpret_cast<ulonglong2 *>(s.acc)[i - s.cap_o - s.cap_c] = zero;
    }
    if (blockIdx.x == 0 && threadIdx.x == 0) {
        *s.err = 0;
        *s.nout = 0;
        Q18Stats st;
        st.amt_min = INT64_MAX; st.amt_max = INT64_MIN; st.ent_min = INT64_MAX; st.ent_max = INT64_MIN;
        st.w_min = INT32_MAX; st.w_max = INT32_MIN; st.d_min = INT32_MAX; st.d_max = INT32_MIN;
        st.o_min = INT32_MAX; st.o_max = INT32_MIN; st.pad0 = st.pad1 = 0;
        *s.stats = st;
    }
}

// ------------------------------------------------------------------ K3 build --
__global__ void q18_build_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                                 const int32_t *__restrict__ o_id, uint64_t n_o,
                                 const int32_t *__restrict__ c_w, const int32_t *__restrict__ c_d,
                                 const int32_t *__restrict__ c_id, uint64_t n_c, Q18Scratch s) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    const unsigned long long mo = s.cap_o - 1, mc = s.cap_c - 1;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n_o + n_c; i += stride) {
        unsigned long long k;
        if (i < n_o) {
            if (!pack_key(o_w[i], o_d[i], o_id[i], k)) { atomicOr(s.err, kErrDomain); continue; }
            ht_insert(s.ht_o, mo, k, (unsigned int)i, s.err, kErrDupOrders);
        } else {
            const uint64_t j = i - n_o;
            if (!pack_key(c_w[j], c_d[j], c_id[j], k)) { atomicOr(s.err, kErrDomain); continue; }
            ht_insert(s.ht_c, mc, k, (unsigned int)j, s.err, kErrDupCustomer);
        }
    }
}

// ------------------------------------------------------- K4 probe + group-join --
// One warp iteration covers 32 consecutive order_line rows (coalesced 4 B / 8 B loads).
// Lines of one order are usually contiguous, so equal keys form runs: a segmented inclusive
// scan (shuffles) sums each run, the run head probes the orders table once, and the run tail
// issues the two atomics — ~3 runs per 32 rows instead of 32 probes and 64 atomics.
constexpr int kProbeThreads = 256;
constexpr int kProbeUnroll = 2;

__global__ void __launch_bounds__(kProbeThreads)
q18_probe_kernel(const int32_t *__restrict__ ol_w, const int32_t *__restrict__ ol_d,
                 const int32_t *__restrict__ ol_o, const int64_t *__restrict__ ol_amt, uint64_t n,
                 Q18Scratch s) {
    const int lane = threadIdx.x & 31;
    const uint64_t gwarp = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    const unsigned long long mask = s.cap_o - 1;
    const unsigned le_mask = 0xffffffffu >> (31 - lane);  // lanes 0..lane
    for (uint64_t base = gwarp * 32 * kProbeUnroll; base < n; base += nwarps * 32 * kProbeUnroll) {
        unsigned long long key[kProbeUnroll];
        long long amt[kProbeUnroll];
#pragma unroll
        for (int u = 0; u < kProbeUnroll; ++u) {
            const uint64_t i = base + u * 32 + lane;
            key[u] = kEmpty;  // invalid rows (tail / out of domain) never match
            amt[u] = 0;
            if (i < n) {
                unsigned long long k;
                if (pack_key(__ldcs(ol_w + i), __ldcs(ol_d + i), __ldcs(ol_o + i), k)) key[u] = k;
                amt[u] = __ldcs(ol_amt + i);
            }
        }
#pragma unroll
        for (int u = 0; u < kProbeUnroll; ++u) {
            const unsigned long long prev = __shfl_up_sync(kFull, key[u], 1);
            const bool head = lane == 0 || key[u] != prev;
            const unsigned heads = __ballot_sync(kFull, head);
            const int leader = 31 - __clz(heads & le_mask);
            long long sum = amt[u];
#pragma unroll
            for (int off = 1; off < 32; off <<= 1) {
                const long long t = __shfl_up_sync(kFull, sum, off);
                if (lane - off >= leader) sum += t;
            }
            const bool tail = lane == 31 || ((heads >> (lane + 1)) & 1u);
            unsigned int row = kNone;
            if (head && key[u] != kEmpty) row = ht_probe(s.ht_o, mask, key[u]);
            row = __shfl_sync(kFull, row, leader);
            if (tail && row != kNone) {
                atomicAdd(reinterpret_cast<unsigned long long *>(&s.acc[row].sum),
                          (unsigned long long)sum);
                atomicAdd(&s.acc[row].cnt, (unsigned int)(lane - leader + 1));
            }
        }
    }
}

// ---------------------------------------- K5 HAVING + customer probe + compaction --
constexpr int kHavingThreads = 256;

__device__ __forceinline__ long long wmin64(long long v) {
    for (int o = 16; o; o >>= 1) { long long t = __shfl_xor_sync(kFull, v, o); v = t < v ? t : v; }
    return v;
}
__device__ __forceinline__ long long wmax64(long long v) {
    for (int o = 16; o; o >>= 1) { long long t = __shfl_xor_sync(kFull, v, o); v = t > v ? t : v; }
    return v;
}
__device__ __forceinline__ int wmin32(int v) { return __reduce_min_sync(kFull, v); }
__device__ __forceinline__ int wmax32(int v) { return __reduce_max_sync(kFull, v); }

struct StatAcc {
    long long amin = INT64_MAX, amax = INT64_MIN, emin = INT64_MAX, emax = INT64_MIN;
    int wmin = INT32_MAX, wmax = INT32_MIN, dmin = INT32_MAX, dmax = INT32_MIN;
    int omin = INT32_MAX, omax = INT32_MIN;
    __device__ void add(long long a, long long e, int w, int d, int o) {
        amin = a < amin ? a : amin; amax = a > amax ? a : amax;
        emin = e < emin ? e : emin; emax = e > emax ? e : emax;
        wmin = min(wmin, w); wmax = max(wmax, w); dmin = min(dmin, d); dmax = max(dmax, d);
        omin = min(omin, o); omax = max(omax, o);
    }
    __device__ void flush(Q18Stats *st) {  // warp-reduce, lane 0 issues the atomics
        amin = wmin64(amin); amax = wmax64(amax); emin = wmin64(emin); emax = wmax64(emax);
        wmin = wmin32(wmin); wmax = wmax32(wmax); dmin = wmin32(dmin); dmax = wmax32(dmax);
        omin = wmin32(omin); omax = wmax32(omax);
        if ((threadIdx.x & 31) == 0 && amin <= amax) {
            atomicMin(&st->amt_min, amin); atomicMax(&st->amt_max, amax);
            atomicMin(&st->ent_min, emin); atomicMax(&st->ent_max, emax);
            atomicMin(&st->w_min, wmin); atomicMax(&st->w_max, wmax);
            atomicMin(&st->d_min, dmin); atomicMax(&st->d_max, dmax);
            atomicMin(&st->o_min, omin); atomicMax(&st->o_max, omax);
        }
    }
};

__global__ void __launch_bounds__(kHavingThreads)
q18_having_kernel(const int32_t *__restrict__ o_w, const int32_t *__restrict__ o_d,
                  const int32_t *__restrict__ o_id, const int32_t *__restrict__ o_c,
                  const int32_t *__restrict__ o_cnt, const int64_t *__restrict__ o_ent, uint64_t n,
                  const int32_t *__restrict__ c_last, long long having, Q18Scratch s) {
    const int lane = threadIdx.x & 31;
    const uint64_t gwarp = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
    const uint64_t nwarps = ((uint64_t)gridDim.x * blockDim.x) >> 5;
    const unsigned long long mc = s.cap_c - 1;
    StatAcc stat;
    for (uint64_t base = gwarp * 32; base < n; base += nwarps * 32) {
        const uint64_t r = base + lane;
        bool pass = false;
        unsigned int crow = kNone;
        long long sum = 0;
        int w = 0, d = 0, c = 0;
        if (r < n) {
            const ulonglong2 a = __ldcs(reinterpret_cast<const ulonglong2 *>(s.acc + r));
            sum = (long long)a.x;
            const unsigned int cnt = (unsigned int)a.y;
            // inner join: a group exists only with >= 1 order_line row; HAVING SUM > having
            if (cnt > 0 && sum > having) {
                w = o_w[r]; d = o_d[r]; c = o_c[r];
                unsigned long long k;
                if (pack_key(w, d, c, k)) crow = ht_probe(s.ht_c, mc, k);  // c ⋈ o
                pass = crow != kNone;
            }
        }
        const unsigned ball = __ballot_sync(kFull, pass);
        if (!ball) continue;
        unsigned long long basepos = 0;
        if (lane == 0) basepos = atomicAdd(s.nout, (unsigned long long)__popc(ball));
        basepos = __shfl_sync(kFull, basepos, 0);
        if (pass) {
            const uint64_t p = basepos + __popc(ball & ((1u << lane) - 1u));
            const int oid = o_id[r];
            const long long ent = o_ent[r];
            s.un.c_last[p] = c_last[crow];
            s.un.c_id[p] = c;
            s.un.o_id[p] = oid;
            s.un.o_entry_d[p] = ent;
            s.un.o_ol_cnt[p] = o_cnt[r];
            s.un.amount_sum[p] = sum;
            s.un.o_w_id[p] = w;
            s.un.o_d_id[p] = d;
            stat.add(sum, ent, w, d, oid);
        }
    }
    stat.flush(s.stats);
}

__global__ void q18_stats_kernel(Q18Cols cols, uint64_t n, Q18Stats *st) {
    StatAcc stat;
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
        stat.add(cols.amount_sum[i], cols.o_entry_d[i], cols.o_w_id[i], cols.o_d_id[i], cols.o_id[i]);
    stat.flush(st);
}

__global__ void fill_u64_kernel(unsigned long long *p, uint64_t n, unsigned long long v) {
    const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
    for (uint64_t i = (uint64_t)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) p[i] = v;
}

unsigned grid_for(uint64_t work, int threads, int num_sms, int per_sm) {
    uint64_t want = (work + threads - 1) / threads;
    uint64_t cap = (uint64_t)num_sms * per_sm;
    if (want > cap) want = cap;
    return want ? (unsigned)want : 1u;
}

}  // namespace

void launch_q18_init(const Q18Scratch &s, uint64_t n_orders, cudaStream_t st) {
    int dev = 0, sms = 148;
    cudaGetDevice(&dev);
    cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, dev);
    q18_init_kernel<<<grid_for(s.cap_o + s.cap_c + n_orders, 256, sms, 8), 256, 0, st>>>(s, n_orders);
    count_launches(1);
}

void launch_q18_build(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, uint64_t n_o,
                      const int32_t *c_w, const int32_t *c_d, const int32_t *c_id, uint64_t n_c,
                      const Q18Scratch &s, int num_sms, cudaStream_t st) {
    q18_build_kernel<<<grid_for(n_o + n_c, 256, num_sms, 8), 256, 0, st>>>(o_w, o_d, o_id, n_o, c_w,
                                                                         c_d, c_id, n_c, s);
    count_launches(1);
}

void launch_q18_probe(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o,
                      const int64_t *ol_amt, uint64_t n_ol, const Q18Scratch &s, int num_sms,
                      cudaStream_t st) {
    q18_probe_kernel<<<grid_for((n_ol + kProbeUnroll - 1) / kProbeUnroll, kProbeThreads, num_sms, 8),
                       kProbeThreads, 0, st>>>(ol_w, ol_d, ol_o, ol_amt, n_ol, s);
    count_launches(1);
}

void launch_q18_having(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id,
                       const int32_t *o_c, const int32_t *o_cnt, const int64_t *o_ent,
                       uint64_t n_o, const int32_t *c_last, int64_t having,
                       const Q18Scratch &s, int num_sms, cudaStream_t st) {
    q18_having_kernel<<<grid_for(n_o, kHavingThreads, num_sms, 8), kHavingThreads, 0, st>>>(
        o_w, o_d, o_id, o_c, o_cnt, o_ent, n_o, c_last, having, s);
        count_launches(1);
}

void launch_q18_stats(const Q18Cols &cols, uint64_t n, Q18Stats *stats, int num_sms,
                      cudaStream_t st) {
    q18_stats_kernel<<<grid_for(n, 256, num_sms, 4), 256, 0, st>>>(cols, n, stats);
    count_launches(1);
}

void launch_fill_u64(unsigned long long *p, uint64_t n, unsigned long long v, cudaStream_t st) {
    fill_u64_kernel<<<grid_for(n, 256, 148, 8), 256, 0, st>>>(p, n, v);
    count_launches(1);
}

}  // namespace h2tap
