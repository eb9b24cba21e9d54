// kernels.cuh — internal interface between the engine (engine.cu) and the sm_100a kernels.
// Product code only; never included by oracle/.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>
#include <utility>

namespace h2tap {

constexpr int64_t kNullTs = INT64_MIN;  // SQL NULL of ol_delivery_d (R5)

// ----------------------------------------------------------------- Q6 (K1) --
// revenue = SUM(amount) over rows with d_lo <= delivery < d_hi AND q_lo <= qty <= q_hi.
// out[0] = revenue, out[1] = qualifying row count. Partials: one {sum,cnt} per block,
// reduced by the last block to finish (no memset needed; the counter self-resets).
struct Q6Scratch {
    long long *block_part;      // [2 * max_blocks]
    unsigned int *done_counter; // [1], zero-initialised once at allocation
    long long *out;             // [2]
    long long *host_out;        // [2] mapped pinned host memory (also written), or null
};
int q6_max_blocks(int num_sms);
void launch_q6(const int64_t *deliv, const int32_t *qty, const int64_t *amt, uint64_t n,
               int64_t d_lo, int64_t d_hi, int64_t q_lo, int64_t q_hi, const Q6Scratch &s,
               int num_sms, cudaStream_t st);
// same result, TMA-bulk (cp.async.bulk) staged through a shared-memory ring, one block per SM
void launch_q6_tma(const int64_t *deliv, const int32_t *qty, const int64_t *amt, uint64_t n,
                   int64_t d_lo, int64_t d_hi, int64_t q_lo, int64_t q_hi, const Q6Scratch &s,
                   int num_sms, cudaStream_t st);

// ----------------------------------------------------------------- Q1 (K2) --
// GROUP BY ol_number over rows with delivery > cutoff; per group (count, sum_qty, sum_amount).
// Keys in [0, kQ1Dense) are aggregated in thread-private shared memory; other keys go through
// warp-aggregated shared-memory atomics into a per-block hash table, then a global hash table.
constexpr int kQ1Dense = 16;
constexpr int kQ1GlobalSlots = 1 << 16;  // max distinct groups per rank
constexpr unsigned kQ1GlobalUsed = 2u;    // Q1Scratch::flags: a group entered the global table
constexpr unsigned kQ1Emitted = 4u;       // Q1Scratch::flags: the compact wrote the output
struct Q1Group { long long key; long long cnt, qty, amt; };  // 32 B, compacted group
struct Q1Scratch {
    unsigned long long *dense;   // [kQ1Dense * 3]: cnt, qty, amt per dense key
    unsigned long long *gtag;    // [kQ1GlobalSlots]: 0 = empty, else (1<<32 | (u32)key)
    unsigned long long *gacc;    // [kQ1GlobalSlots * 3]
    unsigned int *flags;         // [1]: bit0 = global table full, kQ1GlobalUsed, kQ1Emitted
    Q1Group *groups;             // [kQ1GlobalSlots + kQ1Dense] compacted groups
    unsigned long long *ngroups; // [1]
    // output (ranked by key)
    int32_t *o_key; long long *o_qty, *o_amt, *o_cnt; double *o_avg_qty, *o_avg_amt;
    unsigned long long *host_small;  // mapped pinned: emit writes {ngroups, flags} here, or null
};
void launch_q1_reset(const Q1Scratch &s, cudaStream_t st);
void launch_q1(const int32_t *number, const int64_t *deliv, const int32_t *qty,
               const int64_t *amt, uint64_t n, int64_t cutoff, const Q1Scratch &s, int num_sms,
               cudaStream_t st);
void launch_q1_tma(const int32_t *number, const int64_t *deliv, const int32_t *qty,
                   const int64_t *amt, uint64_t n, int64_t cutoff, const Q1Scratch &s, int num_sms,
                   cudaStream_t st);  // same result, TMA-bulk staged, one block per SM
// Shared scan of a batch's Q6 and Q1: one TMA pass over Q1's four columns fills
// Q1's tables (as launch_q1_tma) and writes Q6's {revenue, count} (as launch_q6_tma).
void launch_q61_tma(const int32_t *number, const int64_t *deliv, const int32_t *qty,
                    const int64_t *amt, uint64_t n, int64_t cutoff, const Q1Scratch &s, int64_t d_lo,
                    int64_t d_hi, int64_t q_lo, int64_t q_hi, const Q6Scratch &s6, int num_sms,
                    cudaStream_t st);
void launch_q1_compact(const Q1Scratch &s, cudaStream_t st);        // tables -> groups[], ngroups
void launch_q1_emit(const Q1Scratch &s, uint64_t max_groups, cudaStream_t st);  // rank by key + AVG;
                                                                           // reads *ngroups on device

// ----------------------------------------------------- a7 peer transport (peer.cuh) --
// Cross-GPU merges move data with stores into the other ranks' "peer segments".
constexpr int kMaxRanks = 8;                               // one 8-GPU node
constexpr size_t kPeerCtlBytes = 64u << 10;
constexpr size_t kPeerSlotBytes = (2u << 20) + (64u << 10); // >= 16 + Q1's max group list (2 MB)
// (high bits: they share Q18Plan::err with the join error bits kErr*)
enum : unsigned int { kPeerErrTimeout = 1u << 16, kPeerErrHeap = 1u << 17, kPeerErrNoCarry = 1u << 18,
                      kPeerErrOutCap = 1u << 19 };
struct PeerCtl {                     // at offset 0 of every segment
    unsigned long long flag[kMaxRanks];  // flag[k]: last collective rank k delivered here
    unsigned long long seq;              // last collective this rank issued (device counter)
    unsigned int err;                    // sticky transport error bits
    unsigned int ticket;                 // last-block counter of multi-block producers
};
struct PeerArgs {                    // passed by value to every merge kernel
    char *seg[kMaxRanks];            // rank k's segment as mapped here (seg[rank] = own)
    int rank, world;
    unsigned long long slot_bytes, heap_half, timeout_ns;
    unsigned int *err_host;          // mapped pinned host word: error bits visible to the host
    // 1: another rank runs on this device in this process (N logical ranks on one GPU). A kernel
    // that waits for peers then lets its successor launch (PDL) only after the wait: a successor
    // resident early holds a share of every SM, which another rank's producer (one 224 KB block
    // per SM) may need — the producer this rank is waiting for. 0: the successor
    // launches early, as everywhere else on the hot path.
    int shared_device;
};
// Sum-allreduce of n <= 8 int64 values: dst (device, may equal src) and host_dst (mapped, or null)
void launch_peer_allreduce_i64(const PeerArgs &p, const long long *src, int n, long long *dst,
                               long long *host_dst, cudaStream_t st);
// Producer: copy `count` elements of `elem_bytes` (count read from *count_dev when non-null, else
// count_const) into mailbox[s & 1][rank] of every rank, slot header = the count (u64), data at +16.
void launch_peer_push(const PeerArgs &p, const void *src, const unsigned long long *count_dev,
                      unsigned long long count_const, unsigned int elem_bytes, int num_sms, cudaStream_t st);
// Consumer-only kernel (one thread): wait for every rank's latest collective; the multi-block
// consumers that read the mailboxes / heap run after it in stream order
void launch_peer_wait(const PeerArgs &p, cudaStream_t st);
// Q1: fold every rank's compacted group list (mailbox) into the clean global table. Like every
// multi-block consumer it does not wait itself: launch_peer_wait (one thread) runs before it, so
// waiting never occupies more than one block (N logical ranks on one device: a waiting grid
// could hold the SMs another rank's producer needs)
void launch_q1_peer_merge(const PeerArgs &p, const Q1Scratch &s, int num_sms, cudaStream_t st);

// ------------------------------------------------------------ Q18 (K3-K5) --
struct HtSlot { unsigned long long key; unsigned int row; unsigned int pad; };  // 16 B
constexpr unsigned long long kEmpty = ~0ull;
constexpr unsigned int kNoRow = 0xffffffffu;
struct Q18Acc { long long sum; unsigned int cnt; unsigned int pad; };          // 16 B
enum : unsigned int { kErrDupOrders = 1u, kErrDupCustomer = 2u, kErrDomain = 4u, kErrDupItem = 8u };

// Join index on a (w, d, id) primary key -> row. Two layouts, chosen per query by the planner
// from the snapshot's column statistics:
//  - dense: a perfect hash — slot = rank of (w, d, id) in the [min, max] box of the build side;
//    used when that box holds <= 4 slots per row (TPC-C keys are dense);
//  - hash: open addressing, 16-byte slots {packed key, row}, linear probing, cap = pow2 >= 2n.
struct JoinIndex {
    int dense;
    HtSlot *ht; unsigned long long mask;             // hash
    unsigned int *slots;                              // dense: [range] row or kNoRow
    int w0, d0, k0;                                   // dense: box minimum
    unsigned int nw, nd, nk;                          // dense: box extents
    unsigned long long range;                         // dense: nw * nd * nk
    // dense and exactly one build row per box slot (n == range): the build side MAY be stored in
    // key order ("clustered"), i.e. row == slot for every row. The init kernel verifies that,
    // counting violations into *viol; while *viol == 0 lookups return the slot itself (no slot
    // read, no insert at build: DESIGN.md §4.3). A counter per index per query parity; the init of
    // query k clears the counters query k+1 uses.
    int may_ident;
    unsigned int *viol, *viol_next;
};
struct Q18Stats {            // min/max of the sort fields that only the result rows know
    long long amt_min, amt_max, ent_min, ent_max;
};
struct Q18Zone {             // bounds of the other result-row fields: the snapshot's zone maps
    int w_min, w_max, d_min, d_max, o_min, o_max;      // orders (w, d, o) key columns
    int cl_min, cl_max, ci_min, ci_max, n_min, n_max;  // c_last, c_id, o_ol_cnt (carry payload)
    long long e_min, e_max;  // o_entry_d over every orders row (64-bit zone map), valid if has_e
    int has_e;
};
struct __align__(16) Q18Row {  // one result row before ORDER BY: 32 B = one L2 sector per gather
    long long o_entry_d;       // (amount_sum lives in a parallel array: after the sort it is
    int c_last, c_id, o_id, o_ol_cnt, o_w_id, o_d_id;  //  recovered from the sorted key)
};
static_assert(sizeof(Q18Row) == 32, "Q18Row must be one sector");
struct Q18Cols {             // SoA result columns
    int32_t *c_last, *c_id, *o_id, *o_ol_cnt, *o_w_id, *o_d_id;
    int64_t *o_entry_d, *amount_sum;
};
struct Q18Scratch {
    JoinIndex jo, jc;
    Q18Acc *acc;             // [n_orders]
    unsigned int *err;       // [1]
    unsigned long long *nout;// [1]
    Q18Stats *stats;         // [1] final
    Q18Stats *stat_part;     // [grid] per-block partials
    unsigned int *ticket;    // [1] last-block counter, zero-initialised once, self-resetting
    Q18Row *rows;            // [n_orders] unsorted result rows
    long long *amt;          // [n_orders] their amount_sum
    // CH Q3 only (else null): orders rows marked by the new_order ⋈ customer step, and their count
    unsigned int *cand;      // [n_new_order]
    unsigned long long *ncand;// [1]
    unsigned int *qbits;     // [qwords] bitmap of the marked orders rows (cleared by init)
    unsigned long long qwords;
    unsigned int *tie;       // ORDER BY flag word, zeroed by init (null: not zeroed)
};
// empties both join indexes (and verifies a clustered build side: JoinIndex::may_ident)
void launch_q18_init(const Q18Scratch &s, const int32_t *o_w, const int32_t *o_d, const int32_t *o_id,
                     uint64_t n_o, const int32_t *c_w, const int32_t *c_d, const int32_t *c_id, uint64_t n_c,
                     int num_sms, cudaStream_t st);
void launch_q18_build(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, uint64_t n_o,
                      const int32_t *c_w, const int32_t *c_d, const int32_t *c_id, uint64_t n_c,
                      const Q18Scratch &s, int num_sms, cudaStream_t st);
void launch_q18_probe(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o,
                      const int64_t *ol_amt, uint64_t n_ol, const Q18Scratch &s, int num_sms,
                      cudaStream_t st);
void launch_q18_probe_tma(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o,
                          const int64_t *ol_amt, uint64_t n_ol, const Q18Scratch &s, int num_sms,
                          cudaStream_t st);  // same result, TMA-bulk staged, one block per SM
// the batch's full pass: Q6 + Q1 (as launch_q61_tma) and Q18's probe + group-join (K4) over one
// TMA-staged read of order_line's 7 columns; the orders join index must be built
void launch_q6118_tma(const int32_t *number, const int64_t *deliv, const int32_t *qty, const int64_t *amt,
                      const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o, uint64_t n, int64_t cutoff,
                      const Q1Scratch &s, int64_t d_lo, int64_t d_hi, int64_t q_lo, int64_t q_hi,
                      const Q6Scratch &s6, const Q18Scratch &s18, int num_sms, cudaStream_t st);
void launch_q18_having(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id,
                       const int32_t *o_c, const int32_t *o_cnt, const int64_t *o_ent,
                       uint64_t n_o, const int32_t *c_last, int64_t having,
                       const Q18Scratch &s, int num_sms, cudaStream_t st, int unroll = 2);
// CH Q3 (NEXT-2) on the Q18 machinery: mark orders rows joined by new_order and an 'prefix%'
// customer (multiplicity in acc[].pad, candidate list in cand / *ncand), probe order_line into the
// marked rows only, emit result rows (revenue = sum x multiplicity, count *nout) + sort statistics.
// no_del: the new_order tombstone column (null: no row deleted); deleted rows join nothing
void launch_q3_mark(const int32_t *no_w, const int32_t *no_d, const int32_t *no_o, const int32_t *no_del, uint64_t n_no,
                    const int32_t *o_w, const int32_t *o_d, const int32_t *o_c, const int64_t *o_ent,
                    const int32_t *c_p2, int64_t entry_lo, int prefix, const Q18Scratch &s, int num_sms,
                    cudaStream_t st);
void launch_q3_probe(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o,
                     const int64_t *ol_amt, uint64_t n_ol, const Q18Scratch &s, int num_sms,
                     cudaStream_t st);
void launch_q3_emit(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, const int32_t *o_c,
                    const int32_t *o_cnt, const int64_t *o_ent, uint64_t max_cand, const Q18Scratch &s,
                    int num_sms, cudaStream_t st);
// {nout, err, tie} -> mapped pinned host memory (one launch instead of three D2H copies)
void launch_q18_publish(const unsigned long long *nout, const unsigned int *err, const unsigned int *tie,
                        void *host_small, const JoinIndex &jo, const JoinIndex &jc, cudaStream_t st);

// ------------------------------------------------------------------ sort ---
// Stable LSD radix sort of (u64 key, u32 value) pairs, 8-bit digits, `bits` low key bits.
// Keys travel with values, so every pass reads and writes contiguously.
constexpr int kSortThreads = 256;
constexpr int kSortItems = 16;                              // per lane
constexpr int kSortTile = kSortThreads * kSortItems;        // 4096 elements per block tile
inline uint64_t sort_tiles(uint64_t n) { return (n + kSortTile - 1) / kSortTile; }
struct SortPairs {
    unsigned long long *k[2];
    unsigned int *v[2];
    unsigned int *counts;        // [256 * tiles]
    unsigned int *totals;        // [256]
};
// Returns which buffer (0/1) holds the sorted pairs (input is in k[0]/v[0]).
int radix_sort_pairs(uint64_t n, int bits, const SortPairs &s, int num_sms, cudaStream_t st);

// Scratch of the ORDER BY bucket sort: keys + row ids ping-pong, bucket counts,
// offsets/cursors, a work list of buckets above the small in-shared-memory capacity, and the
// last-block ticket of the keys+histogram kernel.
constexpr int kBucketMaxBits = 15;
struct BucketSort {
    unsigned long long *k[2];
    unsigned int *v[2];
    unsigned int *count;   // [2^kBucketMaxBits + 1]
    unsigned int *cursor;  // [2^kBucketMaxBits]
    unsigned int *offset;  // [2^kBucketMaxBits + 1]
    unsigned int *big;     // [1 + 2^kBucketMaxBits]: count, then ids of buckets > small capacity
    unsigned int *ticket;  // [1], zero-initialised once, self-resetting
    unsigned int *mat;     // v2: [ob_grid * 2^bucket_bits] per-partition bucket counts -> offsets
    unsigned long long *kv;// v2: [2 n] interleaved (key, row id) pairs in bucket order
};
// Optional per-kernel profiling marks (the engine records CUDA events around each phase).
struct PhaseMarks {
    virtual void begin(const char *name) = 0;
    virtual void end() = 0;
    virtual ~PhaseMarks() = default;
};

// Q18 ORDER BY amount_sum DESC, o_entry_d, o_w_id, o_d_id, o_id (R11).
struct Q18SortSpec {         // host-computed from Q18Stats
    long long amt_max, ent_min;
    int w_min, d_min, o_min;
    int bits_w, bits_d, bits_o;  // r = (w - w_min | d - d_min | o - o_min), fields concatenated
    int wide_r;              // bits_w + bits_d + bits_o > 62: exact per-column fallback
    int bits_a, bits_e, bits_r;  // field widths: amount (desc), entry, (w, d, o) tie-break
    int prefix_bits;         // width of the sorted 64-bit prefix of the composite key
    // carry mode: the 128-bit sort record (prefix, low key bits | payload)
    // holds the whole result row, so the emit decodes instead of gathering rows.
    int carry;               // 1 if bits_a + bits_e + bits_r + payload bits <= 128
    int bits_low;            // key bits below the 64-bit prefix (carried in the second word)
    int bits_cl, bits_ci, bits_n;  // payload widths: c_last, c_id, o_ol_cnt (offsets from min)
    int cl_min, ci_min, n_min;
};
// Device-side plan of the ORDER BY, computed from the HAVING kernel's statistics and row count
// (no host round trip): field widths, 64-bit prefix width, whether a tie-fix is needed, and the
// bucket shift for `bucket_bits` buckets.
struct Q18Plan {
    unsigned long long n;        // rows this rank sorts (world > 1: its rows BEFORE the exchange)
    Q18SortSpec spec;
    int tiefix;
    int shift;
    int bucket_bits;             // buckets = 1 << bucket_bits (world > 1: from the global row count)
    // distributed ORDER BY (world > 1): the buckets are range-partitioned over
    // the ranks by their global row positions; rank k holds rows [row0, row0 + n_mine) of the
    // globally ordered result
    int dist;
    unsigned int b_lo, nb_mine;  // this rank's buckets [b_lo, b_lo + nb_mine)
    unsigned long long n_total, n_mine, row0;
    unsigned long long xseq;     // sequence number of the record exchange (heap parity = xseq & 1)
    unsigned long long nbuckets; // dist: 1 << bucket_bits (the length of the pushed count list)
    unsigned int err;            // OR of every rank's join error bits (+ kErrPeer*)
};
void launch_q18_plan(const Q18Stats *stats, const Q18Zone &zone, const unsigned long long *nout,
                     int bucket_bits, bool allow_carry, Q18Plan *plan, unsigned int *flag,
                     cudaStream_t st);
// The whole ORDER BY: keys + histogram -> bucket scatter -> per-bucket sort, tie-fix and emit
// into `dst` (final positions). Everything reads the row count and widths from *plan.
// *flag: bit0 a tie run > 32 rows, bit1 a bucket > 8192 rows (caller redoes it exactly).
void q18_bucket_order(const Q18Row *rows, const long long *amt, const Q18Plan *plan, uint64_t n_max,
                      int bucket_bits, const BucketSort &s, const Q18Cols &dst, unsigned int *flag,
                      int num_sms, cudaStream_t st, PhaseMarks *marks = nullptr);
// Same contract, v2 (default): no global atomics in the partition (count matrix +
// column scan), keys computed in the scatter; the per-bucket sort + emit kernels are v1's.
int ob_grid(int num_sms);
int ob_bucket_bits(uint64_t n_max);
// The inputs of the ORDER BY plan when the v2 histogram kernel computes it (no plan launch).
struct Q18PlanArgs {
    const Q18Stats *stats;
    Q18Zone zone;
    const unsigned long long *nout;
    int allow_carry;
};
void q18_bucket_order_v2(const Q18Row *rows, const long long *amt, Q18Plan *plan, uint64_t n_max,
                         int bucket_bits, const BucketSort &s, const Q18Cols &dst, unsigned int *flag,
                         int num_sms, cudaStream_t st, PhaseMarks *marks = nullptr,
                         const Q18PlanArgs *plan_args = nullptr);  // non-null: hist writes *plan
// Distributed ORDER BY (world > 1): plan from every rank's statistics, local
// partition, exchange of the carry records into the owners' heaps, per-bucket sort + emit of this
// rank's range of the global order into dst (capacity out_cap rows); {n_mine, err, tie, stats,
// row0, n_total} -> host_small (mapped). send: [2^kBucketMaxBits] u64, recv_off: [2^kBucketMaxBits+1].
// v3: the HAVING pass builds the carry records itself, with a plan derived
// beforehand from the accumulators (launch_q18_acc_stats). The arguments of that HAVING pass:
struct Q18HavingArgs {
    const int32_t *o_w, *o_d, *o_id, *o_c, *o_cnt;
    const int64_t *o_ent;
    uint64_t n_o;
    const int32_t *c_last;
    int64_t having;
    Q18Scratch s;
    unsigned int *cnt_part;   // [ob_grid] records per partition
};
// min / max of amount_sum and o_entry_d over the groups passing cnt > 0 AND sum > having (and their
// count, *count); with plan_args, the last block also derives the ORDER BY plan (zone from there)
void launch_q18_acc_stats(const Q18Scratch &s, const int64_t *o_ent, uint64_t n_o, int64_t having,
                          unsigned long long *cpart, unsigned long long *count, const Q18PlanArgs *plan_args,
                          int bucket_bits, Q18Plan *plan, unsigned int *flag, int num_sms, cudaStream_t st);
// one GPU: HAVING + records + histogram -> scan -> scatter -> per-bucket sort + emit; *flag bit 8:
// the records did not fit (the host re-runs the v2 path), bit 1: an oversized bucket (likewise)
void q18_order_v3(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, const int32_t *o_c,
                  const int32_t *o_cnt, const int64_t *o_ent, uint64_t n_o, const int32_t *c_last,
                  int64_t having, const Q18Scratch &s, const Q18Plan *plan, int bucket_bits,
                  const BucketSort &bs, unsigned int *cnt_part, const Q18Cols &dst, unsigned int *flag,
                  int num_sms, cudaStream_t st, PhaseMarks *marks = nullptr, bool counted = false);
// one GPU, direct ORDER BY: the plan (acc_stats) and the bucket counts in one kernel with a grid
// barrier — only when its grid is resident at once (q18_plan_hist_ok) and no other engine shares
// the device
bool q18_plan_hist_ok(int num_sms, int bucket_bits);
void launch_q18_plan_hist(const Q18Scratch &s, uint64_t n_o, int64_t having, unsigned long long *cpart,
                          unsigned long long *gbar, unsigned long long *count, const Q18Zone &zone,
                          int bucket_bits, Q18Plan *plan, unsigned int *flag, const BucketSort &bs, int num_sms,
                          cudaStream_t st);
// hv non-null: the v3 input (records built by the HAVING pass); null: rows + amounts (Q3)
void q18_bucket_order_dist(const PeerArgs &pa, const Q18Row *rows, const long long *amt, Q18Plan *plan,
                           const Q18PlanArgs &meta, const unsigned int *err, const BucketSort &s,
                           unsigned long long *send, unsigned int *recv_off, uint64_t out_cap,
                           const Q18Cols &dst, unsigned int *flag, void *host_small, int num_sms,
                           cudaStream_t st, PhaseMarks *marks = nullptr, const Q18HavingArgs *hv = nullptr);
// The emit phase alone (re-run by the host into larger output columns after kPeerErrOutCap; the
// exchanged records stay in the heap until the next exchange of the same parity).
void q18_dist_emit(const PeerArgs &pa, const Q18Plan *plan, const unsigned int *recv_off, const Q18Cols &dst,
                   unsigned int *flag, const BucketSort &s, int num_sms, cudaStream_t st, PhaseMarks *marks = nullptr);
// Within runs of equal prefix, order by the full tuple; runs longer than 32 raise *flag.
// Exact fallback: three stable passes over the full fields (row rank, entry, amount).
void launch_q18_field_keys(const Q18Row *rows, const long long *amt, const unsigned int *vals,
                           uint64_t n, int field, const Q18Plan *plan, unsigned long long *keys,
                           int num_sms, cudaStream_t st);
void launch_iota(unsigned int *v, uint64_t n, int num_sms, cudaStream_t st);
// Gather rows in `perm` order into SoA columns. amount_sum: decoded from the sorted prefix keys
// when `keys` is given (field a is always whole at the top of the prefix), else read from amt.
// `perm`/`keys` null: identity order (n <= 1) or amounts read from amt (field-key fallback).
void launch_q18_permute(const Q18Row *rows, const long long *amt, const unsigned int *perm,
                        const unsigned long long *keys, const Q18Plan *plan, uint64_t n_max,
                        const Q18Cols &dst, int num_sms, cudaStream_t st);

// ------------------------------------------------------------ store (a1) --
void launch_stats_init(int *out, int n_pairs, cudaStream_t st);
void launch_gate(unsigned long long ns, cudaStream_t st);  // profiling only  // pairs of (INT_MAX, INT_MIN)
void launch_minmax_i32(const int32_t *p, uint64_t n, int *out, int num_sms, cudaStream_t st);
// 64-bit zone map: out[2k] = INT64_MAX, out[2k + 1] = INT64_MIN; then min / max of p[0, n) merged in
void launch_stats_init64(long long *out, int n_pairs, cudaStream_t st);
void launch_minmax_i64(const int64_t *p, uint64_t n, long long *out, int num_sms, cudaStream_t st);
// copy-on-write of updated columns (NEXT-1): page = kCowPageRows rows, one dirty bit per page
constexpr uint64_t kCowPageRows = 4096;
static_assert(kCowPageRows * 4 == 4 * 16 * 256, "catch-up kernel: one page = 4/8 uint4 per thread");
// copy dirty pages (bits) and rows [synced_rows, n_rows) cur -> alt; clear next_bits[0, nwords)
void launch_cow_catchup(void *dst, const void *src, uint32_t es, const uint32_t *bits,
                        uint32_t *next_bits, uint64_t nwords, uint64_t synced_rows, uint64_t n_rows,
                        unsigned long long *pages_copied, int num_sms, cudaStream_t st);
void launch_apply_updates(void *col, uint32_t es, uint32_t *bits, const uint32_t *rows,
                          const void *vals, uint64_t n, int num_sms, cudaStream_t st);

// ---------------------------------------------------------------- helpers --
// Per file: load every kernel and set the dynamic shared-memory limits, for the current device, at
// h2tap_open (per device, return codes checked; no per-process static flags).
cudaError_t set_attributes_scan(int num_sms);
cudaError_t set_attributes_join(int num_sms);
cudaError_t set_attributes_sort(int num_sms);
cudaError_t set_attributes_ch(int num_sms);
cudaError_t set_attributes_layout(int num_sms);
cudaError_t set_attributes_store(int num_sms);
cudaError_t set_attributes_peer(int num_sms);
// Every launcher counts the kernels it launches (reported per query as kernel_launches).
void count_launches(int n);

// Programmatic dependent launch: the hot-path kernels of a batch are launched
// with programmatic stream serialization, so kernel k+1 is already resident when kernel k ends
// (launch latency and its block scheduling overlap k's tail). Every such kernel starts with
// pdl_wait() — it returns once the preceding grid has completed and its writes are visible — and
// pdl_trigger(), which lets the next grid launch. H2TAP_PDL=0 launches them normally (A/B).
// Device-side invariant checks, compiled in only for the checking build (-DH2TAP_CHECKS=1,
// scripts/build_variants.py): a violated index bound traps the kernel (the test then fails with
// a CUDA error) — the bounds checks that stand in for compute-sanitizer where it is unavailable.
#if defined(H2TAP_CHECKS) && H2TAP_CHECKS
#define H2TAP_CHECK(cond) do { if (!(cond)) __trap(); } while (0)
#else
#define H2TAP_CHECK(cond) do { } while (0)
#endif
__device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }
__device__ __forceinline__ void pdl_trigger() { asm volatile("griddepcontrol.launch_dependents;" ::: "memory"); }
bool pdl_enabled();
template <typename... KArgs, typename... Args>
inline void launch_pdl(void (*kern)(KArgs...), dim3 grid, dim3 block, size_t smem, cudaStream_t st,
                       Args &&...args) {
    cudaLaunchAttribute at[1];
    at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
    at[0].val.programmaticStreamSerializationAllowed = pdl_enabled() ? 1 : 0;
    cudaLaunchConfig_t cfg = {};
    cfg.gridDim = grid;
    cfg.blockDim = block;
    cfg.dynamicSmemBytes = smem;
    cfg.stream = st;
    cfg.attrs = at;
    cfg.numAttrs = 1;
    cudaLaunchKernelEx(&cfg, kern, std::forward<Args>(args)...);
}

// ------------------------------------------- NEXT-2: CH Q14 / Q12 / Q4 (ch_kernels.cu) --
// GROUP BY o_ol_cnt with counters (a, b, rows) per group: keys in [0, kSgDense) in thread-private
// shared memory, others in a global open-addressing table of kSgSlots groups.
constexpr int kSgDense = 16;
constexpr int kSgSlots = 2048;
struct SmallGroups {
    unsigned long long *dense;     // [3 * kSgDense]: a, b, rows of key k at 3k..3k+2
    unsigned long long *gtag;      // [kSgSlots]: 0 = empty, else (1 << 32 | (u32)key)
    unsigned long long *gacc;      // [3 * kSgSlots]
    unsigned int *flags;           // [1]: bit0 = table full
    int32_t *o_key; long long *o_a, *o_b; unsigned long long *ngroups;  // output ranked by key
};
void launch_sg_reset(const SmallGroups &g, cudaStream_t st);  // once, at allocation
void launch_sg_emit(const SmallGroups &g, cudaStream_t st);   // rank + write; re-clears the tables
// multi-GPU: wait for every rank's pushed table (dense | gtag | gacc contiguous, launch_peer_push)
// and fold the other ranks' tables into g
void launch_sg_peer_merge(const PeerArgs &p, const SmallGroups &g, cudaStream_t st);
// orders (w, d, o_id) join index alone: clear + insert (and zero mark[] for Q4 when non-null)
void launch_jx_build_orders(const int32_t *o_w, const int32_t *o_d, const int32_t *o_id, uint64_t n_o,
                            const JoinIndex &jo, unsigned int *err, uint8_t *mark, int num_sms,
                            cudaStream_t st);
void launch_q12_probe(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o, const int64_t *ol_dl,
                      uint64_t n_ol, const JoinIndex &jo, const int64_t *o_entry, const int32_t *o_carrier,
                      const int32_t *o_cnt, int64_t d_hi, const SmallGroups &g, int num_sms, cudaStream_t st);
void launch_q4(const int32_t *ol_w, const int32_t *ol_d, const int32_t *ol_o, const int64_t *ol_dl,
               uint64_t n_ol, const JoinIndex &jo, const int64_t *o_entry, const int32_t *o_cnt,
               uint64_t n_o, int64_t e_lo, int64_t e_hi, uint8_t *mark, const SmallGroups &g,
               int num_sms, cudaStream_t st, PhaseMarks *marks);
// Q14: item map, 2 bits per i_id in [i0, i0 + range): bit0 exists, bit1 i_data prefix matches
struct ItemMap { unsigned int *bits; long long i0; unsigned long long range, words; };
void launch_item_map(const int32_t *i_id, const int32_t *p2, uint64_t n, int32_t prefix2, const ItemMap &m,
                     unsigned int *err, int num_sms, cudaStream_t st);
struct Q14Scratch {
    long long *block_part;         // [3 * q14_max_blocks]
    unsigned int *done_counter;    // [1], zero-initialised once, self-resetting
    long long *out;                // [3]: sum_promo, sum_amount, count
    double *promo;                 // [1]
};
int q14_max_blocks(int num_sms);
void launch_q14(const int64_t *deliv, const int32_t *i_id, const int64_t *amt, uint64_t n, int64_t d_lo,
                int64_t d_hi, const ItemMap &m, const Q14Scratch &s, int num_sms, cudaStream_t st);
void launch_q14_finalize(const Q14Scratch &s, cudaStream_t st);
uint64_t launches_total();

// ------------------------------ NEXT-3 / NEXT-4: layout scans (layout_kernels.cu) --
// SUM(col_1 + ... + col_N) over int32 attributes in DSM / PAX / NSM (§5.3); `data` is a
// device pointer or a mapped pinned host pointer (zero-copy over PCIe). *out accumulates (zero it).
enum { kLayoutDsm = 1, kLayoutPax = 2, kLayoutNsm = 3 };
constexpr int kMaxLayoutSel = 64;
struct LayoutSel { int n; int col[kMaxLayoutSel]; };  // selected attribute indices
void launch_layout_sum(const int32_t *data, int layout, uint64_t n, int log_ncols, int log_mp,
                       uint64_t dsm_stride, unsigned long long mask, const LayoutSel &sel,
                       unsigned long long *out, int num_sms, cudaStream_t st);

}  // namespace h2tap
