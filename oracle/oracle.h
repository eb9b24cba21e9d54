/*
 * oracle.h — CPU ORACLE for the CH-benCHmark OLAP hot path. TEST INFRASTRUCTURE ONLY.
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference
 * legs may load liboracle.so. It shares no code, header, table or constant with the
 * CUDA path (paper_conf_cidr_appuswamykpa17_b200/, include/), and never includes them.
 *
 * What it computes: the plain SQL definitions of CH-benCHmark Q1, Q6 and Q18, and (NEXT-2)
 * Q14, Q12, Q4 and Q3, and (NEXT-3) the paper's own layout query SUM(col1 + ... + colN)
 * (SURVEY.md Appendix A.1 [EXT]; the paper's OLAP path is PAPER.md L524-572, its only
 * query text is "TPC-H Q6, a selection over the lineitem table", L687-688), evaluated
 * row at a time, single-threaded, with SQL three-valued logic for NULLs.
 *
 * Encodings (R4-R6): timestamps int64 µs UTC, NULL = INT64_MIN (decoded here,
 * independently of the GPU path); money int64 cents; ids/quantities int32.
 *
 * Parity pins: tests/test_oracle_*.py — SQLite running the literal CH SQL, brute-force
 * nested loops on tiny tables, strict-mode closed forms, hand-derived golden fixture
 * (tests/golden/), re-partition and COUNT invariants. No function here is "parity unpinned".
 */
#ifndef H2TAP_ORACLE_H
#define H2TAP_ORACLE_H
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

/* Borrowed, caller-owned column pointers (SoA). */
typedef struct {
    int64_t n;
    const int32_t *w_id, *d_id, *o_id, *number;
    const int64_t *delivery_d;      /* INT64_MIN = NULL */
    const int32_t *quantity;
    const int64_t *amount;          /* cents */
    const int32_t *i_id;            /* ol_i_id (Q14 only; may be NULL otherwise) */
} or_order_line;

typedef struct {
    int64_t n;
    const int32_t *w_id, *d_id, *o_id, *c_id, *ol_cnt;
    const int64_t *entry_d;
    const int32_t *carrier_id;      /* -1 = NULL (Q12 only; may be NULL otherwise) */
} or_orders;

typedef struct {
    int64_t n;
    const int32_t *i_id;
    const char *i_data;             /* n strings of `width` bytes each, NUL-padded */
    int64_t width;
} or_item;

typedef struct {
    int64_t n;
    const int32_t *w_id, *d_id, *c_id, *c_last;
    const char *state;              /* c_state: n strings of `state_width` bytes (Q3 only) */
    int64_t state_width;
} or_customer;

typedef struct {
    int64_t n;
    const int32_t *w_id, *d_id, *o_id;  /* no_w_id, no_d_id, no_o_id */
} or_new_order;

/* Status codes. */
#define OR_OK        0
#define OR_OVERFLOW -1   /* an int64 SUM overflowed (SQLite raises "integer overflow") */
#define OR_NOMEM    -2

/* 3-valued comparison of a (possibly NULL = INT64_MIN) timestamp v with constant c, as the
 * queries below evaluate it; op 0 '>=', 1 '<', 2 '>'. Returns 0 FALSE, 1 TRUE, 2 UNKNOWN. */
int oracle_ts_cmp(int op, int64_t v, int64_t c);

/* CH Q6: SELECT SUM(ol_amount) FROM order_line WHERE ol_delivery_d >= d_lo AND
 * ol_delivery_d < d_hi AND ol_quantity BETWEEN q_lo AND q_hi.
 * *revenue_is_null = 1 when no row qualifies (SUM over the empty set is NULL).
 * *count = number of qualifying rows (not part of the SQL output; used by invariants). */
int oracle_q6(const or_order_line *ol, int64_t d_lo, int64_t d_hi, int64_t q_lo, int64_t q_hi,
              int64_t *revenue, int32_t *revenue_is_null, int64_t *count);

/* CH Q1: SELECT ol_number, SUM(ol_quantity), SUM(ol_amount), AVG(ol_quantity),
 * AVG(ol_amount), COUNT(*) FROM order_line WHERE ol_delivery_d > cutoff
 * GROUP BY ol_number ORDER BY ol_number.
 * avg_amount is in currency units: (sum_cents / count) / 100.
 * Writes min(ngroups, cap) rows; returns ngroups (>= 0) or a negative status. */
int64_t oracle_q1(const or_order_line *ol, int64_t cutoff, int64_t cap,
                  int32_t *ol_number, int64_t *sum_qty, int64_t *sum_amount,
                  double *avg_qty, double *avg_amount, int64_t *count_order);

/* CH Q18 (customer ⋈ orders ⋈ order_line, GROUP BY, HAVING SUM(ol_amount) > having):
 * output columns c_last, c_id, o_id, o_entry_d, o_ol_cnt, amount_sum, plus o_w_id, o_d_id
 * (R3), ordered by amount_sum DESC, o_entry_d ASC, then o_w_id, o_d_id, o_id,
 * c_id, c_last, o_ol_cnt ASC (R11). Writes min(nrows, cap) rows; returns nrows or < 0. */
int64_t oracle_q18(const or_customer *c, const or_orders *o, const or_order_line *ol,
                   int64_t having, int64_t cap,
                   int32_t *c_last, int32_t *c_id, int32_t *o_id, int64_t *o_entry_d,
                   int32_t *o_ol_cnt, int64_t *amount_sum, int32_t *o_w_id, int32_t *o_d_id);

/* CH Q14: SELECT 100.00 * SUM(CASE WHEN i_data LIKE prefix || '%' THEN ol_amount ELSE 0 END)
 *                / (1 + SUM(ol_amount)) AS promo_revenue
 * FROM order_line, item WHERE ol_i_id = i_id AND ol_delivery_d >= d_lo AND ol_delivery_d < d_hi.
 * Money in cents: promo_revenue = (100.0 * (double)sum_promo) / (100.0 + (double)sum_amount)
 * (R30); NULL (*is_null = 1) when no joined row qualifies. LIKE is case-sensitive. */
int oracle_q14(const or_order_line *ol, const or_item *it, int64_t d_lo, int64_t d_hi,
               const char *prefix, double *promo_revenue, int32_t *is_null, int64_t *sum_promo,
               int64_t *sum_amount, int64_t *count);

/* CH Q12: SELECT o_ol_cnt,
 *   SUM(CASE WHEN o_carrier_id = 1 OR o_carrier_id = 2 THEN 1 ELSE 0 END) AS high_line_count,
 *   SUM(CASE WHEN o_carrier_id <> 1 AND o_carrier_id <> 2 THEN 1 ELSE 0 END) AS low_line_count
 * FROM orders, order_line WHERE ol_w_id = o_w_id AND ol_d_id = o_d_id AND ol_o_id = o_id
 *   AND o_entry_d <= ol_delivery_d AND ol_delivery_d < d_hi GROUP BY o_ol_cnt ORDER BY o_ol_cnt.
 * Writes min(ngroups, cap) rows; returns ngroups or < 0. */
int64_t oracle_q12(const or_orders *o, const or_order_line *ol, int64_t d_hi, int64_t cap,
                   int32_t *o_ol_cnt, int64_t *high_line_count, int64_t *low_line_count);

/* CH Q4: SELECT o_ol_cnt, COUNT(*) AS order_count FROM orders
 * WHERE o_entry_d >= e_lo AND o_entry_d < e_hi AND EXISTS (SELECT * FROM order_line
 *   WHERE o_id = ol_o_id AND o_w_id = ol_w_id AND o_d_id = ol_d_id AND ol_delivery_d >= o_entry_d)
 * GROUP BY o_ol_cnt ORDER BY o_ol_cnt. Writes min(ngroups, cap) rows; returns ngroups or < 0. */
int64_t oracle_q4(const or_orders *o, const or_order_line *ol, int64_t e_lo, int64_t e_hi,
                  int64_t cap, int32_t *o_ol_cnt, int64_t *order_count);

/* CH Q3: SELECT ol_o_id, ol_w_id, ol_d_id, SUM(ol_amount) AS revenue, o_entry_d
 * FROM customer, new_order, orders, order_line
 * WHERE c_state LIKE prefix || '%' AND c_id = o_c_id AND c_w_id = o_w_id AND c_d_id = o_d_id
 *   AND no_w_id = o_w_id AND no_d_id = o_d_id AND no_o_id = o_id
 *   AND ol_w_id = o_w_id AND ol_d_id = o_d_id AND ol_o_id = o_id AND o_entry_d > entry_lo
 * GROUP BY ol_o_id, ol_w_id, ol_d_id, o_entry_d ORDER BY revenue DESC, o_entry_d
 * (ties: ol_w_id, ol_d_id, ol_o_id ASC, R33). Output columns ol_o_id, ol_w_id,
 * ol_d_id, revenue, o_entry_d. Writes min(nrows, cap) rows; returns nrows or < 0. */
int64_t oracle_q3(const or_customer *c, const or_new_order *no, const or_orders *o,
                  const or_order_line *ol, int64_t entry_lo, const char *prefix, int64_t cap,
                  int32_t *ol_o_id, int32_t *ol_w_id, int32_t *ol_d_id, int64_t *revenue,
                  int64_t *o_entry_d);

/* NEXT-3 (§5.3): SELECT SUM(col_c1 + ... + col_cN) FROM dataset, for the
 * attributes c with bit c of col_mask set, over a table of nrows records of ncols int32 attributes
 * stored in one of the paper's three layouts (L968-972), value of record r, attribute c at:
 *   layout 1 DSM (each attribute stored contiguously):  data[c * col_stride + r]
 *   layout 2 PAX (pages of ncols minipages of pax_rows values; the paper: 16 x 64):
 *            data[(r / pax_rows) * ncols * pax_rows + c * pax_rows + r % pax_rows]
 *   layout 3 NSM (each record stored contiguously):      data[r * ncols + c]
 * Per record the selected values are added in int64, then summed over records (overflow-checked).
 * *is_null = 1 iff nrows == 0. Returns OR_OK or OR_OVERFLOW. */
int oracle_layout_sum(const int32_t *data, int layout, int64_t nrows, int64_t ncols, int64_t col_stride,
                      int64_t pax_rows, uint64_t col_mask, int64_t *sum, int32_t *is_null);

#ifdef __cplusplus
}
#endif
#endif
