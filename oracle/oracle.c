/*
 * oracle.c — CPU ORACLE (test infrastructure only; see oracle.h for who may use it).
 *
 * Plain, slow, single-threaded, row-at-a-time evaluation of the CH-benCHmark queries
 * on the hot path, written from their SQL definitions (SURVEY.md Appendix A.1 [EXT]).
 * The paper's OLAP runtime executes such queries over a snapshot of the tables
 * ("Caldera always executes OLAP queries on a database snapshot");
 * a query result is a function of the rows visible in that snapshot only, which is
 * why each function below takes exactly the visible rows.
 *
 * Structure (a tiny Volcano pipeline written out, no fusion beyond the SQL):
 *   scan -> WHERE (3-valued logic) -> [hash join] -> hash GROUP BY -> HAVING -> ORDER BY.
 * The hash table and qsort are library-style primitives; the grouping key is the full
 * GROUP BY tuple, not a shortcut through functional dependencies.
 */
#include "oracle.h"

#include <stdlib.h>
#include <string.h>

/* ---------------------------------------------------------------- SQL 3VL -- */
typedef enum { SQL_FALSE = 0, SQL_TRUE = 1, SQL_UNKNOWN = 2 } sqlbool;

/* The oracle's own decoding of the NULL sentinel (R5). */
static const int64_t OR_NULL_TS = INT64_MIN;

static sqlbool sql_and(sqlbool a, sqlbool b) {
    if (a == SQL_FALSE || b == SQL_FALSE) return SQL_FALSE;
    if (a == SQL_UNKNOWN || b == SQL_UNKNOWN) return SQL_UNKNOWN;
    return SQL_TRUE;
}
/* ts <op> constant, where ts may be NULL: any comparison with NULL is UNKNOWN. */
static sqlbool ts_ge(int64_t v, int64_t c) { return v == OR_NULL_TS ? SQL_UNKNOWN : (v >= c ? SQL_TRUE : SQL_FALSE); }
static sqlbool ts_lt(int64_t v, int64_t c) { return v == OR_NULL_TS ? SQL_UNKNOWN : (v < c ? SQL_TRUE : SQL_FALSE); }
static sqlbool ts_gt(int64_t v, int64_t c) { return v == OR_NULL_TS ? SQL_UNKNOWN : (v > c ? SQL_TRUE : SQL_FALSE); }
/* x BETWEEN lo AND hi  ==  x >= lo AND x <= hi (inclusive, R12); x NOT NULL. */
static sqlbool between(int64_t x, int64_t lo, int64_t hi) {
    return sql_and(x >= lo ? SQL_TRUE : SQL_FALSE, x <= hi ? SQL_TRUE : SQL_FALSE);
}

/* Test hook (test infrastructure only): the timestamp comparisons above, exported so a test
 * can pin their three-valued results against SQLite's NULL semantics, including a constant
 * equal to the sentinel's own value (a NULL test dropped from one helper is otherwise masked
 * in Q6, where ts_ge is ANDed with ts_lt's UNKNOWN). op: 0 = '>=', 1 = '<', 2 = '>'.
 * Returns 0 FALSE, 1 TRUE, 2 UNKNOWN; -1 for an unknown op. */
int oracle_ts_cmp(int op, int64_t v, int64_t c) {
    switch (op) {
        case 0: return (int)ts_ge(v, c);
        case 1: return (int)ts_lt(v, c);
        case 2: return (int)ts_gt(v, c);
        default: return -1;
    }
}

/* ------------------------------------------------------- generic hash map -- */
/* Keys are tuples of k int64 values; each entry carries an int64 payload.
 * Used both as a multimap (join index: every row inserted) and as a map
 * (GROUP BY: find-or-insert). */
typedef struct {
    int k;
    int64_t nbuckets, n, cap;
    int64_t *heads, *keys, *next, *val;
} ormap;

static uint64_t mix64(uint64_t x) {
    x += 0x9E3779B97F4A7C15ull;
    x = (x ^ (x >> 30)) * 0xBF58476D1CE4E5B9ull;
    x = (x ^ (x >> 27)) * 0x94D049BB133111EBull;
    return x ^ (x >> 31);
}
static uint64_t hash_key(const int64_t *key, int k) {
    uint64_t h = 0x12345678ull;
    for (int i = 0; i < k; i++) h = mix64(h ^ (uint64_t)key[i]);
    return h;
}
static int map_init(ormap *m, int k, int64_t expect) {
    memset(m, 0, sizeof *m);
    m->k = k;
    m->nbuckets = 16;
    while (m->nbuckets < 2 * expect) m->nbuckets <<= 1;
    m->cap = expect > 16 ? expect : 16;
    m->heads = malloc(sizeof(int64_t) * m->nbuckets);
    m->keys = malloc(sizeof(int64_t) * m->cap * k);
    m->next = malloc(sizeof(int64_t) * m->cap);
    m->val = malloc(sizeof(int64_t) * m->cap);
    if (!m->heads || !m->keys || !m->next || !m->val) return OR_NOMEM;
    for (int64_t i = 0; i < m->nbuckets; i++) m->heads[i] = -1;
    return OR_OK;
}
static void map_free(ormap *m) {
    free(m->heads); free(m->keys); free(m->next); free(m->val);
    memset(m, 0, sizeof *m);
}
static int64_t map_append(ormap *m, const int64_t *key, int64_t val) {
    if (m->n == m->cap) {
        int64_t nc = m->cap * 2;
        int64_t *nk = realloc(m->keys, sizeof(int64_t) * nc * m->k);
        if (!nk) return OR_NOMEM;
        m->keys = nk;
        int64_t *nn = realloc(m->next, sizeof(int64_t) * nc);
        if (!nn) return OR_NOMEM;
        m->next = nn;
        int64_t *nv = realloc(m->val, sizeof(int64_t) * nc);
        if (!nv) return OR_NOMEM;
        m->val = nv;
        m->cap = nc;
    }
    int64_t e = m->n++;
    memcpy(m->keys + e * m->k, key, sizeof(int64_t) * m->k);
    m->val[e] = val;
    uint64_t b = hash_key(key, m->k) & (uint64_t)(m->nbuckets - 1);
    m->next[e] = m->heads[b];
    m->heads[b] = e;
    return e;
}
static int key_eq(const int64_t *a, const int64_t *b, int k) {
    for (int i = 0; i < k; i++) if (a[i] != b[i]) return 0;
    return 1;
}
/* First entry with this key, or -1. Continue a multimap walk with map_next_same. */
static int64_t map_first(const ormap *m, const int64_t *key) {
    uint64_t b = hash_key(key, m->k) & (uint64_t)(m->nbuckets - 1);
    for (int64_t e = m->heads[b]; e >= 0; e = m->next[e])
        if (key_eq(m->keys + e * m->k, key, m->k)) return e;
    return -1;
}
static int64_t map_next_same(const ormap *m, int64_t e, const int64_t *key) {
    for (e = m->next[e]; e >= 0; e = m->next[e])
        if (key_eq(m->keys + e * m->k, key, m->k)) return e;
    return -1;
}

/* ---------------------------------------------------------------- CH Q6 -- */
int oracle_q6(const or_order_line *ol, int64_t d_lo, int64_t d_hi, int64_t q_lo, int64_t q_hi,
              int64_t *revenue, int32_t *revenue_is_null, int64_t *count) {
    int64_t sum = 0, cnt = 0;
    for (int64_t r = 0; r < ol->n; r++) {                       /* scan order_line */
        sqlbool p = sql_and(sql_and(ts_ge(ol->delivery_d[r], d_lo), ts_lt(ol->delivery_d[r], d_hi)),
                            between(ol->quantity[r], q_lo, q_hi));
        if (p != SQL_TRUE) continue;                             /* WHERE keeps TRUE only */
        if (__builtin_add_overflow(sum, ol->amount[r], &sum)) return OR_OVERFLOW;
        cnt++;
    }
    *revenue = cnt ? sum : 0;
    *revenue_is_null = cnt == 0;                                 /* SUM(empty) IS NULL */
    *count = cnt;
    return OR_OK;
}

/* ---------------------------------------------------------------- CH Q1 -- */
typedef struct { int64_t key, sum_qty, sum_amount, count; } q1_group;

static int cmp_q1(const void *a, const void *b) {
    int64_t x = ((const q1_group *)a)->key, y = ((const q1_group *)b)->key;
    return (x > y) - (x < y);
}

int64_t oracle_q1(const or_order_line *ol, int64_t cutoff, int64_t cap,
                  int32_t *ol_number, int64_t *sum_qty, int64_t *sum_amount,
                  double *avg_qty, double *avg_amount, int64_t *count_order) {
    ormap m;
    if (map_init(&m, 1, 64) != OR_OK) { map_free(&m); return OR_NOMEM; }
    int64_t ngroups = 0, gcap = 64;
    q1_group *g = malloc(sizeof(q1_group) * gcap);
    if (!g) { map_free(&m); return OR_NOMEM; }
    for (int64_t r = 0; r < ol->n; r++) {                       /* scan order_line */
        if (ts_gt(ol->delivery_d[r], cutoff) != SQL_TRUE) continue;   /* WHERE */
        int64_t key = ol->number[r];                             /* GROUP BY ol_number */
        int64_t e = map_first(&m, &key), gi;
        if (e < 0) {
            if (ngroups == gcap) {
                gcap *= 2;
                q1_group *ng = realloc(g, sizeof(q1_group) * gcap);
                if (!ng) { free(g); map_free(&m); return OR_NOMEM; }
                g = ng;
            }
            gi = ngroups++;
            g[gi].key = key; g[gi].sum_qty = 0; g[gi].sum_amount = 0; g[gi].count = 0;
            if (map_append(&m, &key, gi) < 0) { free(g); map_free(&m); return OR_NOMEM; }
        } else {
            gi = m.val[e];
        }
        if (__builtin_add_overflow(g[gi].sum_qty, (int64_t)ol->quantity[r], &g[gi].sum_qty) ||
            __builtin_add_overflow(g[gi].sum_amount, ol->amount[r], &g[gi].sum_amount)) {
            free(g); map_free(&m); return OR_OVERFLOW;
        }
        g[gi].count++;
    }
    qsort(g, (size_t)ngroups, sizeof(q1_group), cmp_q1);        /* ORDER BY ol_number */
    for (int64_t i = 0; i < ngroups && i < cap; i++) {
        ol_number[i] = (int32_t)g[i].key;
        sum_qty[i] = g[i].sum_qty;
        sum_amount[i] = g[i].sum_amount;
        count_order[i] = g[i].count;
        avg_qty[i] = (double)g[i].sum_qty / (double)g[i].count;                 /* AVG = SUM/COUNT */
        avg_amount[i] = ((double)g[i].sum_amount / (double)g[i].count) / 100.0; /* cents -> units */
    }
    free(g);
    map_free(&m);
    return ngroups;
}

/* --------------------------------------------------------------- CH Q18 -- */
/* GROUP BY o_id, o_w_id, o_d_id, c_id, c_last, o_entry_d, o_ol_cnt */
enum { G_O_ID, G_O_W_ID, G_O_D_ID, G_C_ID, G_C_LAST, G_O_ENTRY_D, G_O_OL_CNT, G_NKEY };
typedef struct { int64_t key[G_NKEY]; int64_t amount_sum; } q18_group;

static int cmp_i64(int64_t x, int64_t y) { return (x > y) - (x < y); }
static int cmp_q18(const void *pa, const void *pb) {
    const q18_group *a = pa, *b = pb;
    int c;
    if ((c = cmp_i64(b->amount_sum, a->amount_sum))) return c;          /* amount_sum DESC */
    if ((c = cmp_i64(a->key[G_O_ENTRY_D], b->key[G_O_ENTRY_D]))) return c;  /* o_entry_d ASC */
    static const int tie[] = {G_O_W_ID, G_O_D_ID, G_O_ID, G_C_ID, G_C_LAST, G_O_OL_CNT};
    for (int i = 0; i < 6; i++)
        if ((c = cmp_i64(a->key[tie[i]], b->key[tie[i]]))) return c;
    return 0;
}

int64_t oracle_q18(const or_customer *c, const or_orders *o, const or_order_line *ol,
                   int64_t having, int64_t cap,
                   int32_t *c_last, int32_t *c_id, int32_t *o_id, int64_t *o_entry_d,
                   int32_t *o_ol_cnt, int64_t *amount_sum, int32_t *o_w_id, int32_t *o_d_id) {
    ormap hc, ho, hg;
    int st = OR_OK;
    int64_t ngroups = 0, gcap = 1024;
    q18_group *g = NULL;
    memset(&hc, 0, sizeof hc); memset(&ho, 0, sizeof ho); memset(&hg, 0, sizeof hg);
    if (map_init(&hc, 3, c->n) || map_init(&ho, 3, o->n) || map_init(&hg, G_NKEY, o->n)) {
        st = OR_NOMEM; goto done;
    }
    g = malloc(sizeof(q18_group) * gcap);
    if (!g) { st = OR_NOMEM; goto done; }

    /* Join index on customer (c_w_id, c_d_id, c_id): one entry per row (multimap). */
    for (int64_t r = 0; r < c->n; r++) {
        int64_t k[3] = {c->w_id[r], c->d_id[r], c->c_id[r]};
        if (map_append(&hc, k, r) < 0) { st = OR_NOMEM; goto done; }
    }
    /* Join index on orders (o_w_id, o_d_id, o_id). */
    for (int64_t r = 0; r < o->n; r++) {
        int64_t k[3] = {o->w_id[r], o->d_id[r], o->o_id[r]};
        if (map_append(&ho, k, r) < 0) { st = OR_NOMEM; goto done; }
    }
    /* Scan order_line; join ol_w_id = o_w_id AND ol_d_id = o_d_id AND ol_o_id = o_id,
     * then c_w_id = o_w_id AND c_d_id = o_d_id AND c_id = o_c_id; aggregate per group. */
    for (int64_t l = 0; l < ol->n; l++) {
        int64_t ko[3] = {ol->w_id[l], ol->d_id[l], ol->o_id[l]};
        for (int64_t eo = map_first(&ho, ko); eo >= 0; eo = map_next_same(&ho, eo, ko)) {
            int64_t orow = ho.val[eo];
            int64_t kc[3] = {o->w_id[orow], o->d_id[orow], o->c_id[orow]};
            for (int64_t ec = map_first(&hc, kc); ec >= 0; ec = map_next_same(&hc, ec, kc)) {
                int64_t crow = hc.val[ec];
                int64_t gk[G_NKEY];
                gk[G_O_ID] = o->o_id[orow]; gk[G_O_W_ID] = o->w_id[orow];
                gk[G_O_D_ID] = o->d_id[orow]; gk[G_C_ID] = c->c_id[crow];
                gk[G_C_LAST] = c->c_last[crow]; gk[G_O_ENTRY_D] = o->entry_d[orow];
                gk[G_O_OL_CNT] = o->ol_cnt[orow];
                int64_t eg = map_first(&hg, gk), gi;
                if (eg < 0) {
                    if (ngroups == gcap) {
                        gcap *= 2;
                        q18_group *ng = realloc(g, sizeof(q18_group) * gcap);
                        if (!ng) { st = OR_NOMEM; goto done; }
                        g = ng;
                    }
                    gi = ngroups++;
                    memcpy(g[gi].key, gk, sizeof gk);
                    g[gi].amount_sum = 0;
                    if (map_append(&hg, gk, gi) < 0) { st = OR_NOMEM; goto done; }
                } else {
                    gi = hg.val[eg];
                }
                if (__builtin_add_overflow(g[gi].amount_sum, ol->amount[l], &g[gi].amount_sum)) {
                    st = OR_OVERFLOW; goto done;
                }
            }
        }
    }
    /* HAVING SUM(ol_amount) > having (groups exist only if >= 1 joined row: inner join). */
    int64_t nout = 0;
    for (int64_t i = 0; i < ngroups; i++)
        if (g[i].amount_sum > having) g[nout++] = g[i];
    qsort(g, (size_t)nout, sizeof(q18_group), cmp_q18);          /* ORDER BY */
    for (int64_t i = 0; i < nout && i < cap; i++) {
        c_last[i] = (int32_t)g[i].key[G_C_LAST];
        c_id[i] = (int32_t)g[i].key[G_C_ID];
        o_id[i] = (int32_t)g[i].key[G_O_ID];
        o_entry_d[i] = g[i].key[G_O_ENTRY_D];
        o_ol_cnt[i] = (int32_t)g[i].key[G_O_OL_CNT];
        amount_sum[i] = g[i].amount_sum;
        o_w_id[i] = (int32_t)g[i].key[G_O_W_ID];
        o_d_id[i] = (int32_t)g[i].key[G_O_D_ID];
    }
    ngroups = nout;
done:
    free(g);
    map_free(&hc); map_free(&ho); map_free(&hg);
    return st == OR_OK ? ngroups : st;
}

/* ---------------------------------------------------------------- CH Q14 -- */
/* i_data LIKE 'prefix%': case-sensitive prefix match of the NUL-padded fixed-width string. */
static int like_prefix(const char *str, int64_t width, const char *prefix) {
    int64_t i = 0;
    for (; prefix[i]; i++)
        if (i >= width || str[i] != prefix[i]) return 0;
    return 1;
}

int oracle_q14(const or_order_line *ol, const or_item *it, int64_t d_lo, int64_t d_hi,
               const char *prefix, double *promo_revenue, int32_t *is_null, int64_t *sum_promo,
               int64_t *sum_amount, int64_t *count) {
    ormap hi;
    int st = OR_OK;
    int64_t sp = 0, sa = 0, cnt = 0;
    if (map_init(&hi, 1, it->n)) { st = OR_NOMEM; goto done; }
    for (int64_t r = 0; r < it->n; r++) {                      /* join index on item (i_id) */
        int64_t k[1] = {it->i_id[r]};
        if (map_append(&hi, k, r) < 0) { st = OR_NOMEM; goto done; }
    }
    for (int64_t l = 0; l < ol->n; l++) {                      /* scan order_line */
        sqlbool p = sql_and(ts_ge(ol->delivery_d[l], d_lo), ts_lt(ol->delivery_d[l], d_hi));
        if (p != SQL_TRUE) continue;
        int64_t k[1] = {ol->i_id[l]};
        for (int64_t e = map_first(&hi, k); e >= 0; e = map_next_same(&hi, e, k)) {  /* ol_i_id = i_id */
            int64_t irow = hi.val[e];
            int64_t promo = like_prefix(it->i_data + irow * it->width, it->width, prefix) ? ol->amount[l] : 0;
            if (__builtin_add_overflow(sp, promo, &sp) ||
                __builtin_add_overflow(sa, ol->amount[l], &sa)) { st = OR_OVERFLOW; goto done; }
            cnt++;
        }
    }
    *is_null = cnt == 0;                                        /* SUM(empty) IS NULL -> NULL */
    *promo_revenue = cnt ? (100.0 * (double)sp) / (100.0 + (double)sa) : 0.0;
    *sum_promo = sp;
    *sum_amount = sa;
    *count = cnt;
done:
    map_free(&hi);
    return st;
}

/* ------------------------------------------------------- Q12 / Q4 groups -- */
typedef struct { int64_t key, a, b; } small_group;

static int cmp_small(const void *x, const void *y) {
    int64_t a = ((const small_group *)x)->key, b = ((const small_group *)y)->key;
    return (a > b) - (a < b);
}

/* find-or-insert the group of `key` (GROUP BY o_ol_cnt) */
static int64_t group_of(ormap *m, small_group **g, int64_t *n, int64_t *cap, int64_t key) {
    int64_t k[1] = {key};
    int64_t e = map_first(m, k);
    if (e >= 0) return m->val[e];
    if (*n == *cap) {
        *cap *= 2;
        small_group *ng = realloc(*g, sizeof(small_group) * *cap);
        if (!ng) return OR_NOMEM;
        *g = ng;
    }
    int64_t gi = (*n)++;
    (*g)[gi].key = key; (*g)[gi].a = 0; (*g)[gi].b = 0;
    if (map_append(m, k, gi) < 0) return OR_NOMEM;
    return gi;
}

/* carrier = 1 OR carrier = 2 (NULL -> UNKNOWN); carrier <> 1 AND carrier <> 2 (NULL -> UNKNOWN) */
static sqlbool carrier_eq(int32_t c, int32_t v) { return c == -1 ? SQL_UNKNOWN : (c == v ? SQL_TRUE : SQL_FALSE); }
static sqlbool sql_or(sqlbool a, sqlbool b) {
    if (a == SQL_TRUE || b == SQL_TRUE) return SQL_TRUE;
    if (a == SQL_UNKNOWN || b == SQL_UNKNOWN) return SQL_UNKNOWN;
    return SQL_FALSE;
}
static sqlbool sql_not(sqlbool a) { return a == SQL_UNKNOWN ? SQL_UNKNOWN : (a == SQL_TRUE ? SQL_FALSE : SQL_TRUE); }

int64_t oracle_q12(const or_orders *o, const or_order_line *ol, int64_t d_hi, int64_t cap,
                   int32_t *o_ol_cnt, int64_t *high_line_count, int64_t *low_line_count) {
    ormap ho, hg;
    int st = OR_OK;
    int64_t ng = 0, gcap = 64;
    small_group *g = malloc(sizeof(small_group) * gcap);
    memset(&ho, 0, sizeof ho); memset(&hg, 0, sizeof hg);
    if (!g || map_init(&ho, 3, o->n) || map_init(&hg, 1, 64)) { st = OR_NOMEM; goto done; }
    for (int64_t r = 0; r < o->n; r++) {                       /* join index on orders */
        int64_t k[3] = {o->w_id[r], o->d_id[r], o->o_id[r]};
        if (map_append(&ho, k, r) < 0) { st = OR_NOMEM; goto done; }
    }
    for (int64_t l = 0; l < ol->n; l++) {                      /* scan order_line */
        int64_t k[3] = {ol->w_id[l], ol->d_id[l], ol->o_id[l]};
        for (int64_t e = map_first(&ho, k); e >= 0; e = map_next_same(&ho, e, k)) {
            int64_t orow = ho.val[e];
            /* o_entry_d <= ol_delivery_d AND ol_delivery_d < d_hi (NULL delivery -> UNKNOWN) */
            sqlbool p = sql_and(sql_not(ts_lt(ol->delivery_d[l], o->entry_d[orow])),
                                ts_lt(ol->delivery_d[l], d_hi));
            if (p != SQL_TRUE) continue;
            int64_t gi = group_of(&hg, &g, &ng, &gcap, o->ol_cnt[orow]);
            if (gi < 0) { st = OR_NOMEM; goto done; }
            int32_t c = o->carrier_id[orow];
            if (sql_or(carrier_eq(c, 1), carrier_eq(c, 2)) == SQL_TRUE) g[gi].a++;
            if (sql_and(sql_not(carrier_eq(c, 1)), sql_not(carrier_eq(c, 2))) == SQL_TRUE) g[gi].b++;
        }
    }
    qsort(g, (size_t)ng, sizeof(small_group), cmp_small);       /* ORDER BY o_ol_cnt */
    for (int64_t i = 0; i < ng && i < cap; i++) {
        o_ol_cnt[i] = (int32_t)g[i].key;
        high_line_count[i] = g[i].a;
        low_line_count[i] = g[i].b;
    }
done:
    free(g);
    map_free(&ho); map_free(&hg);
    return st == OR_OK ? ng : st;
}

int64_t oracle_q4(const or_orders *o, const or_order_line *ol, int64_t e_lo, int64_t e_hi,
                  int64_t cap, int32_t *o_ol_cnt, int64_t *order_count) {
    ormap hl, hg;
    int st = OR_OK;
    int64_t ng = 0, gcap = 64;
    small_group *g = malloc(sizeof(small_group) * gcap);
    memset(&hl, 0, sizeof hl); memset(&hg, 0, sizeof hg);
    if (!g || map_init(&hl, 3, ol->n) || map_init(&hg, 1, 64)) { st = OR_NOMEM; goto done; }
    for (int64_t l = 0; l < ol->n; l++) {                      /* index on order_line (w, d, o) */
        int64_t k[3] = {ol->w_id[l], ol->d_id[l], ol->o_id[l]};
        if (map_append(&hl, k, l) < 0) { st = OR_NOMEM; goto done; }
    }
    for (int64_t r = 0; r < o->n; r++) {                       /* scan orders */
        /* o_entry_d >= e_lo AND o_entry_d < e_hi (entry is never NULL) */
        if (!(o->entry_d[r] >= e_lo && o->entry_d[r] < e_hi)) continue;
        int exists = 0;                                          /* EXISTS (correlated) */
        int64_t k[3] = {o->w_id[r], o->d_id[r], o->o_id[r]};
        for (int64_t e = map_first(&hl, k); e >= 0 && !exists; e = map_next_same(&hl, e, k))
            exists = ts_ge(ol->delivery_d[hl.val[e]], o->entry_d[r]) == SQL_TRUE;
        if (!exists) continue;
        int64_t gi = group_of(&hg, &g, &ng, &gcap, o->ol_cnt[r]);
        if (gi < 0) { st = OR_NOMEM; goto done; }
        g[gi].a++;
    }
    qsort(g, (size_t)ng, sizeof(small_group), cmp_small);
    for (int64_t i = 0; i < ng && i < cap; i++) {
        o_ol_cnt[i] = (int32_t)g[i].key;
        order_count[i] = g[i].a;
    }
done:
    free(g);
    map_free(&hl); map_free(&hg);
    return st == OR_OK ? ng : st;
}

/* ----------------------------------------------------------------- CH Q3 -- */
/* GROUP BY ol_o_id, ol_w_id, ol_d_id, o_entry_d */
enum { G3_O_ID, G3_W_ID, G3_D_ID, G3_ENTRY_D, G3_NKEY };
typedef struct { int64_t key[G3_NKEY]; int64_t revenue; } q3_group;

static int cmp_q3(const void *pa, const void *pb) {
    const q3_group *a = pa, *b = pb;
    int c;
    if ((c = cmp_i64(b->revenue, a->revenue))) return c;                     /* revenue DESC */
    if ((c = cmp_i64(a->key[G3_ENTRY_D], b->key[G3_ENTRY_D]))) return c;      /* o_entry_d ASC */
    static const int tie[] = {G3_W_ID, G3_D_ID, G3_O_ID};                     /* R33 */
    for (int i = 0; i < 3; i++)
        if ((c = cmp_i64(a->key[tie[i]], b->key[tie[i]]))) return c;
    return 0;
}

int64_t oracle_q3(const or_customer *c, const or_new_order *no, const or_orders *o,
                  const or_order_line *ol, int64_t entry_lo, const char *prefix, int64_t cap,
                  int32_t *ol_o_id, int32_t *ol_w_id, int32_t *ol_d_id, int64_t *revenue,
                  int64_t *o_entry_d) {
    ormap hc, hn, ho, hg;
    int st = OR_OK;
    int64_t ngroups = 0, gcap = 1024;
    q3_group *g = NULL;
    memset(&hc, 0, sizeof hc); memset(&hn, 0, sizeof hn);
    memset(&ho, 0, sizeof ho); memset(&hg, 0, sizeof hg);
    if (map_init(&hc, 3, c->n) || map_init(&hn, 3, no->n) || map_init(&ho, 3, o->n) ||
        map_init(&hg, G3_NKEY, 1024)) { st = OR_NOMEM; goto done; }
    g = malloc(sizeof(q3_group) * gcap);
    if (!g) { st = OR_NOMEM; goto done; }
    /* join indexes (multimaps, every row inserted): customer (c_w_id, c_d_id, c_id),
     * new_order (no_w_id, no_d_id, no_o_id), orders (o_w_id, o_d_id, o_id) */
    for (int64_t r = 0; r < c->n; r++) {
        int64_t k[3] = {c->w_id[r], c->d_id[r], c->c_id[r]};
        if (map_append(&hc, k, r) < 0) { st = OR_NOMEM; goto done; }
    }
    for (int64_t r = 0; r < no->n; r++) {
        int64_t k[3] = {no->w_id[r], no->d_id[r], no->o_id[r]};
        if (map_append(&hn, k, r) < 0) { st = OR_NOMEM; goto done; }
    }
    for (int64_t r = 0; r < o->n; r++) {
        int64_t k[3] = {o->w_id[r], o->d_id[r], o->o_id[r]};
        if (map_append(&ho, k, r) < 0) { st = OR_NOMEM; goto done; }
    }
    /* scan order_line; ol = o on (w, d, o_id); o_entry_d > entry_lo; no = o on (w, d, o_id);
     * c = o on (w, d, c_id) with c_state LIKE 'prefix%'; one joined tuple per combination */
    for (int64_t l = 0; l < ol->n; l++) {
        int64_t ko[3] = {ol->w_id[l], ol->d_id[l], ol->o_id[l]};
        for (int64_t eo = map_first(&ho, ko); eo >= 0; eo = map_next_same(&ho, eo, ko)) {
            int64_t orow = ho.val[eo];
            if (ts_gt(o->entry_d[orow], entry_lo) != SQL_TRUE) continue;
            int64_t kn[3] = {o->w_id[orow], o->d_id[orow], o->o_id[orow]};
            for (int64_t en = map_first(&hn, kn); en >= 0; en = map_next_same(&hn, en, kn)) {
                int64_t kc[3] = {o->w_id[orow], o->d_id[orow], o->c_id[orow]};
                for (int64_t ec = map_first(&hc, kc); ec >= 0; ec = map_next_same(&hc, ec, kc)) {
                    int64_t crow = hc.val[ec];
                    if (!like_prefix(c->state + crow * c->state_width, c->state_width, prefix)) continue;
                    int64_t gk[G3_NKEY];
                    gk[G3_O_ID] = ol->o_id[l]; gk[G3_W_ID] = ol->w_id[l]; gk[G3_D_ID] = ol->d_id[l];
                    gk[G3_ENTRY_D] = o->entry_d[orow];
                    int64_t eg = map_first(&hg, gk), gi;
                    if (eg < 0) {
                        if (ngroups == gcap) {
                            gcap *= 2;
                            q3_group *ng = realloc(g, sizeof(q3_group) * gcap);
                            if (!ng) { st = OR_NOMEM; goto done; }
                            g = ng;
                        }
                        gi = ngroups++;
                        memcpy(g[gi].key, gk, sizeof gk);
                        g[gi].revenue = 0;
                        if (map_append(&hg, gk, gi) < 0) { st = OR_NOMEM; goto done; }
                    } else {
                        gi = hg.val[eg];
                    }
                    if (__builtin_add_overflow(g[gi].revenue, ol->amount[l], &g[gi].revenue)) {
                        st = OR_OVERFLOW; goto done;
                    }
                }
            }
        }
    }
    qsort(g, (size_t)ngroups, sizeof(q3_group), cmp_q3);               /* ORDER BY */
    for (int64_t i = 0; i < ngroups && i < cap; i++) {
        ol_o_id[i] = (int32_t)g[i].key[G3_O_ID];
        ol_w_id[i] = (int32_t)g[i].key[G3_W_ID];
        ol_d_id[i] = (int32_t)g[i].key[G3_D_ID];
        revenue[i] = g[i].revenue;
        o_entry_d[i] = g[i].key[G3_ENTRY_D];
    }
done:
    free(g);
    map_free(&hc); map_free(&hn); map_free(&ho); map_free(&hg);
    return st == OR_OK ? ngroups : st;
}

/* ------------------------------------------------ layout scan (NEXT-3) -- */
/* Address of record r, attribute c in each layout, as PAPER.md §5.3 describes them (L968-972). */
static int64_t layout_addr(int layout, int64_t r, int64_t c, int64_t ncols, int64_t col_stride,
                           int64_t pax_rows) {
    if (layout == 1) return c * col_stride + r;                                       /* DSM */
    if (layout == 2) return (r / pax_rows) * ncols * pax_rows + c * pax_rows + r % pax_rows;  /* PAX */
    return r * ncols + c;                                                             /* NSM */
}

int oracle_layout_sum(const int32_t *data, int layout, int64_t nrows, int64_t ncols, int64_t col_stride,
                      int64_t pax_rows, uint64_t col_mask, int64_t *sum, int32_t *is_null) {
    int64_t total = 0;
    for (int64_t r = 0; r < nrows; r++) {                 /* scan, one record at a time */
        int64_t row = 0;                                   /* col_c1 + ... + col_cN */
        for (int64_t c = 0; c < ncols; c++)
            if (col_mask >> c & 1) row += data[layout_addr(layout, r, c, ncols, col_stride, pax_rows)];
        if (__builtin_add_overflow(total, row, &total)) return OR_OVERFLOW;
    }
    *sum = total;
    *is_null = nrows == 0;                                 /* SUM over no rows is NULL */
    return OR_OK;
}
