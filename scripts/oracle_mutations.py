"""Mutation check of the CPU oracle's pins (CPU only, no GPU).

Applies one plausible mistake at a time to a scratch copy of oracle/oracle.c and runs the oracle's
CPU pin tests against it; every mutation must make at least one test fail ("killed"). Writes a
summary line per mutation (and profiles/oracle_mutations_<tag>.txt with --out).
"""
import argparse
import os
import shutil
import subprocess
import sys
import tempfile

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

# (name, exact text in oracle.c, replacement)
MUTATIONS = [
    ("Q18 HAVING > -> >=", "if (g[i].amount_sum > having)", "if (g[i].amount_sum >= having)"),
    ("ts_ge drops its NULL test",
     "static sqlbool ts_ge(int64_t v, int64_t c) { return v == OR_NULL_TS ? SQL_UNKNOWN : (v >= c ? SQL_TRUE : SQL_FALSE); }",
     "static sqlbool ts_ge(int64_t v, int64_t c) { return (v >= c ? SQL_TRUE : SQL_FALSE); }"),
    ("ts_lt drops its NULL test",
     "static sqlbool ts_lt(int64_t v, int64_t c) { return v == OR_NULL_TS ? SQL_UNKNOWN : (v < c ? SQL_TRUE : SQL_FALSE); }",
     "static sqlbool ts_lt(int64_t v, int64_t c) { return (v < c ? SQL_TRUE : SQL_FALSE); }"),
    ("ts_gt drops its NULL test",
     "static sqlbool ts_gt(int64_t v, int64_t c) { return v == OR_NULL_TS ? SQL_UNKNOWN : (v > c ? SQL_TRUE : SQL_FALSE); }",
     "static sqlbool ts_gt(int64_t v, int64_t c) { return (v > c ? SQL_TRUE : SQL_FALSE); }"),
    ("Q6 d_hi '<' -> '<=' inlined",
     "ts_lt(ol->delivery_d[r], d_hi)),",
     "(ol->delivery_d[r] <= d_hi ? SQL_TRUE : SQL_FALSE)),"),
    ("Q6 d_lo '>=' -> '>' inlined",
     "sql_and(sql_and(ts_ge(ol->delivery_d[r], d_lo),",
     "sql_and(sql_and((ol->delivery_d[r] != OR_NULL_TS && ol->delivery_d[r] > d_lo ? SQL_TRUE : SQL_FALSE),"),
    ("Q1 cutoff '>' -> '>=' inlined",
     "if (ts_gt(ol->delivery_d[r], cutoff) != SQL_TRUE) continue;",
     "if (!(ol->delivery_d[r] != OR_NULL_TS && ol->delivery_d[r] >= cutoff)) continue;"),
    ("BETWEEN upper bound exclusive", "x <= hi ? SQL_TRUE", "x < hi ? SQL_TRUE"),
    ("BETWEEN lower bound exclusive", "x >= lo ? SQL_TRUE", "x > lo ? SQL_TRUE"),
    ("Q1 AVG amount without /100", "/ (double)g[i].count) / 100.0;", "/ (double)g[i].count);"),
    ("Q18 ORDER BY amount ASC", "if ((c = cmp_i64(b->amount_sum, a->amount_sum))) return c;",
     "if ((c = cmp_i64(a->amount_sum, b->amount_sum))) return c;"),
    ("Q6 empty SUM not NULL", "*revenue_is_null = cnt == 0;", "*revenue_is_null = 0;"),
    # round 2, wider sweep: joins, group keys, tie-breaks, the NEXT-2 queries and the layout scan
    ("Q6 sums quantity instead of amount", "if (__builtin_add_overflow(sum, ol->amount[r], &sum)) return OR_OVERFLOW;",
     "if (__builtin_add_overflow(sum, (int64_t)ol->quantity[r], &sum)) return OR_OVERFLOW;"),
    ("Q1 AVG qty over amount", "avg_qty[i] = (double)g[i].sum_qty / (double)g[i].count;",
     "avg_qty[i] = (double)g[i].sum_amount / (double)g[i].count;"),
    ("Q1 groups by ol_o_id", "int64_t key = ol->number[r];", "int64_t key = ol->o_id[r];"),
    ("Q1 ORDER BY ol_number DESC", "return (x > y) - (x < y);\n}\n\nint64_t oracle_q1",
     "return (x < y) - (x > y);\n}\n\nint64_t oracle_q1"),
    ("Q18 orders join ignores ol_d_id", "int64_t ko[3] = {ol->w_id[l], ol->d_id[l], ol->o_id[l]};\n        for (int64_t eo = map_first(&ho, ko); eo >= 0; eo = map_next_same(&ho, eo, ko)) {\n            int64_t orow = ho.val[eo];\n            int64_t kc[3]",
     "int64_t ko[3] = {ol->w_id[l], 1, ol->o_id[l]};\n        for (int64_t eo = map_first(&ho, ko); eo >= 0; eo = map_next_same(&ho, eo, ko)) {\n            int64_t orow = ho.val[eo];\n            int64_t kc[3]"),
    ("Q18 customer join on o_id instead of o_c_id", "int64_t kc[3] = {o->w_id[orow], o->d_id[orow], o->c_id[orow]};\n            for (int64_t ec = map_first(&hc, kc); ec >= 0; ec = map_next_same(&hc, ec, kc)) {\n                int64_t crow = hc.val[ec];\n                int64_t gk[G_NKEY];",
     "int64_t kc[3] = {o->w_id[orow], o->d_id[orow], o->o_id[orow]};\n            for (int64_t ec = map_first(&hc, kc); ec >= 0; ec = map_next_same(&hc, ec, kc)) {\n                int64_t crow = hc.val[ec];\n                int64_t gk[G_NKEY];"),
    ("Q18 o_entry_d tie-break DESC", "if ((c = cmp_i64(a->key[G_O_ENTRY_D], b->key[G_O_ENTRY_D]))) return c;",
     "if ((c = cmp_i64(b->key[G_O_ENTRY_D], a->key[G_O_ENTRY_D]))) return c;"),
    ("Q18 w/d tie-break order swapped", "static const int tie[] = {G_O_W_ID, G_O_D_ID, G_O_ID, G_C_ID, G_C_LAST, G_O_OL_CNT};",
     "static const int tie[] = {G_O_D_ID, G_O_W_ID, G_O_ID, G_C_ID, G_C_LAST, G_O_OL_CNT};"),
    ("Q18 result c_last from c_id", "c_last[i] = (int32_t)g[i].key[G_C_LAST];", "c_last[i] = (int32_t)g[i].key[G_C_ID];"),
    ("Q14 promo formula drops the 100.0 offset", "(100.0 * (double)sp) / (100.0 + (double)sa)", "(100.0 * (double)sp) / ((double)sa)"),
    ("Q14 LIKE prefix ignores width", "if (i >= width || str[i] != prefix[i]) return 0;", "if (str[i] != prefix[i]) return 0;"),
    ("Q12 high lines: carrier 1 or 3", "if (sql_or(carrier_eq(c, 1), carrier_eq(c, 2)) == SQL_TRUE) g[gi].a++;",
     "if (sql_or(carrier_eq(c, 1), carrier_eq(c, 3)) == SQL_TRUE) g[gi].a++;"),
    ("Q12 o_entry_d <= delivery becomes <", "sqlbool p = sql_and(sql_not(ts_lt(ol->delivery_d[l], o->entry_d[orow])),",
     "sqlbool p = sql_and(ts_gt(ol->delivery_d[l], o->entry_d[orow]),"),
    ("Q4 EXISTS with delivery > entry", "exists = ts_ge(ol->delivery_d[hl.val[e]], o->entry_d[r]) == SQL_TRUE;",
     "exists = ts_gt(ol->delivery_d[hl.val[e]], o->entry_d[r]) == SQL_TRUE;"),
    ("Q4 entry window inclusive at e_hi", "if (!(o->entry_d[r] >= e_lo && o->entry_d[r] < e_hi)) continue;",
     "if (!(o->entry_d[r] >= e_lo && o->entry_d[r] <= e_hi)) continue;"),
    ("Q3 skips the new_order join", "for (int64_t en = map_first(&hn, kn); en >= 0; en = map_next_same(&hn, en, kn)) {",
     "for (int64_t en = 0; en == 0; en = -1) { (void)kn;"),
    ("Q3 o_entry_d filter '>' -> '>='", "if (ts_gt(o->entry_d[orow], entry_lo) != SQL_TRUE) continue;",
     "if (o->entry_d[orow] < entry_lo) continue;"),
    ("layout PAX minipage stride", "return (r / pax_rows) * ncols * pax_rows + c * pax_rows + r % pax_rows;",
     "return (r / pax_rows) * ncols * pax_rows + c + (r % pax_rows) * ncols;"),
    ("layout empty SUM not NULL", "*is_null = nrows == 0;", "*is_null = 0;"),
]

TESTS = ["tests/test_oracle.py", "tests/test_oracle_boundaries.py", "tests/test_oracle_next2.py",
         "tests/test_oracle_q3.py", "tests/test_oracle_layout.py"]


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    src = open(os.path.join(ROOT, "oracle", "oracle.c")).read()
    lines = []
    for name, old, new in MUTATIONS:
        if old not in src:
            lines.append(f"SKIP (text not found)  {name}")
            continue
        with tempfile.TemporaryDirectory() as d:
            for sub in ("oracle", "tests", "chgen"):
                shutil.copytree(os.path.join(ROOT, sub), os.path.join(d, sub),
                                ignore=shutil.ignore_patterns("*.so", "__pycache__"))
            with open(os.path.join(d, "oracle", "oracle.c"), "w") as f:
                f.write(src.replace(old, new, 1))
            env = dict(os.environ, PYTHONPATH=d)
            # a minimal conftest-free run: the oracle builds itself on import
            r = subprocess.run([sys.executable, "-m", "pytest", "-q", "-x", "-p", "no:cacheprovider",
                                "--noconftest", "-m", "not gpu"] + TESTS, cwd=d, env=env,
                               capture_output=True, text=True)
            verdict = "KILLED" if r.returncode != 0 else "SURVIVED"
            tail = r.stdout.strip().splitlines()[-1] if r.stdout.strip() else ""
            lines.append(f"{verdict:8s}  {name}  [{tail}]")
        print(lines[-1], flush=True)
    if a.out:
        with open(a.out, "w") as f:
            f.write("\n".join(lines) + "\n")
    return 0 if all(l.startswith("KILLED") for l in lines) else 1


if __name__ == "__main__":
    sys.exit(main())
