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
]

TESTS = ["tests/test_oracle.py", "tests/test_oracle_boundaries.py"]


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
