"""Boundary pins for the CPU oracle (``-m "not gpu"``).

Every predicate bound of the hot-path queries is exercised EXACTLY ON the bound, by a
hand-derived fixture (tests/golden/boundaries_ch.json, each case with its derivation) and by
SQLite running the literal CH SQL on the same rows:
  * Q6  ``ol_delivery_d >= d_lo AND ol_delivery_d < d_hi`` (half-open; PAPER.md L687-688 is the
    TPC-H analogue) and ``ol_quantity BETWEEN q_lo AND q_hi`` (inclusive, R12);
  * Q1  ``ol_delivery_d > cutoff`` (strict);
  * Q18 ``HAVING SUM(ol_amount) > 200`` (strict; a group summing to exactly the threshold is out);
  * NULL dates (R5) against constants equal to the sentinel's own value INT64_MIN.
Also the Q18 tie-break (tests/golden/tiebreak_q18.json: ties on (amount_sum, o_entry_d) across
warehouses and districts). The mutations these catch (each fails at least one test here): HAVING '>' -> '>=',
Q6 '<' -> '<=' on d_hi, '>=' -> '>' on d_lo, Q1 '>' -> '>=', BETWEEN made exclusive, and a NULL
test dropped from any one of the 3-valued comparison helpers (pinned against SQLite directly,
because inside Q6 a dropped NULL test in one helper is masked by the other's UNKNOWN).
"""
import math

import numpy as np
import pytest

import oracle
from chref import (brute_q1, brute_q6, brute_q18, golden, iso_us, sqlite_load, sqlite_q1,
                   sqlite_q6, sqlite_q18, ts_param)

Q18_NAMES = ["c_last", "c_id", "o_id", "o_entry_d", "o_ol_cnt", "amount_sum", "o_w_id", "o_d_id"]
FIXTURE = "boundaries_ch.json"
I64_MIN, I64_MAX = np.iinfo(np.int64).min, np.iinfo(np.int64).max


def q18_tuples(r):
    return list(zip(*[r[k].tolist() for k in Q18_NAMES]))


def q1_rows(r):
    return list(zip(r["ol_number"].tolist(), r["sum_qty"].tolist(), r["sum_amount"].tolist(),
                    r["avg_qty"].tolist(), r["avg_amount"].tolist(), r["count_order"].tolist()))


def assert_q1(got, want):
    assert len(got) == len(want)
    for g, w in zip(got, want):
        assert (g[0], g[1], g[2], g[5]) == (w[0], w[1], w[2], w[5])
        assert math.isclose(g[3], w[3], rel_tol=1e-9, abs_tol=0)
        assert math.isclose(g[4], w[4], rel_tol=1e-9, abs_tol=0)


def want_q1(case):
    return [(w["ol_number"], w["sum_qty"], w["sum_amount"], w["avg_qty"], w["avg_amount"],
             w["count_order"]) for w in case["rows"]]


def want_q18(case):
    return [(w["c_last"], w["c_id"], w["o_id"], iso_us(w["o_entry_d"]), w["o_ol_cnt"],
             w["amount_sum"], w["o_w_id"], w["o_d_id"]) for w in case["rows"]]


def test_fixture_rows_sit_on_the_ch_bounds():
    """The fixture's boundary rows are where its _about says (guards the fixture itself)."""
    t, _ = golden(FIXTURE)
    d = t["order_line"]["ol_delivery_d"].tolist()
    assert d[0] == iso_us("2020-01-01T00:00:00")          # = Q6 d_hi
    assert d[1] == iso_us("2007-01-02T00:00:00")          # = Q1 cutoff
    assert d[2] == iso_us("1999-01-01T00:00:00")          # = Q6 d_lo
    assert d[4] == d[1] + 1 and d[7] == d[0] - 1
    assert d[3] == I64_MIN and d[5] == I64_MIN            # NULL
    q = t["order_line"]["ol_quantity"].tolist()
    assert (q[7], q[8], q[9]) == (100000, 0, 100001)      # q_hi, q_lo - 1, q_hi + 1


def test_boundaries_q6_golden():
    t, exp = golden(FIXTURE)
    for case in exp["q6"]:
        p = [ts_param(v) for v in case["params"]]
        r = oracle.q6(t, *p)
        assert (r["revenue"], r["count"]) == (case["revenue"], case["count"]), case["_why"]


def test_boundaries_q1_golden():
    t, exp = golden(FIXTURE)
    for case in exp["q1"]:
        assert_q1(q1_rows(oracle.q1(t, ts_param(case["params"][0]))), want_q1(case))


def test_boundaries_q18_golden():
    t, exp = golden(FIXTURE)
    for case in exp["q18"]:
        assert q18_tuples(oracle.q18(t, case["params"][0])) == want_q18(case), case["_why"]


def test_boundaries_fixture_vs_sqlite_and_brute_force():
    """The hand-derived values are also what SQLite's CH SQL and the nested loops produce."""
    t, exp = golden(FIXTURE)
    db = sqlite_load(t)
    for case in exp["q6"]:
        p = [ts_param(v) for v in case["params"]]
        assert sqlite_q6(db, *p) == case["revenue"], case["_why"]
        assert brute_q6(t, *p) == (case["revenue"], case["count"]), case["_why"]
    for case in exp["q1"]:
        c = ts_param(case["params"][0])
        assert_q1(sqlite_q1(db, c), want_q1(case))
        assert_q1(brute_q1(t, c), want_q1(case))
    for case in exp["q18"]:
        assert sqlite_q18(db, case["params"][0]) == want_q18(case), case["_why"]
        assert brute_q18(t, case["params"][0]) == want_q18(case), case["_why"]


def test_q18_tiebreak_golden():
    """tests/golden/tiebreak_q18.json (hand-derived): rows tied on (amount_sum, o_entry_d) come in
    (o_w_id, o_d_id, o_id) order (R33). The brute-force evaluation implements the same
    reading; SQLite runs the literal CH SQL, whose ORDER BY stops at o_entry_d, so it fixes the
    sequence of (amount_sum, o_entry_d) and the row set, not the order inside a tie."""
    t, exp = golden("tiebreak_q18.json")
    db = sqlite_load(t)
    for case in exp["q18"]:
        want = want_q18(case)
        assert q18_tuples(oracle.q18(t, case["params"][0])) == want, case["_why"]
        assert brute_q18(t, case["params"][0]) == want, case["_why"]
        lite = sqlite_q18(db, case["params"][0])
        assert sorted(lite) == sorted(want)
        assert [(r[5], r[3]) for r in lite] == [(r[5], r[3]) for r in want]


@pytest.mark.parametrize("op", [">=", "<", ">"])
def test_ts_compare_three_valued_logic_matches_sqlite(op):
    """The oracle's 3-valued timestamp comparisons equal SQLite's on NULL and on every
    neighbour of the bound, with constants at both int64 extremes (incl. the NULL sentinel's
    value INT64_MIN as a real constant: NULL >= INT64_MIN is UNKNOWN, not TRUE)."""
    import sqlite3
    db = sqlite3.connect(":memory:")
    consts = [I64_MIN, I64_MIN + 1, -1, 0, 1, iso_us("2007-01-02T00:00:00"), I64_MAX - 1, I64_MAX]
    for c in consts:
        vals = [None] + [v for v in (c - 1, c, c + 1) if I64_MIN < v <= I64_MAX or v == I64_MIN]
        for v in vals:
            if v == I64_MIN:
                continue  # INT64_MIN is the NULL sentinel, not a storable timestamp (R5)
            (s,) = db.execute(f"SELECT ? {op} ?", (v, c)).fetchone()
            want = None if s is None else bool(s)
            assert oracle.ts_cmp(op, v, c) is want if want is None else oracle.ts_cmp(op, v, c) == want, (op, v, c)
