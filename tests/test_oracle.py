"""Pins for the CPU oracle (runs on CPU, ``-m "not gpu"``).

Each test checks the oracle against something other than itself: the hand-derived
golden fixture, SQLite running the literal CH SQL, brute-force nested loops over the
cartesian product, strict-mode closed forms of the TPC-C population, and invariants
(re-partitioning, COUNT, constant column, full window). A plausible mistake in
oracle.c — a dropped NULL test, an exclusive/inclusive bound swapped, a wrong join
column, a missing /100, a sort direction — fails at least one of them.
"""
import math

import numpy as np
import pytest

import chgen
import oracle
from chref import (Q1_CUTOFF, Q6_D_HI, Q6_D_LO, Q6_Q_HI, Q6_Q_LO, Q18_HAVING, brute_q1,
                   brute_q6, brute_q18, golden, iso_us, sqlite_load, sqlite_q1, sqlite_q6,
                   sqlite_q18, NULL_SENTINEL)

Q18_NAMES = ["c_last", "c_id", "o_id", "o_entry_d", "o_ol_cnt", "amount_sum", "o_w_id", "o_d_id"]


def q18_tuples(r):
    return list(zip(*[r[k].tolist() for k in Q18_NAMES]))


def q1_tuples(r):
    return list(zip(r["ol_number"].tolist(), r["sum_qty"].tolist(), r["sum_amount"].tolist(),
                    r["avg_qty"].tolist(), r["avg_amount"].tolist(), r["count_order"].tolist()))


def assert_q1_equal(got, want):
    assert len(got) == len(want)
    for g, w in zip(got, want):
        assert (g[0], g[1], g[2], g[5]) == (w[0], w[1], w[2], w[5])
        assert math.isclose(g[3], w[3], rel_tol=1e-9, abs_tol=0)
        assert math.isclose(g[4], w[4], rel_tol=1e-9, abs_tol=0)


# ----------------------------------------------------------------- golden --
def test_timestamp_constants_are_ch_literals():
    # '2007-01-02 00:00:00.000000' etc. as int64 µs UTC (R4), via datetime.
    assert Q1_CUTOFF == 1_167_696_000_000_000
    assert Q6_D_LO == 915_148_800_000_000
    assert Q6_D_HI == 1_577_836_800_000_000
    assert chgen.LOAD_TS == iso_us("2015-01-01T00:00:00")


def test_golden_q6():
    t, exp = golden()
    for case in exp["q6"]:
        d_lo, d_hi, q_lo, q_hi = case["params"]
        r = oracle.q6(t, iso_us(d_lo), iso_us(d_hi), q_lo, q_hi)
        assert r["revenue"] == case["revenue"]
        assert r["count"] == case["count"]


def test_golden_q1():
    t, exp = golden()
    for case in exp["q1"]:
        r = oracle.q1(t, iso_us(case["params"][0]))
        want = [(w["ol_number"], w["sum_qty"], w["sum_amount"], w["avg_qty"], w["avg_amount"],
                 w["count_order"]) for w in case["rows"]]
        assert_q1_equal(q1_tuples(r), want)


def test_golden_q18():
    t, exp = golden()
    for case in exp["q18"]:
        r = oracle.q18(t, case["params"][0])
        want = [(w["c_last"], w["c_id"], w["o_id"], iso_us(w["o_entry_d"]), w["o_ol_cnt"],
                 w["amount_sum"], w["o_w_id"], w["o_d_id"]) for w in case["rows"]]
        assert q18_tuples(r) == want


# ------------------------------------------------------------ brute force --
@pytest.mark.parametrize("seed,mode", [(1, "spread"), (7, "strict"), (3, "spread")])
def test_brute_force_tiny(seed, mode):
    t = chgen.generate(1, 2, seed=seed, mode=mode, scale=chgen.TINY)
    rng = np.random.default_rng(seed)
    for _ in range(3):
        d_lo = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
        d_hi = int(rng.integers(d_lo, chgen.TS_2025 + 40 * chgen.DAY_US))
        q_lo = int(rng.integers(0, 6))
        q_hi = int(rng.integers(q_lo, 12))
        r = oracle.q6(t, d_lo, d_hi, q_lo, q_hi)
        rev, cnt = brute_q6(t, d_lo, d_hi, q_lo, q_hi)
        assert (r["revenue"], r["count"]) == (rev, cnt)
        cutoff = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
        assert_q1_equal(q1_tuples(oracle.q1(t, cutoff)), brute_q1(t, cutoff))
    for having in (Q18_HAVING, -1, 1_000_000, 3_000_000):
        assert q18_tuples(oracle.q18(t, having)) == brute_q18(t, having)


def test_brute_force_q18_duplicates_and_orphans():
    """Non-PK data: duplicate customers and orders multiply join rows; orphans drop out."""
    t = chgen.generate(1, 2, seed=5, scale=chgen.TINY)
    c, o, ol = t["customer"], t["orders"], t["order_line"]
    # duplicate customer row 3 with a different c_last, duplicate orders row 0
    for k in c:
        c[k] = np.concatenate([c[k], c[k][3:4]])
    c["c_last"][-1] = 777
    for k in o:
        o[k] = np.concatenate([o[k], o[k][0:1]])
    # orphan order_line rows (o_id that does not exist)
    for k in ol:
        ol[k] = np.concatenate([ol[k], ol[k][0:2]])
    ol["ol_o_id"][-2:] = 9999
    for having in (-1, Q18_HAVING):
        assert q18_tuples(oracle.q18(t, having)) == brute_q18(t, having)


# ------------------------------------------------------------------ SQLite --
@pytest.mark.parametrize("W,mode,seed", [(1, "spread", 1), (2, "strict", 2), (1, "spread", 11)])
def test_sqlite_full_warehouses(W, mode, seed):
    t = chgen.generate(1, W + 1, seed=seed, mode=mode)
    db = sqlite_load(t)
    rng = np.random.default_rng(seed)
    params6 = [(Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI)]
    for _ in range(2):
        d_lo = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
        params6.append((d_lo, int(rng.integers(d_lo, chgen.TS_2025)), int(rng.integers(1, 6)),
                        int(rng.integers(5, 11))))
    for p in params6:
        assert oracle.q6(t, *p)["revenue"] == sqlite_q6(db, *p)
    for cutoff in (Q1_CUTOFF, int(rng.integers(chgen.TS_1995, chgen.TS_2025))):
        assert_q1_equal(q1_tuples(oracle.q1(t, cutoff)), sqlite_q1(db, cutoff))
    for having in (Q18_HAVING, 6_000_000):
        got = q18_tuples(oracle.q18(t, having))
        want = sqlite_q18(db, having)
        # SQLite breaks ORDER BY ties arbitrarily: compare the ordered sort keys and the row set.
        assert [(r[5], r[3]) for r in got] == [(r[5], r[3]) for r in want]
        assert sorted(got) == sorted(want)


# ------------------------------------------------------------ closed forms --
def test_strict_closed_forms():
    """TPC-C §4.3.3.1 population (SURVEY.md §8c 'What pins each part')."""
    W = 2
    t = chgen.generate(1, W + 1, mode="strict", seed=4)
    o = t["orders"]
    delivered = o["o_id"] < 2101
    # Q6: delivered lines are dated LOAD_TS (inside the window), amount 0, qty 5 -> revenue 0.
    r6 = oracle.q6(t, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI)
    assert r6["revenue"] == 0
    assert r6["count"] == int(o["o_ol_cnt"][delivered].sum())
    # Q1: count_n = #{delivered orders with ol_cnt >= n}; n <= 5 -> 21,000 W.
    r1 = oracle.q1(t, Q1_CUTOFF)
    assert r1["ol_number"].tolist() == list(range(1, 16))
    for n, sq, sa, aq, aa, cnt in q1_tuples(r1):
        want = int((o["o_ol_cnt"][delivered] >= n).sum())
        assert cnt == want
        if n <= 5:
            assert cnt == 21_000 * W
        assert sq == 5 * cnt and sa == 0 and aq == 5.0 and aa == 0.0
    # Q18: only undelivered orders (o_id >= 2101) carry money; 9,000 W of them, each with
    # >= 5 lines of U[1, 999999] cents, exceed 200.00 with overwhelming probability.
    r18 = oracle.q18(t, Q18_HAVING)
    assert len(r18["o_id"]) == 9_000 * W
    assert (r18["o_id"] >= 2101).all()
    assert (r18["o_entry_d"] == chgen.LOAD_TS).all()
    assert (np.diff(r18["amount_sum"]) <= 0).all()


# -------------------------------------------------------------- invariants --
def test_invariants_count_and_window():
    t = chgen.generate(1, 4, seed=9)
    ol = t["order_line"]
    d = ol["ol_delivery_d"]
    # (i) sum_n count_n = rows with delivery_d > cutoff (independent numpy count, NULL excluded)
    r1 = oracle.q1(t, Q1_CUTOFF)
    assert int(r1["count_order"].sum()) == int(((d != NULL_SENTINEL) & (d > Q1_CUTOFF)).sum())
    assert int(r1["sum_qty"].sum()) == int(ol["ol_quantity"][(d != NULL_SENTINEL) & (d > Q1_CUTOFF)].sum())
    # (iv) full window, full quantity range = sum of amount over non-NULL-dated rows
    r6 = oracle.q6(t, np.iinfo(np.int64).min + 1, np.iinfo(np.int64).max, -2**31, 2**31 - 1)
    assert r6["revenue"] == int(ol["ol_amount"][d != NULL_SENTINEL].sum())
    # (iii) constant column amount = 1 -> revenue = count
    t2 = {"order_line": dict(ol, ol_amount=np.ones_like(ol["ol_amount"]))}
    r = oracle.q6(t2, Q6_D_LO, Q6_D_HI, 1, 10)
    assert r["revenue"] == r["count"] > 0
    # (v) Q18 with HAVING below every sum: sum of results = sum of ol_amount over lines
    #     whose order and customer exist (all of them in generated data)
    r18 = oracle.q18(t, -1)
    assert int(r18["amount_sum"].sum()) == int(ol["ol_amount"].sum())
    assert len(r18["o_id"]) == len(t["orders"]["o_id"])


@pytest.mark.parametrize("k", [2, 3, 5])
def test_invariant_repartition(k):
    """(ii) per-warehouse-range partials merged = whole (sums are associative)."""
    W = 5
    whole = chgen.generate(1, W + 1, seed=13)
    r6 = oracle.q6(whole, Q6_D_LO, Q6_D_HI, 2, 9)
    r1 = oracle.q1(whole, Q1_CUTOFF)
    r18 = oracle.q18(whole, Q18_HAVING)
    rev, cnt, q1m, rows18 = 0, 0, {}, []
    for lo, hi in chgen.warehouse_ranges(W, k):
        part = chgen.generate(lo, hi, seed=13, with_item=False)
        p6 = oracle.q6(part, Q6_D_LO, Q6_D_HI, 2, 9)
        rev += p6["revenue"] or 0
        cnt += p6["count"]
        for n, sq, sa, _, _, c in q1_tuples(oracle.q1(part, Q1_CUTOFF)):
            m = q1m.setdefault(n, [0, 0, 0])
            m[0] += sq; m[1] += sa; m[2] += c
        rows18 += q18_tuples(oracle.q18(part, Q18_HAVING))
    assert (rev, cnt) == (r6["revenue"], r6["count"])
    assert sorted(q1m) == r1["ol_number"].tolist()
    for n, sq, sa, _, _, c in q1_tuples(r1):
        assert q1m[n] == [sq, sa, c]
    assert sorted(rows18) == sorted(q18_tuples(r18))


def test_empty_inputs():
    t = chgen.generate(1, 1, seed=1)      # zero warehouses
    assert oracle.q6(t, Q6_D_LO, Q6_D_HI, 1, 10) == {"revenue": None, "count": 0}
    assert len(oracle.q1(t, Q1_CUTOFF)["ol_number"]) == 0
    assert len(oracle.q18(t, -10)["o_id"]) == 0


def test_overflow_detected():
    ol = {"ol_w_id": np.ones(2, np.int32), "ol_d_id": np.ones(2, np.int32),
          "ol_o_id": np.ones(2, np.int32), "ol_number": np.ones(2, np.int32),
          "ol_delivery_d": np.full(2, Q6_D_LO, np.int64), "ol_quantity": np.ones(2, np.int32),
          "ol_amount": np.full(2, 2**62 + 1, np.int64)}
    with pytest.raises(OverflowError):
        oracle.q6({"order_line": ol}, Q6_D_LO, Q6_D_HI, 1, 10)
