"""Pins of the NEXT-2 oracle functions (CH Q14, Q12, Q4), none of which use
the oracle's own code: a hand-derived fixture (tests/golden/ch_next2.json), brute force over the
cartesian product on tiny tables, SQLite running the literal CH SQL (case-sensitive LIKE), and
strict-mode closed forms."""
import math

import numpy as np
import pytest

import chgen
import oracle
from chref import (brute_q4, brute_q12, brute_q14, golden_next2, iso_us, sqlite_load, sqlite_q4,
                   sqlite_q12, sqlite_q14)

Q14_LO, Q14_HI = iso_us("2007-01-02T00:00:00"), iso_us("2020-01-02T00:00:00")
Q12_HI = iso_us("2020-01-01T00:00:00")
Q4_LO, Q4_HI = iso_us("2007-01-02T00:00:00"), iso_us("2012-01-02T00:00:00")


def mutate(t, seed):
    """Make Q14/Q12/Q4 non-degenerate and hit their edge cases: promo items ('PR'), look-alikes
    ('pr', 'XPR', 'P'), NULL / 1 / 2 / other carriers, random delivery dates around the entry
    dates, and lines of missing items."""
    rng = np.random.default_rng(seed)
    t = {k: dict(v) for k, v in t.items()}
    it = t["item"]
    data = np.array(it["i_data"], dtype="S50")
    for i in range(len(data)):
        r = rng.random()
        s = bytes(data[i])
        if r < 0.25:
            s = b"PR" + s[2:]
        elif r < 0.30:
            s = b"pr" + s[2:]
        elif r < 0.35:
            s = b"XPR" + s[3:]
        elif r < 0.37:
            s = b"P"
        data[i] = s
    it["i_data"] = data
    it["i_data_p2"] = chgen.i_data_prefix2(data)
    o = t["orders"]
    o["o_carrier_id"] = rng.choice(np.array([-1, 1, 2, 3, 7], np.int32), size=len(o["o_id"]))
    ol = t["order_line"]
    n = len(ol["ol_o_id"])
    d = ol["ol_delivery_d"].copy()
    lag = rng.integers(-20 * chgen.DAY_US, 40 * chgen.DAY_US, size=n)
    ent = dict(zip(zip(o["o_w_id"].tolist(), o["o_d_id"].tolist(), o["o_id"].tolist()), o["o_entry_d"].tolist()))
    e_of = np.array([ent.get(k, chgen.TS_2025) for k in zip(ol["ol_w_id"].tolist(), ol["ol_d_id"].tolist(),
                                                           ol["ol_o_id"].tolist())], np.int64)
    d = np.where(rng.random(n) < 0.8, e_of + lag, chgen.NULL_TS)
    eq = rng.random(n) < 0.05
    d[eq] = e_of[eq]  # delivery == entry (the <= / >= edges of Q12 / Q4)
    ol["ol_delivery_d"] = d.astype(np.int64)
    iid = ol["ol_i_id"].copy()
    iid[rng.random(n) < 0.03] = len(data) + 1000  # no such item
    ol["ol_i_id"] = iid.astype(np.int32)
    return t


def test_golden_fixture():
    t, p, want = golden_next2()
    r14 = oracle.q14(t, *p["q14"])
    w = want["q14"]
    assert (r14["sum_promo"], r14["sum_amount"], r14["count"]) == (w["sum_promo"], w["sum_amount"], w["count"])
    assert r14["promo_revenue"] == w["promo_num"] / w["promo_den"]
    r12 = oracle.q12(t, *p["q12"])
    assert [list(x) for x in zip(*[r12[k].tolist() for k in ("o_ol_cnt", "high_line_count", "low_line_count")])] == want["q12"]
    r4 = oracle.q4(t, *p["q4"])
    assert [list(x) for x in zip(r4["o_ol_cnt"].tolist(), r4["order_count"].tolist())] == want["q4"]


def test_golden_fixture_vs_sqlite_and_brute_force():
    """The hand-derived Q4 / Q12 groups of the fixture (incl. orders entered exactly at Q4's
    window bounds) are also what SQLite's CH SQL and the nested loops give."""
    t, p, want = golden_next2()
    db = sqlite_load(t)
    assert [list(r) for r in sqlite_q4(db, *p["q4"])] == want["q4"]
    assert [list(r) for r in brute_q4(t, *p["q4"])] == want["q4"]
    assert [list(r) for r in sqlite_q12(db, *p["q12"])] == want["q12"]
    assert [list(r) for r in brute_q12(t, *p["q12"])] == want["q12"]


def test_q14_prefix_longer_than_the_column():
    """LIKE 'p%' with p longer than the fixed-width i_data value matches nothing (the value is too
    short to start with p): a 50-byte i_data followed in memory by a row starting with the
    pattern's 51st character must not match."""
    t, p, _ = golden_next2()
    d50 = b"PR" + b"x" * 48
    t["item"] = {"i_id": np.array([1, 2, 3], np.int32),
                 "i_data": np.array([d50, b"Yzz", b"XPR"], dtype="S50")}
    r = oracle.q14(t, *p["q14"][:2], prefix=d50 + b"Y")
    assert r["sum_promo"] == 0 and r["count"] > 0
    r = oracle.q14(t, *p["q14"][:2], prefix=d50)  # the whole value as the prefix: a match
    assert r["sum_promo"] > 0
    db = sqlite_load(t)
    assert sqlite_q14(db, *p["q14"][:2], prefix=(d50 + b"Y").decode())[1] == 0


@pytest.mark.parametrize("seed", [1, 2, 3])
def test_brute_force_tiny(seed):
    t = mutate(chgen.generate(1, 3, seed=seed, scale=chgen.TINY), seed)
    for lo, hi, pre in ((Q14_LO, Q14_HI, b"PR"), (chgen.TS_1995, chgen.TS_2025 + 99 * chgen.DAY_US, b"PR"),
                        (chgen.TS_1995, chgen.TS_2025, b"X"), (Q14_HI, Q14_LO, b"PR")):
        r = oracle.q14(t, lo, hi, pre)
        sp, sa, cnt = brute_q14(t, lo, hi, pre)
        assert (r["sum_promo"], r["sum_amount"], r["count"]) == (sp, sa, cnt)
        assert (r["promo_revenue"] is None) == (cnt == 0)
        if cnt:
            assert r["promo_revenue"] == (100.0 * sp) / (100.0 + sa)
    for hi in (Q12_HI, chgen.TS_2025 + 99 * chgen.DAY_US, chgen.TS_1995):
        r = oracle.q12(t, hi)
        assert list(zip(*[r[k].tolist() for k in ("o_ol_cnt", "high_line_count", "low_line_count")])) == brute_q12(t, hi)
    for lo, hi in ((Q4_LO, Q4_HI), (chgen.TS_1995, chgen.TS_2025), (Q4_HI, Q4_LO)):
        r = oracle.q4(t, lo, hi)
        assert list(zip(r["o_ol_cnt"].tolist(), r["order_count"].tolist())) == brute_q4(t, lo, hi)


@pytest.mark.parametrize("mutated", [False, True])
def test_sqlite_literal_sql(mutated):
    t = chgen.generate(1, 2, seed=7)
    if mutated:
        t = mutate(t, 7)
    db = sqlite_load(t)
    for lo, hi, pre in ((Q14_LO, Q14_HI, "PR"), (chgen.TS_1995, chgen.TS_2025, "PR"), (Q14_LO, Q14_HI, "pr")):
        r = oracle.q14(t, lo, hi, pre.encode())
        promo, sp, sa, cnt = sqlite_q14(db, lo, hi, pre)
        assert (r["sum_promo"], r["sum_amount"], r["count"]) == ((sp or 0), (sa or 0), cnt)
        if cnt:
            assert math.isclose(r["promo_revenue"], promo, rel_tol=1e-9)
        else:
            assert r["promo_revenue"] is None and promo is None
    r = oracle.q12(t, Q12_HI)
    assert list(zip(*[r[k].tolist() for k in ("o_ol_cnt", "high_line_count", "low_line_count")])) == \
        [tuple(x) for x in sqlite_q12(db, Q12_HI)]
    for lo, hi in ((Q4_LO, Q4_HI), (chgen.TS_1995, chgen.TS_2025)):
        r = oracle.q4(t, lo, hi)
        assert list(zip(r["o_ol_cnt"].tolist(), r["order_count"].tolist())) == [tuple(x) for x in sqlite_q4(db, lo, hi)]


def test_strict_closed_forms():
    """TPC-C population: delivered orders (o_id < 2101) have carrier 1..10 and every line
    delivered at o_entry_d = LOAD_TS with amount 0; undelivered ones have NULL carrier and
    NULL delivery dates."""
    W = 2
    t = chgen.generate(1, W + 1, seed=4, mode="strict")
    o, ol = t["orders"], t["order_line"]
    delivered = o["o_id"] < chgen.FULL.delivered_below
    # Q12: every line of a delivered order qualifies (entry == delivery < 2020): per o_ol_cnt k,
    # high + low = k x (#delivered orders with ol_cnt k); high counts carriers 1 and 2
    r = oracle.q12(t, Q12_HI)
    for k, hi_, lo_ in zip(r["o_ol_cnt"].tolist(), r["high_line_count"].tolist(), r["low_line_count"].tolist()):
        sel = delivered & (o["o_ol_cnt"] == k)
        assert hi_ + lo_ == k * int(sel.sum())
        assert hi_ == k * int((sel & np.isin(o["o_carrier_id"], [1, 2])).sum())
    # Q4 around LOAD_TS: every delivered order exists-qualifies, undelivered never
    r = oracle.q4(t, chgen.LOAD_TS, chgen.LOAD_TS + 1)
    for k, c in zip(r["o_ol_cnt"].tolist(), r["order_count"].tolist()):
        assert c == int((delivered & (o["o_ol_cnt"] == k)).sum())
    assert oracle.q4(t, Q4_LO, Q4_HI)["o_ol_cnt"].size == 0  # LOAD_TS = 2015 is outside
    # Q14: all delivered lines qualify with amount 0 -> promo_revenue 0.0
    r = oracle.q14(t, Q14_LO, Q14_HI)
    assert r["count"] == int((ol["ol_delivery_d"] != chgen.NULL_TS).sum()) and r["promo_revenue"] == 0.0


def test_q14_all_promo_closed_form():
    """If every item matches the prefix, promo_revenue = 100*S/(100+S) with S the window sum."""
    t = chgen.generate(1, 2, seed=8)
    t["item"] = dict(t["item"])
    t["item"]["i_data"] = np.array([b"PR" + bytes(x)[2:] for x in t["item"]["i_data"]], dtype="S50")
    ol = t["order_line"]
    d = ol["ol_delivery_d"]
    m = (d != chgen.NULL_TS) & (d >= Q14_LO) & (d < Q14_HI)
    S = int(ol["ol_amount"][m].sum())
    r = oracle.q14(t, Q14_LO, Q14_HI)
    assert r["sum_promo"] == r["sum_amount"] == S and r["promo_revenue"] == 100.0 * S / (100.0 + S)
