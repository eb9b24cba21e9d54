"""Pins of the CH Q3 oracle function (NEXT-2), none of which use the oracle's own
code: the hand-derived fixture (tests/golden/ch_q3.json), brute force over the cartesian product
on tiny tables, SQLite running the literal CH SQL (case-sensitive LIKE), strict-mode invariants."""
import numpy as np
import pytest

import chgen
import oracle
from chref import brute_q3, golden_q3, iso_us, sqlite_load, sqlite_q3

Q3_LO = iso_us("2007-01-02T00:00:00")


def rows_of(r):
    return list(zip(*[r[k].tolist() for k in ("ol_o_id", "ol_w_id", "ol_d_id", "revenue", "o_entry_d")]))


def mutate(t, seed):
    """Edge cases for Q3: 'A'-states made common, look-alikes ('a', 'BA'), duplicated and orphan
    new_order rows, entry dates at the cutoff, equal revenues."""
    rng = np.random.default_rng(seed)
    t = {k: dict(v) for k, v in t.items()}
    c = t["customer"]
    st = np.array(c["c_state"], dtype="S2")
    r = rng.random(len(st))
    st[r < 0.3] = b"AK"
    st[(r >= 0.3) & (r < 0.35)] = b"ak"
    st[(r >= 0.35) & (r < 0.4)] = b"BA"
    c["c_state"] = st
    c["c_state_p2"] = chgen.prefix2(st)
    no = t["new_order"]
    k = len(no["no_o_id"])
    dup = rng.random(k) < 0.1
    t["new_order"] = {n: np.concatenate([v, v[dup], np.array([99], np.int32)]) for n, v in no.items()}
    o = t["orders"]
    e = o["o_entry_d"].copy()
    e[rng.random(len(e)) < 0.1] = Q3_LO
    o["o_entry_d"] = e
    ol = t["order_line"]
    a = ol["ol_amount"].copy()
    a[rng.random(len(a)) < 0.5] = 100  # many equal revenues
    ol["ol_amount"] = a
    return t


def test_golden_fixture():
    t, (lo, pre), want = golden_q3()
    assert rows_of(oracle.q3(t, lo, pre)) == want


@pytest.mark.parametrize("seed", [1, 2])
def test_brute_force_tiny(seed):
    t = mutate(chgen.generate(1, 2, seed=seed, scale=chgen.TINY), seed)
    for lo, pre in ((Q3_LO, b"A"), (chgen.TS_1995, b"A"), (Q3_LO, b"AK"), (Q3_LO, b"a"), (chgen.TS_2025, b"A")):
        assert rows_of(oracle.q3(t, lo, pre)) == brute_q3(t, lo, pre)


@pytest.mark.parametrize("mutated", [False, True])
def test_sqlite_literal_sql(mutated):
    t = chgen.generate(1, 2, seed=5)
    if mutated:
        t = mutate(t, 5)
    db = sqlite_load(t)
    for lo, pre in ((Q3_LO, "A"), (chgen.TS_1995, "B"), (Q3_LO, "a")):
        got = rows_of(oracle.q3(t, lo, pre.encode()))
        want = [tuple(x) for x in sqlite_q3(db, lo, pre)]
        # SQLite fixes revenue DESC, o_entry_d only: compare that order, then the full rows
        assert [(r[3], r[4]) for r in got] == [(r[3], r[4]) for r in want]
        assert sorted(got) == sorted(want)


def test_strict_invariants():
    """TPC-C population: new_order = orders 2101..3000 of every district, entry = LOAD_TS (after
    the cutoff), so every result row is a new order of an 'A%' customer, its revenue is the sum
    of all its lines, and the row count is the number of such orders."""
    t = chgen.generate(1, 3, seed=6, mode="strict")
    r = oracle.q3(t, Q3_LO)
    o, c, ol = t["orders"], t["customer"], t["order_line"]
    cust_a = {(w, d, i) for w, d, i, s in zip(c["c_w_id"].tolist(), c["c_d_id"].tolist(), c["c_id"].tolist(),
                                              [bytes(x) for x in c["c_state"]]) if s[:1] == b"A"}
    sel = [(w, d, i) for w, d, i, cc in zip(o["o_w_id"].tolist(), o["o_d_id"].tolist(), o["o_id"].tolist(),
                                            o["o_c_id"].tolist())
           if i >= chgen.FULL.delivered_below and (w, d, cc) in cust_a]
    assert len(r["ol_o_id"]) == len(sel) > 0
    assert set(zip(r["ol_w_id"].tolist(), r["ol_d_id"].tolist(), r["ol_o_id"].tolist())) == set(sel)
    assert np.all(r["o_entry_d"] == chgen.LOAD_TS)
    key = ol["ol_w_id"].astype(np.int64) << 40 | ol["ol_d_id"].astype(np.int64) << 32 | ol["ol_o_id"]
    want = {}
    for k, a in zip(key.tolist(), ol["ol_amount"].tolist()):
        want[k] = want.get(k, 0) + a
    for w, d, i, rev in zip(r["ol_w_id"].tolist(), r["ol_d_id"].tolist(), r["ol_o_id"].tolist(), r["revenue"].tolist()):
        assert rev == want[w << 40 | d << 32 | i]
    assert np.all(np.diff(r["revenue"]) <= 0)
