"""GPU parity: the CUDA path, called through the C ABI, against the CPU oracle on the same
seeded inputs (``-m gpu``; needs a B200).

Bars (BASELINE.json north_star): sums, counts, keys and row sets bit-exact; AVG within relative
1e-9 (we in fact require bit-equality, both sides compute (double)sum/(double)count the same way,
and fall back to 1e-9 only in the assertion helper); Q18 rows in the exact ORDER BY order
(the tie-break makes the order total, R11).
"""
import math

import numpy as np
import pytest

import chgen
import oracle
from chref import (Q1_CUTOFF, Q6_D_HI, Q6_D_LO, Q6_Q_HI, Q6_Q_LO, Q18_HAVING, golden, iso_us,
                   ts_param)

pytestmark = pytest.mark.gpu
HASH = 4  # H2TAP_QUERY_HASH_JOIN

Q18_NAMES = ["c_last", "c_id", "o_id", "o_entry_d", "o_ol_cnt", "amount_sum", "o_w_id", "o_d_id"]
Q1_NAMES = ["ol_number", "sum_qty", "sum_amount", "avg_qty", "avg_amount", "count_order"]


@pytest.fixture(scope="module")
def h():
    import paper_conf_cidr_appuswamykpa17_b200 as mod
    return mod


@pytest.fixture(scope="module")
def eng(h):
    e = h.h2tap_open(0)
    yield e
    h.h2tap_close(e)


class Loader:
    """Loads a whole table set as one new epoch (full reload) and runs queries."""

    def __init__(self, h, e):
        self.h, self.e, self.epoch = h, e, 0

    def load(self, tables, flags=0):
        self.epoch += 1
        self.h.h2tap_load_snapshot(self.e, self.h.hot_path_tables(tables), self.epoch, flags=flags)

    def q(self, plan, params=None, flags=0):
        r = self.h.h2tap_run_query(self.e, plan, params, flags=flags)
        try:
            out = r.to_numpy()
            out["_nulls"] = dict(r.nulls)
            out["_meta"] = (r.epoch, r.nrows, r.rows_scanned)
        finally:
            r.free()
        return out


@pytest.fixture(scope="module")
def L(h, eng):
    return Loader(h, eng)


@pytest.fixture(params=["carry", "rowid", "scatter"])
def order_mode(request, monkeypatch):
    """The ORDER BY's two record layouts: 128-bit carry records (default when
    the row fits) and (64-bit prefix, row id) pairs with tie-fix / exact fallback."""
    if request.param == "rowid":
        monkeypatch.setenv("H2TAP_ORDER_CARRY", "0")
    else:
        monkeypatch.delenv("H2TAP_ORDER_CARRY", raising=False)
    if request.param == "scatter":  # carry records through the staged HAVING output + scatter pass
        monkeypatch.setenv("H2TAP_ORDER_DIRECT", "0")
    else:
        monkeypatch.delenv("H2TAP_ORDER_DIRECT", raising=False)
    return request.param


def assert_q6(got, want):
    assert got["count_rows"][0] == want["count"]
    if want["revenue"] is None:
        assert got["_nulls"]["revenue"][0] == 1
    else:
        assert got["_nulls"]["revenue"][0] == 0
        assert got["revenue"][0] == want["revenue"]


def assert_q1(got, want):
    for k in ("ol_number", "sum_qty", "sum_amount", "count_order"):
        assert np.array_equal(got[k], want[k]), k
    for k in ("avg_qty", "avg_amount"):
        assert len(got[k]) == len(want[k])
        for a, b in zip(got[k].tolist(), want[k].tolist()):
            assert math.isclose(a, b, rel_tol=1e-9, abs_tol=0.0), (k, a, b)


def assert_q18(got, want):
    for k in Q18_NAMES:
        assert np.array_equal(got[k], want[k]), k


def run_all(L, t, rng=None, n_rand=2):
    L.load(t)
    assert_q6(L.q(6, [Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI]), oracle.q6(t, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI))
    assert_q6(L.q(6), oracle.q6(t, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI))  # CH defaults in the library
    assert_q1(L.q(1, [Q1_CUTOFF]), oracle.q1(t, Q1_CUTOFF))
    assert_q1(L.q(1), oracle.q1(t, Q1_CUTOFF))
    want18 = oracle.q18(t, Q18_HAVING)
    assert_q18(L.q(18, [Q18_HAVING]), want18)
    assert_q18(L.q(18), want18)
    assert_q18(L.q(18, flags=HASH), want18)  # open-addressing join indexes forced
    rng = rng or np.random.default_rng(0)
    for _ in range(n_rand):
        d_lo = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
        d_hi = int(rng.integers(d_lo, chgen.TS_2025 + 31 * chgen.DAY_US))
        q_lo, q_hi = int(rng.integers(0, 6)), int(rng.integers(4, 12))
        assert_q6(L.q(6, [d_lo, d_hi, q_lo, q_hi]), oracle.q6(t, d_lo, d_hi, q_lo, q_hi))
        cut = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
        assert_q1(L.q(1, [cut]), oracle.q1(t, cut))
        thr = int(rng.integers(-10, 8_000_000))
        want18 = oracle.q18(t, thr)
        assert_q18(L.q(18, [thr]), want18)
        assert_q18(L.q(18, [thr], flags=HASH), want18)


# ----------------------------------------------------------------- cases --
def test_golden_fixture(L):
    t, exp = golden()
    L.load(t)
    for case in exp["q6"]:
        d_lo, d_hi, q_lo, q_hi = case["params"]
        got = L.q(6, [iso_us(d_lo), iso_us(d_hi), q_lo, q_hi])
        assert_q6(got, {"revenue": case["revenue"], "count": case["count"]})
    for case in exp["q1"]:
        got = L.q(1, [iso_us(case["params"][0])])
        assert got["ol_number"].tolist() == [r["ol_number"] for r in case["rows"]]
        assert got["sum_amount"].tolist() == [r["sum_amount"] for r in case["rows"]]
        assert got["avg_amount"].tolist() == [r["avg_amount"] for r in case["rows"]]
    for case in exp["q18"]:
        got = L.q(18, case["params"])
        assert got["amount_sum"].tolist() == [r["amount_sum"] for r in case["rows"]]
        assert got["o_entry_d"].tolist() == [iso_us(r["o_entry_d"]) for r in case["rows"]]
        assert got["c_last"].tolist() == [r["c_last"] for r in case["rows"]]


def test_boundaries_fixture(L, order_mode):
    """tests/golden/boundaries_ch.json: rows exactly on every predicate bound (Q6 d_lo/d_hi, BETWEEN
    ends, Q1 cutoff, NULL vs INT64_MIN constants) and a Q18 group summing to exactly the HAVING
    threshold; hand-derived expectations (also pinned by SQLite and brute force on the CPU)."""
    t, exp = golden("boundaries_ch.json")
    L.load(t)
    for case in exp["q6"]:
        p = [ts_param(v) for v in case["params"]]
        assert_q6(L.q(6, p), {"revenue": case["revenue"], "count": case["count"]})
    for case in exp["q1"]:
        got = L.q(1, [ts_param(case["params"][0])])
        rows = case["rows"]
        for k in ("ol_number", "sum_qty", "sum_amount", "count_order"):
            assert got[k].tolist() == [r[k] for r in rows], (case["_why"], k)
        for k in ("avg_qty", "avg_amount"):
            for a, b in zip(got[k].tolist(), [r[k] for r in rows]):
                assert math.isclose(a, b, rel_tol=1e-9, abs_tol=0.0), (case["_why"], k)
    for case in exp["q18"]:
        for flags in (0, HASH):
            got = L.q(18, case["params"], flags=flags)
            want = [(r["c_last"], r["c_id"], r["o_id"], iso_us(r["o_entry_d"]), r["o_ol_cnt"],
                     r["amount_sum"], r["o_w_id"], r["o_d_id"]) for r in case["rows"]]
            assert list(zip(*[got[k].tolist() for k in Q18_NAMES])) == want, case["_why"]


def test_q18_tiebreak_fixture(L, order_mode):
    """tests/golden/tiebreak_q18.json: four groups tied on (amount_sum, o_entry_d) in different
    warehouses and districts, ordered by o_w_id, o_d_id, o_id (R33); hand-derived."""
    t, exp = golden("tiebreak_q18.json")
    L.load(t)
    for case in exp["q18"]:
        for flags in (0, HASH):
            got = L.q(18, case["params"], flags=flags)
            want = [(r["c_last"], r["c_id"], r["o_id"], iso_us(r["o_entry_d"]), r["o_ol_cnt"],
                     r["amount_sum"], r["o_w_id"], r["o_d_id"]) for r in case["rows"]]
            assert list(zip(*[got[k].tolist() for k in Q18_NAMES])) == want, case["_why"]


def test_q18_having_exactly_at_group_sums(L, order_mode):
    """HAVING thresholds equal to existing group sums (the '>' boundary) at W=2: the group at the
    threshold is excluded, the one 1 cent above it included, on both join-index layouts."""
    t = chgen.generate(1, 3, seed=21)
    L.load(t)
    sums = oracle.q18(t, -1)["amount_sum"]
    picks = sorted({int(sums[0]), int(sums[len(sums) // 2]), int(sums[-1]), Q18_HAVING})
    for thr in picks + [picks[1] - 1, picks[1] + 1]:
        want = oracle.q18(t, thr)
        assert thr not in want["amount_sum"].tolist()
        assert_q18(L.q(18, [thr]), want)
        assert_q18(L.q(18, [thr], flags=HASH), want)


@pytest.mark.parametrize("W,mode,seed", [(1, "spread", 1), (3, "spread", 2), (2, "strict", 3)])
def test_parity_small(L, W, mode, seed, order_mode):
    run_all(L, chgen.generate(1, W + 1, seed=seed, mode=mode), np.random.default_rng(seed))


@pytest.mark.parametrize("n", [0, 1, 2, 3, 4, 5, 7, 127, 128, 129, 4097, 100_003])
def test_ragged_order_line(L, n):
    """Row counts that leave a ragged tail after 4-row vectors / 32-row warps / tiles."""
    t = chgen.generate(1, 2, seed=5)
    t["order_line"] = {k: v[:n].copy() for k, v in t["order_line"].items()}
    run_all(L, t, n_rand=1)


def test_empty_tables(L):
    t = chgen.generate(1, 1, seed=1)  # zero warehouses: every table empty
    L.load(t)
    got = L.q(6)
    assert got["_nulls"]["revenue"][0] == 1 and got["count_rows"][0] == 0
    assert len(L.q(1)["ol_number"]) == 0
    assert len(L.q(18, [-100])["o_id"]) == 0


def test_q1_sparse_group_keys(L):
    """Keys outside the dense range [0,16): warp-aggregated shared/global hash path."""
    t = chgen.generate(1, 3, seed=8)
    ol = t["order_line"]
    rng = np.random.default_rng(8)
    n = len(ol["ol_number"])
    keys = ol["ol_number"].copy()
    pick = rng.random(n) < 0.5
    keys[pick] = rng.integers(-3000, 3000, size=int(pick.sum()), dtype=np.int32)
    keys[:1000] = 2**31 - 1            # long runs of one sparse key
    keys[1000:1500] = -(2**31)
    ol["ol_number"] = keys
    L.load(t)
    for cut in (Q1_CUTOFF, chgen.TS_1995):
        assert_q1(L.q(1, [cut]), oracle.q1(t, cut))


@pytest.mark.parametrize("shared", ["1", "0"])
def test_shared_q6_q1_scan(h, monkeypatch, shared):
    """A batch with one Q6 before one Q1 runs one shared scan: random Q6 windows
    and quantity ranges (incl. empty and inverted ones, bounds at INT64_MIN), random Q1 cutoffs,
    ragged sizes and NULL dates, vs the oracle; H2TAP_SHARED_SCAN=0 runs the two scans."""
    monkeypatch.setenv("H2TAP_SHARED_SCAN", shared)
    e = h.h2tap_open(0)
    try:
        L = Loader(h, e)
        rng = np.random.default_rng(57)
        for n_keep in (100_003, 2049, 1023, 1):
            t = chgen.generate(1, 3, seed=57)
            t["order_line"] = {k: v[:n_keep].copy() for k, v in t["order_line"].items()}
            L.load(t)
            cases = [(Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI, Q1_CUTOFF),
                     (-(2**63), 2**63 - 1, -(2**63), 2**63 - 1, -(2**63)),  # everything non-NULL
                     (chgen.TS_2025, chgen.TS_1995, 1, 10, chgen.TS_2025),   # inverted / empty
                     (chgen.TS_1995, chgen.TS_2025, 7, 3, chgen.TS_1995)]   # empty quantity range
            for _ in range(3):
                d_lo = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
                cases.append((d_lo, int(rng.integers(d_lo, chgen.TS_2025 + 10**12)), int(rng.integers(0, 6)),
                              int(rng.integers(4, 12)), int(rng.integers(chgen.TS_1995, chgen.TS_2025))))
            for d_lo, d_hi, q_lo, q_hi, cut in cases:
                rs = h.h2tap_run_queries(e, [(6, [d_lo, d_hi, q_lo, q_hi], 0), (1, [cut], 0)])
                g6, g1 = rs[0].to_numpy(), rs[1].to_numpy()
                g6["_nulls"] = dict(rs[0].nulls)
                for r in rs:
                    h.h2tap_free(r)
                assert_q6(g6, oracle.q6(t, d_lo, d_hi, q_lo, q_hi))
                assert_q1(g1, oracle.q1(t, cut))
    finally:
        h.h2tap_close(e)


def test_q6_quantity_and_null_edges(L):
    t = chgen.generate(1, 2, seed=4)
    L.load(t)
    i64 = np.iinfo(np.int64)
    for p in ([i64.min, i64.max, i64.min, i64.max],      # NULL dates must still be excluded
              [i64.min + 1, i64.max, 0, 0],              # no quantity 0 -> NULL revenue
              [Q6_D_LO, Q6_D_LO, 1, 10],                 # empty date window
              [Q6_D_LO, Q6_D_HI, 10, 1]):                # inverted BETWEEN
        assert_q6(L.q(6, p), oracle.q6(t, *p))


def test_q18_join_edges(L, order_mode):
    """Orphan lines, orders without lines, customers missing, negative HAVING."""
    t = chgen.generate(1, 2, seed=6)
    ol, o, c = t["order_line"], t["orders"], t["customer"]
    ol["ol_o_id"][:50] = 7777                      # orphan lines
    keep = np.ones(len(c["c_id"]), bool)
    keep[::7] = False                              # drop every 7th customer
    t["customer"] = {k: v[keep].copy() for k, v in c.items()}
    mask = o["o_id"] % 11 != 0                     # orders without some rows
    t["orders"] = {k: v[mask].copy() for k, v in o.items()}
    L.load(t)
    for thr in (-1, 0, Q18_HAVING, 4_000_000):
        want = oracle.q18(t, thr)
        assert_q18(L.q(18, [thr]), want)
        assert_q18(L.q(18, [thr], flags=HASH), want)


def test_q18_ties_use_full_order(L, order_mode):
    """Equal amount_sum and o_entry_d: the (w, d, o) tie-break decides (R11)."""
    t = chgen.generate(1, 3, seed=9)
    t["order_line"]["ol_amount"][:] = 1000
    t["orders"]["o_entry_d"][:] = chgen.LOAD_TS
    L.load(t)
    for thr in (0, 6000):
        assert_q18(L.q(18, [thr]), oracle.q18(t, thr))


def test_q18_sort_fallback_long_prefix_runs(L, order_mode):
    """Composite key > 64 bits and > 32 rows sharing the 48-bit prefix: exact field-by-field
    re-sort path."""
    for variant in ("short_runs", "long_runs"):
        t = chgen.generate(1, 3, seed=17)
        t["order_line"]["ol_amount"][:] = 1000            # amount_sum in {5000, ..., 15000}
        o = t["orders"]
        half = np.arange(len(o["o_id"])) % 2 == 0
        if variant == "short_runs":                      # tie-fix path (runs of ~3 rows)
            o["o_entry_d"][half] = chgen.TS_2025 - 10**6 + (np.arange(int(half.sum())) % 1000)
        else:                                            # exact field-by-field fallback
            o["o_entry_d"][half] = chgen.TS_2025 - 10**6
        L.load(t)
        for thr in (0, 9000):
            want = oracle.q18(t, thr)
            assert_q18(L.q(18, [thr]), want)
            assert_q18(L.q(18, [thr], flags=HASH), want)


def test_q18_wide_payload_disables_carry(L):
    """c_last codes spanning 32 bits (and a 96-bit key): the carry record cannot hold the row,
    the plan falls back to row-id pairs on its own (no env knob)."""
    t = chgen.generate(1, 3, seed=23)
    rng = np.random.default_rng(23)
    c = t["customer"]
    c["c_last"][:] = rng.integers(-2**31, 2**31 - 1, len(c["c_last"]), dtype=np.int64).astype(np.int32)
    L.load(t)
    for thr in (0, Q18_HAVING):
        want = oracle.q18(t, thr)
        assert_q18(L.q(18, [thr]), want)
        assert_q18(L.q(18, [thr], flags=HASH), want)


def test_q18_carry_field_extremes(L):
    """Carry decode with full 128-bit records: 44-bit amount_sum field, o_entry_d far below 1970
    (negative µs), a 17-bit o_ol_cnt payload field; a negative o_ol_cnt (32-bit field) no
    longer fits and the plan falls back to row ids."""
    t = chgen.generate(1, 2, seed=29)
    o, c = t["orders"], t["customer"]
    o["o_entry_d"][:] = -(10**15) + np.arange(len(o["o_id"]), dtype=np.int64) * 7919
    o["o_ol_cnt"][::3] = 1 << 16                  # 17-bit o_ol_cnt field, record still fits
    t["order_line"]["ol_amount"][::5] = 10**12
    L.load(t)
    for thr in (-10**13, 0, 10**12):
        want = oracle.q18(t, thr)
        assert_q18(L.q(18, [thr]), want)
    o["o_ol_cnt"][::7] = -5
    L.load(t)
    for thr in (0, 10**12):
        assert_q18(L.q(18, [thr]), oracle.q18(t, thr))


def test_q18_planner_dense_and_hash(h, eng, L):
    """TPC-C keys are dense -> perfect-hash indexes; sparse keys -> open addressing."""
    t = chgen.generate(1, 3, seed=19)
    L.load(t)
    r = h.h2tap_run_query(eng, h.H2TAP_Q18)
    assert r.plan_flags & 3 == 3
    assert r.plan_flags >> 3 == 3  # generated tables are in key order: positional indexes (§4.3)
    r.free()
    r = h.h2tap_run_query(eng, h.H2TAP_Q18, flags=HASH)
    assert r.plan_flags == 0
    r.free()
    for tab, col in (("orders", "o_id"), ("order_line", "ol_o_id")):
        t[tab][col] = t[tab][col] * 1000 + 7         # same join, sparse key box
    t["customer"]["c_id"] = t["customer"]["c_id"] * 977
    t["orders"]["o_c_id"] = t["orders"]["o_c_id"] * 977
    L.load(t)
    r = h.h2tap_run_query(eng, h.H2TAP_Q18)
    got = r.to_numpy()
    assert r.plan_flags == 0
    r.free()
    assert_q18(got, oracle.q18(t, Q18_HAVING))


def test_q18_duplicate_key_rejected(h, L):
    t = chgen.generate(1, 2, seed=2)
    o = t["orders"]
    for k in o:
        o[k] = np.concatenate([o[k], o[k][:1]])
    L.load(t)
    with pytest.raises(h.H2tapError) as ei:
        L.q(18)
    assert ei.value.status == h.H2TAP_EDUPKEY
    with pytest.raises(h.H2tapError) as ei:
        L.q(18, flags=HASH)
    assert ei.value.status == h.H2TAP_EDUPKEY
    assert_q6(L.q(6), oracle.q6(t, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI))  # engine still usable


def test_device_resident_results(h, L):
    t = chgen.generate(1, 3, seed=12)
    L.load(t)
    assert_q18(L.q(18, flags=h.H2TAP_RESULT_DEVICE), oracle.q18(t, Q18_HAVING))
    assert_q1(L.q(1, flags=h.H2TAP_RESULT_DEVICE | h.H2TAP_QUERY_PROFILE), oracle.q1(t, Q1_CUTOFF))


def test_last_batch_device_ms(h):
    """h2tap_last_batch_ms: EPLAN before any batch; after a batch, the GPU span of its kernels —
    positive, at least the longest query's own device time, at most the call's wall clock."""
    e = h.h2tap_open(0)
    try:
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_last_batch_ms(e)
        assert ei.value.status == h.H2TAP_EPLAN
        t = chgen.generate(1, 3, seed=4)
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
        rs = h.h2tap_run_queries(e, [(h.H2TAP_Q6, None, 0), (h.H2TAP_Q1, None, 0), (h.H2TAP_Q18, None, 0)])
        ms = h.h2tap_last_batch_ms(e)
        assert 0 < ms <= max(r.e2e_ms for r in rs) + 1e-3
        assert ms >= max(r.device_ms for r in rs) - 1e-3
        for r in rs:
            h.h2tap_free(r)
    finally:
        h.h2tap_close(e)


def test_profile_reports_kernels(h, eng, L):
    t = chgen.generate(1, 2, seed=3)
    L.load(t)
    r = h.h2tap_run_query(eng, h.H2TAP_Q18, flags=h.H2TAP_QUERY_PROFILE)
    names = [k for k, _ in r.kernels]
    # v3 ORDER BY: bucket counts from the accumulators, the column scan, then the
    # HAVING pass writes each carry record at its final bucket position (no scatter pass)
    # (the plan and the counts in one grid-barrier kernel when the engine is alone on the device)
    assert {"q18_build", "q18_probe_groupjoin", "q18_sort_scan", "q18_having_records",
            "q18_bucket_sort_emit"} <= set(names)
    assert {"q18_plan_count"} <= set(names) or {"q18_acc_stats", "q18_bucket_count"} <= set(names), names
    assert "q18_bucket_scatter" not in names
    assert all(ms >= 0 for _, ms in r.kernels) and r.device_ms > 0
    r.free()


def test_batch_queries_one_epoch(h, eng, L):
    """h2tap_run_queries: several plans (repeats included) enqueued back to back, one sync."""
    t = chgen.generate(1, 3, seed=27)
    L.load(t)
    batch = [(6, None, 0), (1, None, h.H2TAP_RESULT_DEVICE), (18, [Q18_HAVING], 0),
             (18, [5_000_000], h.H2TAP_RESULT_DEVICE | HASH), (6, [Q6_D_LO, Q6_D_HI, 3, 7], 0),
             (1, [chgen.TS_1995], h.H2TAP_QUERY_PROFILE)]
    rs = h.h2tap_run_queries(eng, batch)
    try:
        got = []
        for r in rs:
            x = r.to_numpy()
            x["_nulls"] = dict(r.nulls)
            got.append(x)
        assert len({r.epoch for r in rs}) == 1
    finally:
        for r in rs:
            r.free()
    assert_q6(got[0], oracle.q6(t, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI))
    assert_q1(got[1], oracle.q1(t, Q1_CUTOFF))
    assert_q18(got[2], oracle.q18(t, Q18_HAVING))
    assert_q18(got[3], oracle.q18(t, 5_000_000))
    assert_q6(got[4], oracle.q6(t, Q6_D_LO, Q6_D_HI, 3, 7))
    assert_q1(got[5], oracle.q1(t, chgen.TS_1995))
    with pytest.raises(h.H2tapError):
        h.h2tap_run_queries(eng, [(6, None, 0), (99, None, 0)])


# ------------------------------------------------------- snapshot semantics --
def test_snapshot_epochs_append_and_errors(h):
    """a1: append-only refresh, epoch monotonicity, shape errors, async publish."""
    e = h.h2tap_open(0)
    try:
        base = chgen.generate(1, 3, seed=21)
        cols = h.hot_path_tables(base)
        h.h2tap_load_snapshot(e, cols, 10)
        r = h.h2tap_run_query(e, h.H2TAP_Q18)
        assert r.epoch == 10 and r.rows_scanned == len(base["order_line"]["ol_w_id"])
        r.free()
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_load_snapshot(e, cols, 10)
        assert ei.value.status == h.H2TAP_ESTALE
        # NewOrder delta appended at epoch 11 (host row store -> columns -> H2D delta only)
        st = chgen.NewOrderState(1, 3)
        delta = chgen.neworder_delta(st, 300, seed=21, batch=0)
        n_ol = len(base["order_line"]["ol_w_id"])
        n_o = len(base["orders"]["o_id"])
        d = h.hot_path_tables({"order_line": delta["order_line"], "orders": delta["orders"],
                               "customer": {k: v[:0] for k, v in base["customer"].items()}})
        d.pop("customer")
        with pytest.raises(h.H2tapError) as ei:  # wrong first_row
            h.h2tap_load_snapshot(e, d, 11, full_reload=False, first_row={"order_line": n_ol - 1, "orders": n_o})
        assert ei.value.status == h.H2TAP_ESHAPE
        h.h2tap_load_snapshot(e, d, 11, full_reload=False, first_row={"order_line": n_ol, "orders": n_o},
                              flags=h.H2TAP_LOAD_ASYNC)
        assert h.h2tap_sync(e) == 11
        merged = {t: {k: np.concatenate([base[t][k], delta[t][k]]) for k in base[t]}
                  for t in ("order_line", "orders")}
        merged["customer"] = base["customer"]
        r = h.h2tap_run_query(e, h.H2TAP_Q18, [-1])
        got = r.to_numpy()
        assert r.epoch == 11 and r.rows_scanned == n_ol + len(delta["order_line"]["ol_w_id"])
        r.free()
        assert_q18(got, oracle.q18(merged, -1))
        # Q6/Q1 unchanged by NewOrder rows (NULL delivery dates, R16) but see the new epoch
        r6 = h.h2tap_run_query(e, h.H2TAP_Q6)
        assert r6.to_numpy()["count_rows"][0] == oracle.q6(base, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI)["count"]
        r6.free()
        # a result from an earlier epoch stays valid after a full reload
        old = h.h2tap_run_query(e, h.H2TAP_Q1)
        h.h2tap_load_snapshot(e, h.hot_path_tables(chgen.generate(1, 2, seed=99)), 12)
        assert_q1(old.to_numpy(), oracle.q1(merged, Q1_CUTOFF))
        old.free()
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_run_query(e, h.H2TAP_Q6, [1, 2])
        assert ei.value.status == h.H2TAP_EINVAL
    finally:
        h.h2tap_close(e)


def test_async_borrowed_pinned_loads(h):
    """H2TAP_LOAD_ASYNC | H2TAP_LOAD_BORROW: the call returns before the DMA of the lent pinned
    buffers; queries run on the latest PUBLISHED epoch and every result equals the oracle of the
    epoch it reports; alternating two table sets catches a query that mixes them."""
    import torch
    sets = [chgen.generate(1, 4, seed=41), chgen.generate(1, 4, seed=42)]
    pinned = [{t: {c: torch.from_numpy(v).pin_memory() for c, v in cols.items()}
               for t, cols in h.hot_path_tables(ts).items()} for ts in sets]
    want = [(oracle.q6(ts, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI), oracle.q1(ts, Q1_CUTOFF),
             oracle.q18(ts, Q18_HAVING)) for ts in sets]
    e = h.h2tap_open(0)
    try:
        h.h2tap_load_snapshot(e, pinned[1], 1)  # epoch k holds set k % 2
        seen = set()
        for ep in range(2, 10):
            h.h2tap_load_snapshot(e, pinned[ep % 2], ep, flags=h.H2TAP_LOAD_ASYNC | h.H2TAP_LOAD_BORROW)
            rs = h.h2tap_run_queries(e, [(6, None, 0), (1, None, 0), (18, None, 0)])
            for plan, r in zip((6, 1, 18), rs):
                got, k = r.to_numpy(), r.epoch % 2
                seen.add(ep - r.epoch)
                if plan == 6:
                    assert got["revenue"][0] == want[k][0]["revenue"]
                elif plan == 1:
                    assert np.array_equal(got["sum_amount"], want[k][1]["sum_amount"])
                else:
                    assert_q18(got, want[k][2])
                h.h2tap_free(r)
        assert h.h2tap_sync(e) == 9
        assert seen <= {0, 1}
    finally:
        h.h2tap_close(e)


def test_row_store_refresh(h):
    """h2tap_load_snapshot_rows: NSM records -> DSM snapshot (full load, then an append)."""
    e = h.h2tap_open(0)
    try:
        base = chgen.generate(1, 3, seed=33)
        cols = {tb: list(c) for tb, c in h.hot_path_tables(base).items()}
        recs = {tb: chgen.to_records(tb, base[tb]) for tb in ("order_line", "orders", "customer")}
        h.h2tap_load_snapshot_rows(e, recs, 1, columns=cols)
        r = h.h2tap_run_query(e, h.H2TAP_Q18, [-1]); got = r.to_numpy(); r.free()
        assert_q18(got, oracle.q18(base, -1))
        h.h2tap_reserve(e, "order_line", len(recs["order_line"]) + 100_000)  # pre-size, then append
        h.h2tap_reserve(e, "orders", len(recs["orders"]) + 10_000)
        st = chgen.NewOrderState(1, 3)
        d = chgen.neworder_batch(st, 500, seed=33, batch=0, item=base["item"])
        drec = {tb: chgen.to_records(tb, d[tb]) for tb in ("order_line", "orders")}
        h.h2tap_load_snapshot_rows(e, drec, 2, full_reload=False, columns=cols,
                                   first_row={tb: len(recs[tb]) for tb in drec})
        merged = {tb: {c: np.concatenate([base[tb][c], d[tb][c]]) for c in base[tb]}
                  for tb in ("order_line", "orders")}
        merged["customer"] = base["customer"]
        r = h.h2tap_run_query(e, h.H2TAP_Q18, [-1]); got = r.to_numpy(); r.free()
        assert_q18(got, oracle.q18(merged, -1))
        r = h.h2tap_run_query(e, h.H2TAP_Q1); got = r.to_numpy(); r.free()
        assert_q1(got, oracle.q1(merged, Q1_CUTOFF))
    finally:
        h.h2tap_close(e)


def test_concurrent_refresh_and_queries(h):
    """Queries running while another thread appends see a consistent published epoch."""
    import threading
    e = h.h2tap_open(0)
    try:
        base = chgen.generate(1, 3, seed=31)
        h.h2tap_load_snapshot(e, h.hot_path_tables(base), 1)
        st = chgen.NewOrderState(1, 3)
        deltas = [chgen.neworder_delta(st, 50, seed=31, batch=b) for b in range(6)]
        errors = []

        def refresher():
            try:
                n_ol, n_o = len(base["order_line"]["ol_w_id"]), len(base["orders"]["o_id"])
                for b, d in enumerate(deltas):
                    dd = h.hot_path_tables({**d, "customer": base["customer"]})
                    dd.pop("customer")
                    h.h2tap_load_snapshot(e, dd, 2 + b, full_reload=False,
                                          first_row={"order_line": n_ol, "orders": n_o},
                                          flags=h.H2TAP_LOAD_ASYNC)
                    n_ol += len(d["order_line"]["ol_w_id"])
                    n_o += len(d["orders"]["o_id"])
            except Exception as x:  # pragma: no cover
                errors.append(x)

        th = threading.Thread(target=refresher)
        th.start()
        seen = []
        for _ in range(20):
            r = h.h2tap_run_query(e, h.H2TAP_Q18, [-1])
            seen.append((r.epoch, r.nrows, r.rows_scanned))
            r.free()
        th.join()
        assert not errors
        h.h2tap_sync(e)
        # each observed epoch must be exactly the base plus the first (epoch-1) deltas
        for ep, nrows, scanned in seen:
            k = ep - 1
            want_rows = len(base["orders"]["o_id"]) + sum(len(d["orders"]["o_id"]) for d in deltas[:k])
            want_scan = len(base["order_line"]["ol_w_id"]) + sum(len(d["order_line"]["ol_w_id"]) for d in deltas[:k])
            assert (nrows, scanned) == (want_rows, want_scan), (ep, nrows, scanned)
        assert [s[0] for s in seen] == sorted(s[0] for s in seen)
    finally:
        h.h2tap_close(e)


# ------------------------------------------------------ re-partition on 1 GPU --
def test_repartition_matches_whole(h):
    """Per-shard results (the per-rank partials of a multi-GPU run) merged = whole."""
    W, k = 6, 3
    whole = chgen.generate(1, W + 1, seed=41)
    rev = cnt = 0
    q1m = {}
    rows = []
    for lo, hi in chgen.warehouse_ranges(W, k):
        e = h.h2tap_open(0)
        try:
            part = chgen.generate(lo, hi, seed=41)
            h.h2tap_load_snapshot(e, h.hot_path_tables(part), 1)
            r = h.h2tap_run_query(e, h.H2TAP_Q6); x = r.to_numpy(); r.free()
            rev += int(x["revenue"][0]); cnt += int(x["count_rows"][0])
            r = h.h2tap_run_query(e, h.H2TAP_Q1); x = r.to_numpy(); r.free()
            for i, n in enumerate(x["ol_number"].tolist()):
                m = q1m.setdefault(n, [0, 0, 0])
                m[0] += int(x["sum_qty"][i]); m[1] += int(x["sum_amount"][i]); m[2] += int(x["count_order"][i])
            r = h.h2tap_run_query(e, h.H2TAP_Q18); x = r.to_numpy(); r.free()
            rows += list(zip(*[x[c].tolist() for c in Q18_NAMES]))
        finally:
            h.h2tap_close(e)
    w6 = oracle.q6(whole, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI)
    assert (rev, cnt) == (w6["revenue"], w6["count"])
    w1 = oracle.q1(whole, Q1_CUTOFF)
    for i, n in enumerate(w1["ol_number"].tolist()):
        assert q1m[n] == [int(w1["sum_qty"][i]), int(w1["sum_amount"][i]), int(w1["count_order"][i])]
    w18 = oracle.q18(whole, Q18_HAVING)
    assert sorted(rows) == sorted(zip(*[w18[c].tolist() for c in Q18_NAMES]))


# --------------------------------------------- full size, bench configuration --
@pytest.fixture(scope="module")
def w100():
    return chgen.generate(1, 101, seed=1, mode="spread")


def test_bench_line_contract():
    """bench.py at N=1 on a small snapshot prints one JSON line with every key the measurement
    contract names, consistent with itself."""
    import json as _json
    import os
    import subprocess
    import sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    env = {k: v for k, v in os.environ.items() if k not in ("RANK", "WORLD_SIZE", "LOCAL_RANK")}
    r = subprocess.run([sys.executable, os.path.join(root, "bench.py"), "--steps", "3", "--warmup", "3",
                        "--warehouses", "2", "--e2e-steps", "3", "--inc-neworders", "500",
                        "--inc-deliveries", "50"], capture_output=True, text=True, env=env, timeout=900)
    assert r.returncode == 0, r.stderr[-3000:]
    d = _json.loads([x for x in r.stdout.splitlines() if x.startswith("{")][-1])
    for k in ("metric", "value", "unit", "n_gpus", "steps", "warmup", "ms_per_step", "higher_is_better",
              "scaling", "vs_baseline", "dtype", "data", "config", "roofline", "cpu_baseline", "e2e",
              "gpu_launches", "clocks", "c1", "c2", "c3", "e2e_incremental"):
        assert k in d, k
    assert d["n_gpus"] == 1 and d["steps"] == 3 and d["warmup"] == 3 and d["higher_is_better"] is True
    assert d["value"] > 0 and d["ms_per_step"] > 0 and d["gpu_launches"] > 0
    assert math.isclose(d["value"], d["config"]["order_line_rows_total"] / (d["ms_per_step"] / 1e3), rel_tol=1e-6)
    roof = d["roofline"]
    for k in ("bound", "achieved", "peak", "unit", "frac", "traffic"):
        assert k in roof, k
    assert math.isclose(roof["frac"], roof["achieved"] / roof["peak"], rel_tol=1e-3)
    for k in ("value", "unit", "h2d_bytes_per_step", "d2h_bytes_per_step"):
        assert k in d["e2e"], k
    assert d["e2e"]["h2d_bytes_per_step"] > 0 and d["e2e"]["d2h_bytes_per_step"] > 0
    assert d["e2e"]["value"] < d["value"]  # host copies inside: not the device figure again
    cb = d["cpu_baseline"]
    assert cb["kind"] == "oracle" and cb["cores"] == 1 and cb["value"] > 0
    assert {"sm_mhz", "sm_max_mhz", "reasons"} <= set(d["clocks"])
    assert d["e2e_incremental"]["h2d_bytes_per_step"] > 0 and d["e2e_incremental"]["pipelined"]["value"] > 0


def test_full_size_w100_bench_config(h, w100):
    """BASELINE configs[1]/[2] size (W=100, 30M order_line rows), launched exactly as bench.py
    does (same engine entry points, default CH params), compared element by element."""
    e = h.h2tap_open(0)
    try:
        h.h2tap_load_snapshot(e, h.hot_path_tables(w100), 1)
        L = Loader(h, e)
        want6 = oracle.q6(w100, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI)
        want1 = oracle.q1(w100, Q1_CUTOFF)
        want = oracle.q18(w100, Q18_HAVING)
        # the bench's step: one batch, device-resident results (shared Q6+Q1 scan, PDL chain)
        rs = h.h2tap_run_queries(e, [(6, None, h.H2TAP_RESULT_DEVICE), (1, None, h.H2TAP_RESULT_DEVICE),
                                     (18, None, h.H2TAP_RESULT_DEVICE)])
        got = []
        for r in rs:
            x = r.to_numpy()
            x["_nulls"] = {k: (v.copy() if hasattr(v, "copy") else v) for k, v in r.nulls.items()}
            got.append(x)
            h.h2tap_free(r)
        assert_q6(got[0], want6)
        assert_q1(got[1], want1)
        assert_q18(got[2], want)
        assert_q6(L.q(6), want6)
        assert_q1(L.q(1), want1)
        assert_q18(L.q(18, flags=h.H2TAP_QUERY_PROFILE), want)
        assert_q18(L.q(18, flags=HASH), want)
    finally:
        h.h2tap_close(e)


def test_full_size_w100_strict(h):
    """W=100 with the strict TPC-C population: 64-bit exact composite ORDER BY path."""
    t = chgen.generate(1, 101, seed=2, mode="strict")
    e = h.h2tap_open(0)
    try:
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
        L = Loader(h, e)
        assert_q6(L.q(6), oracle.q6(t, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI))
        assert_q1(L.q(1), oracle.q1(t, Q1_CUTOFF))
        assert_q18(L.q(18), oracle.q18(t, Q18_HAVING))
    finally:
        h.h2tap_close(e)


def test_full_size_w1000_q6_q1_shared_batch(h):
    """Config C4 size on one GPU: W=1000 (~300 M order_line rows, 7.2 GB of Q1/Q6 columns),
    Q6 + Q1 as one batch (the shared scan) and separately, vs the oracle on every row."""
    cols = ["ol_number", "ol_delivery_d", "ol_quantity", "ol_amount"]
    parts = []
    for lo in range(1, 1001, 50):
        g = chgen.generate(lo, lo + 50, seed=1, with_item=False)
        parts.append({c: g["order_line"][c] for c in cols})
    ol = {c: np.concatenate([p[c] for p in parts]) for c in cols}
    del parts
    t = {"order_line": ol}
    want6 = oracle.q6(t, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI)
    want1 = oracle.q1(t, Q1_CUTOFF)
    e = h.h2tap_open(0)
    try:
        h.h2tap_load_snapshot(e, t, 1)
        rs = h.h2tap_run_queries(e, [(6, None, 0), (1, None, 0)])
        g6, g1 = rs[0].to_numpy(), rs[1].to_numpy()
        g6["_nulls"] = dict(rs[0].nulls)
        for r in rs:
            h.h2tap_free(r)
        assert_q6(g6, want6)
        assert_q1(g1, want1)
        L = Loader(h, e)
        assert_q6(L.q(6), want6)
        assert_q1(L.q(1), want1)
    finally:
        h.h2tap_close(e)


@pytest.mark.parametrize("layout", ["clustered", "one_row_swapped", "shuffled", "customer_shuffled"])
def test_q18_clustered_index_verification(L, layout, order_mode):
    """The positional (clustered) join index is used only while the device finds
    every build row at its own key slot: a generated table (in key order), one swapped pair of
    orders rows, fully shuffled orders, shuffled customers — all must equal the oracle, on the
    perfect-hash and the hash-join plans, Q18 and Q3."""
    from test_oracle_q3 import Q3_LO
    t = chgen.generate(1, 3, seed=41)
    rng = np.random.default_rng(41)
    o, c = t["orders"], t["customer"]
    if layout == "one_row_swapped":
        perm = np.arange(len(o["o_id"]))
        perm[[10, 20000]] = perm[[20000, 10]]
        t["orders"] = {k: v[perm].copy() for k, v in o.items()}
    elif layout == "shuffled":
        perm = rng.permutation(len(o["o_id"]))
        t["orders"] = {k: v[perm].copy() for k, v in o.items()}
    elif layout == "customer_shuffled":
        perm = rng.permutation(len(c["c_id"]))
        t["customer"] = {k: v[perm].copy() for k, v in c.items()}
    L.h.h2tap_load_snapshot(L.e, L.h.hot_path_tables(t, (L.h.H2TAP_Q18, L.h.H2TAP_Q3)), L.epoch + 1)
    L.epoch += 1
    r = L.h.h2tap_run_query(L.e, L.h.H2TAP_Q18)
    expect = {"clustered": 3, "one_row_swapped": 2, "shuffled": 2, "customer_shuffled": 1}[layout]
    assert r.plan_flags >> 3 == expect, (layout, r.plan_flags)  # bit3 orders, bit4 customer positional
    r.free()
    for thr in (Q18_HAVING, 4_000_000):
        want = oracle.q18(t, thr)
        assert_q18(L.q(18, [thr]), want)
        assert_q18(L.q(18, [thr], flags=HASH), want)
    want3 = oracle.q3(t, Q3_LO, b"A")
    got3 = L.q(3, [Q3_LO, 0x4100])
    for k in want3:
        assert np.array_equal(got3[k], want3[k]), k


@pytest.mark.parametrize("layout", ["clustered", "shuffled"])
@pytest.mark.parametrize("full", ["1", "0"])
def test_full_pass_batch(h, monkeypatch, order_mode, layout, full):
    """The batch's full pass: a Q6, Q1, Q18 batch reads order_line once — the
    shared Q6 + Q1 scan also stages Q18's keys and runs its probe. Ragged sizes around the 896-row
    chunk and the 4-row lane group, random parameters (HAVING exactly at a group's sum too),
    positional (clustered) and slot-array (shuffled orders) join indexes, the hash-join plan and
    both ORDER BY layouts, vs the oracle; H2TAP_FULL_PASS=0 runs the probe as its own kernel."""
    monkeypatch.setenv("H2TAP_FULL_PASS", full)
    e = h.h2tap_open(0)
    try:
        rng = np.random.default_rng(91)
        base = chgen.generate(1, 3, seed=91)
        if layout == "shuffled":
            perm = rng.permutation(len(base["orders"]["o_id"]))
            base["orders"] = {k: v[perm].copy() for k, v in base["orders"].items()}
        epoch = 0
        for n_keep in (100_003, 897, 896, 895, 130, 5, 1, 0):
            t = dict(base)
            t["order_line"] = {k: v[:n_keep].copy() for k, v in base["order_line"].items()}
            epoch += 1
            h.h2tap_load_snapshot(e, h.hot_path_tables(t), epoch)
            sums = oracle.q18(t, -(2**62))["amount_sum"]
            thrs = [Q18_HAVING, int(sums[len(sums) // 2]) if len(sums) else 0]
            for k, thr in enumerate(thrs):
                d_lo = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
                p6 = [d_lo, int(rng.integers(d_lo, chgen.TS_2025 + 10**12)), int(rng.integers(0, 6)),
                      int(rng.integers(4, 12))]
                cut = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
                f18 = HASH if k == 1 else 0
                rs = h.h2tap_run_queries(e, [(6, p6, 0), (1, [cut], 0), (18, [thr], f18)])
                got = []
                for r in rs:
                    x = r.to_numpy()
                    x["_nulls"] = dict(r.nulls)
                    got.append(x)
                    h.h2tap_free(r)
                assert_q6(got[0], oracle.q6(t, *p6))
                assert_q1(got[1], oracle.q1(t, cut))
                assert_q18(got[2], oracle.q18(t, thr))
    finally:
        h.h2tap_close(e)


@pytest.mark.parametrize("keys", ["dense", "one_sparse", "negative"])
def test_q1_keys_in_shared_pass_batches(h, keys):
    """Q1 inside the batch's shared / full pass with every ol_number dense, one key
    just outside the dense range (16) and one negative key (the global-table path and the
    general compact + emit), vs the oracle, in the bench's Q6 + Q1 + Q18 batch and in a Q6 + Q1
    batch, repeated (the tables are cleared between queries)."""
    t = chgen.generate(1, 3, seed=73)
    ol = t["order_line"]
    if keys == "one_sparse":
        ol["ol_number"][12345] = 16
    elif keys == "negative":
        ol["ol_number"][777] = -3
    e = h.h2tap_open(0)
    try:
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
        for batch in ([(6, None, 0), (1, None, 0), (18, None, 0)], [(6, None, 0), (1, [chgen.TS_1995], 0)],
                      [(6, None, 0), (1, None, 0), (18, None, 0)]):
            rs = h.h2tap_run_queries(e, batch)
            g1 = rs[1].to_numpy()
            for r in rs:
                h.h2tap_free(r)
            cut = batch[1][1][0] if batch[1][1] else Q1_CUTOFF
            assert_q1(g1, oracle.q1(t, cut))
    finally:
        h.h2tap_close(e)


@pytest.mark.parametrize("empty", ["all", "order_line", "orders", "customer"])
def test_full_pass_batch_empty_tables(h, empty):
    """The full-pass batch (Q6 + Q1 + Q18 in one order_line read) over empty
    tables: every table, or one of order_line / orders / customer emptied (the others full) —
    vs the oracle (NULL revenue, no Q1 groups, no Q18 rows where nothing joins)."""
    t = chgen.generate(1, 1 if empty == "all" else 2, seed=19)
    if empty != "all":
        t[empty] = {k: v[:0].copy() for k, v in t[empty].items()}
    e = h.h2tap_open(0)
    try:
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
        for _ in range(2):
            rs = h.h2tap_run_queries(e, [(6, None, 0), (1, None, 0), (18, [-100], 0)])
            got = []
            for r in rs:
                x = r.to_numpy()
                x["_nulls"] = dict(r.nulls)
                got.append(x)
                h.h2tap_free(r)
            assert_q6(got[0], oracle.q6(t, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI))
            assert_q1(got[1], oracle.q1(t, Q1_CUTOFF))
            assert_q18(got[2], oracle.q18(t, -100))
    finally:
        h.h2tap_close(e)


def test_full_size_w100_full_pass_shuffled_orders(h, w100):
    """BASELINE configs[1]/[2] size with the orders table shuffled: the bench's Q6 + Q1 + Q18 batch
    (the full pass) then probes through the perfect-hash slot array instead of the
    positional index, and the forced hash-join plan through open addressing — element by element
    vs the oracle (whose result does not depend on the row order)."""
    rng = np.random.default_rng(100)
    t = dict(w100)
    perm = rng.permutation(len(w100["orders"]["o_id"]))
    t["orders"] = {k: v[perm].copy() for k, v in w100["orders"].items()}
    e = h.h2tap_open(0)
    try:
        h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
        want6 = oracle.q6(t, Q6_D_LO, Q6_D_HI, Q6_Q_LO, Q6_Q_HI)
        want1 = oracle.q1(t, Q1_CUTOFF)
        want18 = oracle.q18(t, Q18_HAVING)
        for f18 in (0, HASH):
            rs = h.h2tap_run_queries(e, [(6, None, h.H2TAP_RESULT_DEVICE), (1, None, h.H2TAP_RESULT_DEVICE),
                                         (18, None, h.H2TAP_RESULT_DEVICE | f18)])
            got = []
            for r in rs:
                x = r.to_numpy()
                x["_nulls"] = {k: (v.copy() if hasattr(v, "copy") else v) for k, v in r.nulls.items()}
                got.append(x)
                h.h2tap_free(r)
            assert_q6(got[0], want6)
            assert_q1(got[1], want1)
            assert_q18(got[2], want18)
    finally:
        h.h2tap_close(e)
