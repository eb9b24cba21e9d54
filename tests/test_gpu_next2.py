"""GPU parity of the NEXT-2 CH queries (Q14, Q12, Q4) through the C ABI against the CPU oracle
(pinned in tests/test_oracle_next2.py). Integer columns bit-exact; promo_revenue within
relative 1e-9 (both sides compute (100.0 * P) / (100.0 + S) in IEEE double: equal in practice)."""
import math

import numpy as np
import pytest

import chgen
import oracle
from chref import golden_next2, iso_us
from test_oracle_next2 import Q4_HI, Q4_LO, Q12_HI, Q14_HI, Q14_LO, mutate

pytestmark = pytest.mark.gpu
HASH = 4
PLANS = None


@pytest.fixture(scope="module")
def h():
    import paper_conf_cidr_appuswamykpa17_b200 as mod
    global PLANS
    PLANS = (mod.H2TAP_Q1, mod.H2TAP_Q6, mod.H2TAP_Q18, mod.H2TAP_Q14, mod.H2TAP_Q12, mod.H2TAP_Q4)
    return mod


class L2:
    def __init__(self, h):
        self.h, self.e, self.epoch = h, h.h2tap_open(0), 0

    def load(self, t):
        self.epoch += 1
        self.h.h2tap_load_snapshot(self.e, self.h.hot_path_tables(t, PLANS), self.epoch)

    def q(self, plan, params=None, flags=0):
        r = self.h.h2tap_run_query(self.e, plan, params, flags=flags)
        try:
            out = r.to_numpy()
            out["_nulls"] = dict(r.nulls)
            out["_flags"] = r.plan_flags
        finally:
            r.free()
        return out

    def close(self):
        self.h.h2tap_close(self.e)


@pytest.fixture
def L(h):
    x = L2(h)
    yield x
    x.close()


def assert_q14(got, want):
    if want["promo_revenue"] is None:
        assert got["_nulls"]["promo_revenue"][0] == 1 and got["count_rows"][0] == 0
        return
    assert got["_nulls"]["promo_revenue"][0] == 0
    assert (int(got["sum_promo"][0]), int(got["sum_amount"][0]), int(got["count_rows"][0])) == \
        (want["sum_promo"], want["sum_amount"], want["count"])
    assert math.isclose(float(got["promo_revenue"][0]), want["promo_revenue"], rel_tol=1e-9, abs_tol=0.0)


def assert_groups(got, want):
    for k in want:
        assert np.array_equal(got[k], want[k]), k


def run_all(h, L, t, rng=None, n_rand=2):
    L.load(t)
    assert_q14(L.q(h.H2TAP_Q14), oracle.q14(t, Q14_LO, Q14_HI))
    assert_groups(L.q(h.H2TAP_Q12), oracle.q12(t, Q12_HI))
    assert_groups(L.q(h.H2TAP_Q12, flags=HASH), oracle.q12(t, Q12_HI))
    assert_groups(L.q(h.H2TAP_Q4), oracle.q4(t, Q4_LO, Q4_HI))
    assert_groups(L.q(h.H2TAP_Q4, flags=HASH), oracle.q4(t, Q4_LO, Q4_HI))
    rng = rng or np.random.default_rng(0)
    for _ in range(n_rand):
        lo = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
        hi = int(rng.integers(lo - chgen.DAY_US, chgen.TS_2025 + 90 * chgen.DAY_US))
        pre = [b"PR", b"pr", b"XP", b"AB"][int(rng.integers(0, 4))]
        code = (pre[0] << 8) | pre[1]
        assert_q14(L.q(h.H2TAP_Q14, [lo, hi, code]), oracle.q14(t, lo, hi, pre))
        assert_groups(L.q(h.H2TAP_Q12, [hi]), oracle.q12(t, hi))
        assert_groups(L.q(h.H2TAP_Q4, [lo, hi]), oracle.q4(t, lo, hi))


@pytest.mark.parametrize("layout", ["clustered", "one_row_swapped", "shuffled"])
def test_clustered_orders_index_q12_q4(h, L, layout):
    """Q12 / Q4 take the positional orders index only while the device finds every orders row at
    its own key slot: the generated table (key order), one swapped pair of rows,
    fully shuffled rows — all equal the oracle on both index plans."""
    t = mutate(chgen.generate(1, 3, seed=43), 43)
    o = t["orders"]
    perm = np.arange(len(o["o_id"]))
    if layout == "one_row_swapped":
        perm[[7, 15000]] = perm[[15000, 7]]
    elif layout == "shuffled":
        perm = np.random.default_rng(43).permutation(len(perm))
    t["orders"] = {k: v[perm].copy() for k, v in o.items()}
    run_all(h, L, t, np.random.default_rng(43), n_rand=1)


def test_golden_fixture(h, L):
    t, p, want = golden_next2()
    L.load(t)
    lo, hi, pre = p["q14"]
    r = L.q(h.H2TAP_Q14, [lo, hi, (pre[0] << 8) | pre[1]])
    w = want["q14"]
    assert (int(r["sum_promo"][0]), int(r["sum_amount"][0]), int(r["count_rows"][0])) == \
        (w["sum_promo"], w["sum_amount"], w["count"])
    assert float(r["promo_revenue"][0]) == w["promo_num"] / w["promo_den"]
    for flags in (0, HASH):
        r = L.q(h.H2TAP_Q12, list(p["q12"]), flags=flags)
        assert [list(x) for x in zip(r["o_ol_cnt"].tolist(), r["high_line_count"].tolist(),
                                     r["low_line_count"].tolist())] == want["q12"]
        r = L.q(h.H2TAP_Q4, list(p["q4"]), flags=flags)
        assert [list(x) for x in zip(r["o_ol_cnt"].tolist(), r["order_count"].tolist())] == want["q4"]


@pytest.mark.parametrize("W,mode,seed,mut", [(1, "spread", 1, False), (3, "spread", 2, True),
                                             (2, "strict", 3, False), (2, "spread", 4, True)])
def test_parity_small(h, L, W, mode, seed, mut):
    t = chgen.generate(1, W + 1, seed=seed, mode=mode)
    if mut:
        t = mutate(t, seed)
    run_all(h, L, t, np.random.default_rng(seed))


@pytest.mark.parametrize("n", [0, 1, 3, 5, 127, 4097, 100_003])
def test_ragged_order_line(h, L, n):
    t = mutate(chgen.generate(1, 2, seed=5), 5)
    t["order_line"] = {k: v[:n].copy() for k, v in t["order_line"].items()}
    run_all(h, L, t, n_rand=1)


def test_empty_tables(h, L):
    t = chgen.generate(1, 2, seed=6)
    empty = {tb: {c: v[:0].copy() for c, v in cols.items()} for tb, cols in t.items()}
    run_all(h, L, empty, n_rand=1)
    t2 = dict(t)
    t2["item"] = empty["item"]
    run_all(h, L, t2, n_rand=1)


def test_sparse_group_keys_and_orphans(h, L):
    """o_ol_cnt outside [0, 16) (global-table path), negative and huge; orphan lines; lines of
    missing items; NULL carriers."""
    t = mutate(chgen.generate(1, 3, seed=7), 7)
    o = t["orders"]
    rng = np.random.default_rng(7)
    cnt = o["o_ol_cnt"].copy()
    pick = rng.random(len(cnt))
    cnt[pick < 0.2] = rng.integers(16, 2000, size=int((pick < 0.2).sum()))
    cnt[(pick >= 0.2) & (pick < 0.25)] = -3
    cnt[(pick >= 0.25) & (pick < 0.27)] = 2**31 - 1
    o["o_ol_cnt"] = cnt.astype(np.int32)
    ol = t["order_line"]
    orphan = rng.random(len(ol["ol_o_id"])) < 0.05
    ol["ol_o_id"] = np.where(orphan, 999_999, ol["ol_o_id"]).astype(np.int32)
    run_all(h, L, t, np.random.default_rng(7))


def test_item_map_in_global_memory_and_limits(h, L):
    """Sparse i_id (a map too large for shared memory) and an i_id span past the 2^28 limit."""
    t = mutate(chgen.generate(1, 2, seed=8), 8)
    it = dict(t["item"])
    it["i_id"] = (it["i_id"].astype(np.int64) * 7 + 11).astype(np.int32)  # 700k span
    t["item"] = it
    ol = dict(t["order_line"])
    ol["ol_i_id"] = (ol["ol_i_id"].astype(np.int64) * 7 + 11).astype(np.int32)
    t["order_line"] = ol
    L.load(t)
    r = L.q(h.H2TAP_Q14)
    assert r["_flags"] & 4 == 0
    assert_q14(r, oracle.q14(t, Q14_LO, Q14_HI))
    it2 = dict(it)
    it2["i_id"] = it["i_id"].copy()
    it2["i_id"][-1] = 2**30
    t["item"] = it2
    L.load(t)
    with pytest.raises(h.H2tapError) as ei:
        h.h2tap_run_query(L.e, h.H2TAP_Q14)
    assert ei.value.status == h.H2TAP_EPLAN


def test_duplicate_keys_rejected(h, L):
    t = chgen.generate(1, 2, seed=9)
    o = dict(t["orders"])
    o["o_id"] = o["o_id"].copy()
    o["o_id"][1] = o["o_id"][0]
    t2 = dict(t)
    t2["orders"] = o
    L.load(t2)
    for plan in (h.H2TAP_Q12, h.H2TAP_Q4):
        for flags in (0, HASH):
            with pytest.raises(h.H2tapError) as ei:
                h.h2tap_run_query(L.e, plan, flags=flags)
            assert ei.value.status == h.H2TAP_EDUPKEY
    it = dict(t["item"])
    it["i_id"] = it["i_id"].copy()
    it["i_id"][5] = it["i_id"][4]
    t3 = dict(t)
    t3["item"] = it
    L.load(t3)
    with pytest.raises(h.H2tapError) as ei:
        h.h2tap_run_query(L.e, h.H2TAP_Q14)
    assert ei.value.status == h.H2TAP_EDUPKEY


def test_device_results_and_batch(h, L):
    t = mutate(chgen.generate(1, 3, seed=10), 10)
    L.load(t)
    rs = h.h2tap_run_queries(L.e, [(h.H2TAP_Q14, None, h.H2TAP_RESULT_DEVICE), (h.H2TAP_Q12, None, 0),
                                   (h.H2TAP_Q4, None, h.H2TAP_RESULT_DEVICE), (h.H2TAP_Q6, None, 0),
                                   (h.H2TAP_Q12, [Q12_HI], h.H2TAP_RESULT_DEVICE)])
    try:
        assert len({r.epoch for r in rs}) == 1
        g = [r.to_numpy() for r in rs]
    finally:
        for r in rs:
            r.free()
    w14 = oracle.q14(t, Q14_LO, Q14_HI)
    assert math.isclose(float(g[0]["promo_revenue"][0]), w14["promo_revenue"], rel_tol=1e-9)
    assert_groups(g[1], oracle.q12(t, Q12_HI))
    assert_groups(g[2], oracle.q4(t, Q4_LO, Q4_HI))
    assert_groups(g[4], oracle.q12(t, Q12_HI))


def test_profile_kernels(h, L):
    t = chgen.generate(1, 2, seed=11)
    L.load(t)
    for plan, names in ((h.H2TAP_Q14, {"q14_item_map", "q14_scan_join_sum", "q14_finalize"}),
                        (h.H2TAP_Q12, {"q12_build", "q12_probe_groupby", "q12_emit"}),
                        (h.H2TAP_Q4, {"q4_build", "q4_semijoin_mark", "q4_count", "q4_emit"})):
        r = h.h2tap_run_query(L.e, plan, flags=h.H2TAP_QUERY_PROFILE)
        try:
            assert names <= {k for k, _ in r.kernels} and r.kernel_launches > 0
        finally:
            r.free()


def test_full_size_w100(h):
    """BASELINE configs[1] size (W=100, 30 M order_line rows), CH default parameters."""
    t = chgen.generate(1, 101, seed=1)
    L = L2(h)
    try:
        L.load(t)
        assert_q14(L.q(h.H2TAP_Q14), oracle.q14(t, Q14_LO, Q14_HI))
        assert_groups(L.q(h.H2TAP_Q12), oracle.q12(t, Q12_HI))
        assert_groups(L.q(h.H2TAP_Q4), oracle.q4(t, Q4_LO, Q4_HI))
        assert_groups(L.q(h.H2TAP_Q4, flags=HASH), oracle.q4(t, Q4_LO, Q4_HI))
    finally:
        L.close()
