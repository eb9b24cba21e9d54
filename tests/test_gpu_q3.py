"""GPU parity of CH Q3 (NEXT-2: customer ⋈ new_order ⋈ orders ⋈ order_line, GROUP BY, ORDER BY
revenue DESC, o_entry_d) through the C ABI against the CPU oracle (pinned in
tests/test_oracle_q3.py). Every column bit-exact, in the total order of DESIGN.md R33."""
import numpy as np
import pytest

import chgen
import oracle
from chref import golden_q3
from test_oracle_q3 import Q3_LO, mutate

pytestmark = pytest.mark.gpu
HASH = 4
COLS = ("ol_o_id", "ol_w_id", "ol_d_id", "revenue", "o_entry_d")


@pytest.fixture(scope="module")
def h():
    import paper_conf_cidr_appuswamykpa17_b200 as mod
    return mod


def p2(prefix: bytes) -> int:
    b = bytes(prefix) + b"\0\0"
    return b[0] << 8 | b[1]


class Eng:
    def __init__(self, h):
        self.h, self.e, self.epoch = h, h.h2tap_open(0), 0

    def load(self, t):
        self.epoch += 1
        self.h.h2tap_load_snapshot(self.e, self.h.hot_path_tables(t, (self.h.H2TAP_Q3, self.h.H2TAP_Q18)),
                                   self.epoch)

    def q3(self, lo=Q3_LO, prefix=b"A", flags=0):
        r = self.h.h2tap_run_query(self.e, self.h.H2TAP_Q3, [lo, p2(prefix)], flags=flags)
        try:
            out = r.to_numpy()
            out["_flags"] = r.plan_flags
        finally:
            r.free()
        return out

    def close(self):
        self.h.h2tap_close(self.e)


@pytest.fixture
def E(h):
    x = Eng(h)
    yield x
    x.close()


def assert_q3(got, want):
    assert list(got)[:5] == list(COLS)
    for k in COLS:
        assert np.array_equal(got[k], want[k]), (k, got[k][:8], want[k][:8])


def check(E, t, lo=Q3_LO, prefix=b"A"):
    want = oracle.q3(t, lo, prefix)
    for flags in (0, HASH):
        got = E.q3(lo, prefix, flags)
        assert_q3(got, want)
        assert (got["_flags"] & 1) == (0 if flags else got["_flags"] & 1)
    return want


def test_golden_fixture(h, E):
    t, (lo, pre), want = golden_q3()
    E.load(t)
    got = E.q3(lo, pre)
    assert list(zip(*[got[k].tolist() for k in COLS])) == want
    assert list(zip(*[E.q3(lo, pre, HASH)[k].tolist() for k in COLS])) == want


@pytest.mark.parametrize("W,mode", [(1, "spread"), (3, "spread"), (2, "strict")])
def test_generated(h, E, W, mode):
    t = chgen.generate(1, W + 1, seed=40 + W, mode=mode)
    E.load(t)
    want = check(E, t)
    assert len(want["ol_o_id"]) > 0
    rng = np.random.default_rng(W)
    for pre in (b"", b"AK", b"z", b"0"):
        check(E, t, int(rng.integers(chgen.TS_1995, chgen.TS_2025)), pre)
    check(E, t, chgen.TS_2025, b"A")  # nothing qualifies


@pytest.mark.parametrize("seed", [1, 2])
def test_mutated_edges(h, E, seed):
    """duplicated / orphan new_order rows (multiplicity), entries at the cutoff, equal revenues,
    look-alike states."""
    t = mutate(chgen.generate(1, 3, seed=50 + seed), seed)
    E.load(t)
    for pre in (b"A", b"AK", b"a", b"B"):
        check(E, t, Q3_LO, pre)


def test_ragged_and_empty(h, E):
    base = chgen.generate(1, 2, seed=60)
    for n_no in (0, 1, 31, 33, 4097):
        t = {k: dict(v) for k, v in base.items()}
        t["new_order"] = {k: v[:n_no] for k, v in base["new_order"].items()}
        E.load(t)
        check(E, t, chgen.TS_1995, b"")
    for n_ol in (0, 1, 5, 100_003):
        t = {k: dict(v) for k, v in base.items()}
        t["order_line"] = {k: v[:n_ol] for k, v in base["order_line"].items()}
        E.load(t)
        check(E, t, chgen.TS_1995, b"")


def test_duplicate_keys_rejected(h, E):
    t = chgen.generate(1, 2, seed=61)
    t2 = {k: dict(v) for k, v in t.items()}
    t2["orders"]["o_id"] = t["orders"]["o_id"].copy()
    t2["orders"]["o_id"][7] = t2["orders"]["o_id"][6]
    E.load(t2)
    for flags in (0, HASH):
        with pytest.raises(h.H2tapError) as ei:
            E.q3(flags=flags)
        assert ei.value.status == h.H2TAP_EDUPKEY
    t3 = {k: dict(v) for k, v in t.items()}
    t3["customer"]["c_id"] = t["customer"]["c_id"].copy()
    t3["customer"]["c_id"][3] = t3["customer"]["c_id"][2]
    E.load(t3)
    with pytest.raises(h.H2tapError) as ei:
        E.q3()
    assert ei.value.status == h.H2TAP_EDUPKEY
    with pytest.raises(h.H2tapError) as ei:
        h.h2tap_run_query(E.e, h.H2TAP_Q3, [Q3_LO, 0x0041])  # c1 without c0
    assert ei.value.status == h.H2TAP_EINVAL


def test_batch_with_q18_and_device_results(h, E):
    """Q3 shares Q18's scratch: interleaved in one batch both stay correct."""
    t = mutate(chgen.generate(1, 3, seed=62), 62)
    E.load(t)
    rs = h.h2tap_run_queries(E.e, [(h.H2TAP_Q3, None, h.H2TAP_RESULT_DEVICE), (h.H2TAP_Q18, None, 0),
                                   (h.H2TAP_Q3, [chgen.TS_1995, p2(b"")], 0), (h.H2TAP_Q18, [-1], h.H2TAP_RESULT_DEVICE),
                                   (h.H2TAP_Q3, None, 0)])
    try:
        assert len({r.epoch for r in rs}) == 1
        g = [r.to_numpy() for r in rs]
    finally:
        for r in rs:
            r.free()
    w3 = oracle.q3(t, Q3_LO)
    assert_q3(g[0], w3)
    assert_q3(g[2], oracle.q3(t, chgen.TS_1995, b""))
    assert_q3(g[4], w3)
    w18 = oracle.q18(t, 20000)
    for k in w18:
        assert np.array_equal(g[1][k], w18[k]), k
    w18 = oracle.q18(t, -1)
    for k in w18:
        assert np.array_equal(g[3][k], w18[k]), k


def test_neworder_epochs(h, E):
    """NewOrder appends orders, order_line and new_order rows: the next epoch's Q3 sees them."""
    base = chgen.generate(1, 3, seed=63)
    E.load(base)
    st = chgen.NewOrderState(1, 3)
    d = chgen.neworder_batch(st, 2000, seed=63, batch=0, item=base["item"])
    plans = (h.H2TAP_Q3, h.H2TAP_Q18)
    delta = {k: v for k, v in h.hot_path_tables({**d, "customer": base["customer"]}, plans).items() if k != "customer"}
    first = {k: len(next(iter(base[k].values()))) for k in delta}
    E.epoch += 1
    h.h2tap_load_snapshot(E.e, delta, E.epoch, full_reload=False, first_row=first)
    merged = {k: dict(v) for k, v in base.items()}
    for k in delta:
        merged[k] = {c: np.concatenate([base[k][c], d[k][c]]) for c in base[k]}
    want = check(E, merged, Q3_LO, b"")
    assert (want["o_entry_d"] >= chgen.TS_2025).any()  # the new orders are in the result


def test_profile_kernels(h, E):
    E.load(chgen.generate(1, 2, seed=64))
    r = h.h2tap_run_query(E.e, h.H2TAP_Q3, flags=h.H2TAP_QUERY_PROFILE)
    try:
        names = {k for k, _ in r.kernels}
        assert {"q3_build", "q3_mark", "q3_probe_groupjoin", "q3_emit", "q18_bucket_sort_emit"} <= names
        assert r.kernel_launches > 0
    finally:
        r.free()


def test_full_size_w100(h):
    """BASELINE configs[1] size (W=100, 30 M order_line rows, 900 k new_order rows), CH defaults."""
    t = chgen.generate(1, 101, seed=1)
    E = Eng(h)
    try:
        E.load(t)
        want = oracle.q3(t, Q3_LO)
        assert len(want["ol_o_id"]) > 1000
        assert_q3(E.q3(), want)
        assert_q3(E.q3(flags=HASH), want)
    finally:
        E.close()
