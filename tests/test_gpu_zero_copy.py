"""NEXT-4: zero-copy host-resident snapshots (H2TAP_LOAD_ZERO_COPY) — the kernels read the caller's
pinned host columns over PCIe, the paper's UVA data sharing. Every
plan must give the oracle's result on host-resident, HBM-resident and mixed snapshots."""
import numpy as np
import pytest

import chgen
import oracle
from test_gpu_q3 import assert_q3
from test_oracle_q3 import Q3_LO

pytestmark = pytest.mark.gpu
Q1_CUT = chgen.ts_us("2007-01-02")
Q6_P = (chgen.ts_us("1999-01-01"), chgen.ts_us("2020-01-01"), 1, 100000)


@pytest.fixture(scope="module")
def h():
    import paper_conf_cidr_appuswamykpa17_b200 as mod
    return mod


def plans(h):
    return (h.H2TAP_Q1, h.H2TAP_Q6, h.H2TAP_Q18, h.H2TAP_Q3)


def check_all(h, e, t):
    r = h.h2tap_run_query(e, h.H2TAP_Q6, list(Q6_P)); g = r.to_numpy(); r.free()
    w = oracle.q6(t, *Q6_P)
    assert int(g["revenue"][0]) == w["revenue"] and int(g["count_rows"][0]) == w["count"]
    r = h.h2tap_run_query(e, h.H2TAP_Q1, [Q1_CUT]); g = r.to_numpy(); r.free()
    w = oracle.q1(t, Q1_CUT)
    for k in ("ol_number", "sum_qty", "sum_amount", "count_order"):
        assert np.array_equal(g[k], w[k]), k
    for flags in (0, 4):
        r = h.h2tap_run_query(e, h.H2TAP_Q18, [20000], flags=flags); g = r.to_numpy(); r.free()
        w = oracle.q18(t, 20000)
        for k in w:
            assert np.array_equal(g[k], w[k]), k
    r = h.h2tap_run_query(e, h.H2TAP_Q3); g = r.to_numpy(); r.free()
    assert_q3(g, oracle.q3(t, Q3_LO))


def test_host_resident_snapshot_and_append(h):
    base = chgen.generate(1, 3, seed=70)
    st = chgen.NewOrderState(1, 3)
    delta = chgen.neworder_batch(st, 3000, seed=70, batch=0, item=base["item"])
    hot = h.hot_path_tables(base, plans(h))
    cap = {k: len(next(iter(v.values()))) + len(next(iter(delta[k].values()))) if k in delta else 0
           for k, v in hot.items()}
    pin = h.pinned_tables(hot, cap)
    e = h.h2tap_open(0)
    try:
        h.h2tap_load_snapshot(e, pin, 1, flags=h.H2TAP_LOAD_ZERO_COPY)
        check_all(h, e, base)
        # the OLTP side appends rows in place into the same pinned buffers, then publishes them
        first = {k: len(next(iter(hot[k].values()))) for k in delta}
        dtab = {}
        for k, cols in h.hot_path_tables({**delta, "customer": base["customer"]}, plans(h)).items():
            if k not in delta:
                continue
            dtab[k] = {}
            for c, a in cols.items():
                full = pin[k][c].as_strided((first[k] + len(a),), (1,))  # same storage, longer view
                import torch
                full[first[k]:].copy_(torch.from_numpy(np.ascontiguousarray(a)))
                dtab[k][c] = full[first[k]:]
        h.h2tap_load_snapshot(e, dtab, 2, flags=h.H2TAP_LOAD_ZERO_COPY, full_reload=False, first_row=first)
        merged = {k: dict(v) for k, v in base.items()}
        for k in delta:
            merged[k] = {c: np.concatenate([base[k][c], delta[k][c]]) for c in base[k]}
        check_all(h, e, merged)
        st_ = h.h2tap_get_store_stats(e)
        assert st_["device_bytes"] == 0  # nothing copied to HBM
    finally:
        h.h2tap_close(e)


def test_mixed_residency(h):
    """order_line host-resident (the big fact table), orders / customer / new_order in HBM."""
    t = chgen.generate(1, 3, seed=71)
    hot = h.hot_path_tables(t, plans(h))
    e = h.h2tap_open(0)
    try:
        pin = h.pinned_tables({"order_line": hot["order_line"]})
        h.h2tap_load_snapshot(e, pin, 1, flags=h.H2TAP_LOAD_ZERO_COPY)
        h.h2tap_load_snapshot(e, {k: v for k, v in hot.items() if k != "order_line"}, 2)
        check_all(h, e, t)
        # back to HBM for order_line: needs a full reload
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_load_snapshot(e, {"order_line": hot["order_line"]}, 3, full_reload=False,
                                  first_row={"order_line": len(hot["order_line"]["ol_w_id"])})
        assert ei.value.status == h.H2TAP_ESHAPE
        h.h2tap_load_snapshot(e, {"order_line": hot["order_line"]}, 4)
        check_all(h, e, t)
    finally:
        h.h2tap_close(e)


def test_zero_copy_errors(h):
    import torch
    t = chgen.generate(1, 2, seed=72)
    hot = h.hot_path_tables(t, plans(h))
    e = h.h2tap_open(0)
    try:
        with pytest.raises(h.H2tapError) as ei:  # pageable numpy buffers
            h.h2tap_load_snapshot(e, {"orders": hot["orders"]}, 1, flags=h.H2TAP_LOAD_ZERO_COPY)
        assert ei.value.status == h.H2TAP_EINVAL
        pin = h.pinned_tables(hot)
        h.h2tap_load_snapshot(e, pin, 2, flags=h.H2TAP_LOAD_ZERO_COPY)
        with pytest.raises(h.H2tapError) as ei:  # in-place update of a host-resident table
            h.h2tap_refresh(e, None, {"orders": {"o_c_id": (np.array([0], np.uint32), np.array([3], np.int32))}}, 3)
        assert ei.value.status in (h.H2TAP_EPLAN, h.H2TAP_EINVAL)
        other = h.pinned_tables({"new_order": {k: v[:5] for k, v in hot["new_order"].items()}})
        n_no = len(hot["new_order"]["no_o_id"])
        with pytest.raises(h.H2tapError) as ei:  # append from a different buffer
            h.h2tap_load_snapshot(e, other, 4, flags=h.H2TAP_LOAD_ZERO_COPY, full_reload=False,
                                  first_row={"new_order": n_no})
        assert ei.value.status in (h.H2TAP_ESHAPE, h.H2TAP_EINVAL)
        check_all(h, e, t)  # failed calls changed nothing
    finally:
        h.h2tap_close(e)
