"""Config C5 driven by the native C++ driver (tools/c5_native.cpp): NewOrder + Delivery threads,
an epoch cutter (h2tap_refresh_rows with appends + copy-on-write updates incl. new_order
tombstones) and the query loop, all C++ threads. After the run the driver publishes a final epoch
holding every committed transaction, queries it and dumps its row store and the results; this
test checks those results against the oracle on the dumped rows (the driver never touches the
oracle) and sanity-checks the report."""
import json
import math
import os
import subprocess
import sys

import numpy as np
import pytest

import oracle

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _load(d, name, dt, n):
    a = np.fromfile(os.path.join(d, name), dtype=dt)
    assert len(a) == n, (name, len(a), n)
    return a


def test_c5_native_final_epoch_matches_oracle(tmp_path):
    sys.path.insert(0, os.path.join(ROOT, "tools"))
    import c5_native
    exe = c5_native.build()
    r = subprocess.run([exe, "--warehouses", "2", "--seconds", "3", "--epoch-ms", "50", "--tps", "20000",
                        "--threads", "2", "--dump", str(tmp_path)], capture_output=True, text=True, timeout=300)
    assert r.returncode == 0, r.stderr[-2000:]
    rep = json.loads(r.stdout.strip().splitlines()[-1])
    assert rep["epochs_published"] > 5 and rep["neworder_tx_per_s"] > 1000 and rep["rows_updated"] > 0
    first, last = rep["q1_delivered_lines_first_last"]
    assert last > first  # Deliveries are visible to later epochs (Q1 at 2025-01-01)
    m = json.load(open(tmp_path / "manifest.json"))
    n_ol, n_o, n_c = m["n_ol"], m["n_o"], m["n_c"]
    t = {"order_line": {c: _load(tmp_path, c, dt, n_ol) for c, dt in
                        [("ol_w_id", np.int32), ("ol_d_id", np.int32), ("ol_o_id", np.int32), ("ol_number", np.int32),
                         ("ol_delivery_d", np.int64), ("ol_quantity", np.int32), ("ol_amount", np.int64)]},
         "orders": {c: _load(tmp_path, c, dt, n_o) for c, dt in
                    [("o_w_id", np.int32), ("o_d_id", np.int32), ("o_id", np.int32), ("o_c_id", np.int32),
                     ("o_ol_cnt", np.int32), ("o_carrier_id", np.int32), ("o_entry_d", np.int64)]},
         "customer": {c: _load(tmp_path, c, dt, n_c) for c, dt in
                      [("c_w_id", np.int32), ("c_d_id", np.int32), ("c_id", np.int32), ("c_last", np.int32)]}}
    res = m["results"]

    def col(q, name, dt):
        return np.fromfile(tmp_path / f"{q}.{name}", dtype=dt)
    w6 = oracle.q6(t, 915148800000000, 1577836800000000, 1, 100000)
    assert int(col("q6", "revenue", np.int64)[0]) == w6["revenue"]
    assert int(col("q6", "count_rows", np.int64)[0]) == w6["count"]
    w1 = oracle.q1(t, 1167696000000000)
    assert res["q1"]["nrows"] == len(w1["ol_number"])
    for k, dt in (("ol_number", np.int32), ("sum_qty", np.int64), ("sum_amount", np.int64), ("count_order", np.int64)):
        assert np.array_equal(col("q1", k, dt), w1[k]), k
    for k in ("avg_qty", "avg_amount"):
        for a, b in zip(col("q1", k, np.float64).tolist(), w1[k].tolist()):
            assert math.isclose(a, b, rel_tol=1e-9, abs_tol=0.0)
    w18 = oracle.q18(t, 20000)
    assert res["q18"]["nrows"] == len(w18["o_id"])
    for k, dt in oracle.Q18_COLUMNS:
        assert np.array_equal(col("q18", k, dt), w18[k]), k
