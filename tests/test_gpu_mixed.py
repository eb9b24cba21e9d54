"""Config C5 (mixed HTAP) end to end on one GPU, small: NewOrder appends and Delivery updates
committed by a host OLTP thread into the row store, epochs cut every 50 ms with
h2tap_refresh_rows (appends + copy-on-write updates), queries running concurrently. The final
epoch must equal the oracle over the final row store (every committed transaction)."""
import os
import sys

import numpy as np
import pytest

import chgen
import oracle
from chref import Q18_HAVING

pytestmark = pytest.mark.gpu
sys.path.insert(0, os.path.join(os.path.dirname(os.path.dirname(os.path.abspath(__file__))), "scripts"))


def test_mixed_run_final_epoch_parity():
    import htap_mixed
    import paper_conf_cidr_appuswamykpa17_b200 as h
    checked = {}

    def on_final(e, final):
        q6 = [chgen.TS_1995, chgen.TS_2025 + 365 * chgen.DAY_US, 1, 100000]
        r = h.h2tap_run_query(e, h.H2TAP_Q6, q6); got6 = r.to_numpy(); r.free()
        want6 = oracle.q6(final, *q6)
        assert int(got6["count_rows"][0]) == want6["count"]
        assert int(got6["revenue"][0]) == want6["revenue"]
        r = h.h2tap_run_query(e, h.H2TAP_Q1, [chgen.TS_2025]); got1 = r.to_numpy(); r.free()
        want1 = oracle.q1(final, chgen.TS_2025)
        for k in ("ol_number", "sum_qty", "sum_amount", "count_order"):
            assert np.array_equal(got1[k], want1[k]), k
        assert int(want1["count_order"].sum()) > 0  # deliveries happened and are visible
        r = h.h2tap_run_query(e, h.H2TAP_Q18, [Q18_HAVING]); got18 = r.to_numpy(); r.free()
        want18 = oracle.q18(final, Q18_HAVING)
        for k, _ in oracle.Q18_COLUMNS:
            assert np.array_equal(got18[k], want18[k]), k
        checked["ok"] = True

    out = htap_mixed.run(W=2, seconds=3.0, epoch_ms=50.0, txn_batch=200, tps=20_000.0,
                         on_final=on_final)
    assert checked.get("ok")
    assert out["epochs_published"] >= 5 and out["rows_updated"] > 0
    assert out["cow_pages_copied"] > 0
