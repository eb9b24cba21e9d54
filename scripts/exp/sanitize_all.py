"""Small runs of every plan for compute-sanitizer (memcheck / racecheck): Q6, Q1, Q18, Q3, Q14,
Q12, Q4 at W=1 (clustered and shuffled orders), an appends + updates refresh, the layout scans."""
import os, sys
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import numpy as np
import chgen
import paper_conf_cidr_appuswamykpa17_b200 as h
for shuffled in (False, True):
    t = chgen.generate(1, 2, seed=7)
    if shuffled:
        perm = np.random.default_rng(7).permutation(len(t["orders"]["o_id"]))
        t["orders"] = {k: v[perm].copy() for k, v in t["orders"].items()}
    e = h.h2tap_open(0)
    plans = (h.H2TAP_Q6, h.H2TAP_Q1, h.H2TAP_Q18, h.H2TAP_Q3, h.H2TAP_Q14, h.H2TAP_Q12, h.H2TAP_Q4)
    h.h2tap_load_snapshot(e, h.hot_path_tables(t, plans), 1)
    for p in plans:
        r = h.h2tap_run_query(e, p); print("plan", p, r.nrows); r.free()
    rs = h.h2tap_run_queries(e, [(6, None, 0), (1, None, 0), (18, None, 0)])
    for r in rs: r.free()
    # a refresh: appended NewOrder rows + Delivery updates (host zone maps), then the batch again
    st = chgen.NewOrderState(1, 2)
    d = chgen.neworder_batch(st, 200, seed=7, batch=1, item=t["item"])
    dl = chgen.DeliveryState(); dl.add(t["orders"], 0, 0)
    w, c = chgen.delivery_inputs(20, seed=7, batch=1, w_lo=1, w_hi=2)
    upd = chgen.delivery_batch(dl, w, c, chgen.TS_2025)
    hot = h.hot_path_tables({**d, "customer": t["customer"], "item": t["item"]}, plans)
    hot.pop("customer"); hot.pop("item", None)
    upd = {k: {c2: v2 for c2, v2 in cols.items() if c2 == "ol_delivery_d"} for k, cols in upd.items() if k == "order_line"}
    h.h2tap_refresh(e, hot, upd, 2, first_row={"orders": len(t["orders"]["o_id"]), "order_line": len(t["order_line"]["ol_o_id"]),
                                               "new_order": len(t["new_order"]["no_o_id"])})
    rs = h.h2tap_run_queries(e, [(6, None, 0), (1, None, 0), (18, None, 0)])
    for r in rs: r.free()
    h.h2tap_close(e)
e = h.h2tap_open(0)
import torch
for layout in ("dsm", "pax", "nsm"):
    m = chgen.layout_matrix(100_003, 16, seed=3)
    enc = chgen.encode_layout(m, layout)
    buf = torch.from_numpy(np.ascontiguousarray(enc)).cuda()
    lid = {"dsm": h.H2TAP_DSM, "pax": h.H2TAP_PAX, "nsm": h.H2TAP_NSM}[layout]
    for cols in ([0], [1, 5], list(range(16)), [0, 3, 7]):
        s, ms = h.h2tap_layout_sum(e, buf, lid, 100_003, 16, cols)
        print(layout, cols[:3], s)
h.h2tap_close(e)
print("done")
