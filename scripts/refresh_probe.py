"""Time the refresh path (h2tap_load_snapshot_rows / _snapshot) for NewOrder-sized deltas."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import chgen
import paper_conf_cidr_appuswamykpa17_b200 as h
t = chgen.generate(1, 101, seed=1)
item = t.pop("item")
cols = {tb: list(c) for tb, c in h.hot_path_tables(t).items()}
recs = {tb: chgen.to_records(tb, t[tb]) for tb in ("order_line", "orders", "customer")}
e = h.h2tap_open(0)
t0 = time.perf_counter(); h.h2tap_load_snapshot_rows(e, recs, 1, columns=cols); print("full rows load", time.perf_counter() - t0)
st = chgen.NewOrderState(1, 101)
n = {tb: len(recs[tb]) for tb in ("order_line", "orders")}
ep = 1
for size in (2000, 20000, 20000, 20000, 200000):
    d = chgen.neworder_batch(st, size, seed=1, batch=ep, item=item)
    dr = {tb: chgen.to_records(tb, d[tb]) for tb in ("order_line", "orders")}
    ep += 1
    t0 = time.perf_counter()
    h.h2tap_load_snapshot_rows(e, dr, ep, full_reload=False, first_row=n, columns=cols, flags=h.H2TAP_LOAD_ASYNC)
    t1 = time.perf_counter(); h.h2tap_sync(e); t2 = time.perf_counter()
    for tb in n: n[tb] += len(dr[tb])
    mb = sum(len(dr[tb]) * 40 for tb in dr) / 1e6
    print(f"rows delta {size} txns ({mb:.1f} MB): load {1e3*(t1-t0):.2f} ms sync {1e3*(t2-t1):.2f} ms")
    # column path for comparison
    ep += 1
    d = chgen.neworder_batch(st, size, seed=1, batch=1000 + ep, item=item)
    dc = {tb: {c: d[tb][c] for c in cols[tb]} for tb in ("order_line", "orders")}
    t0 = time.perf_counter()
    h.h2tap_load_snapshot(e, dc, ep, full_reload=False, first_row=n, flags=h.H2TAP_LOAD_ASYNC)
    t1 = time.perf_counter(); h.h2tap_sync(e); t2 = time.perf_counter()
    for tb in n: n[tb] += len(dc[tb][cols[tb][0]])
    print(f"cols delta {size} txns: load {1e3*(t1-t0):.2f} ms sync {1e3*(t2-t1):.2f} ms")
h.h2tap_close(e)
