"""Where C1's e2e time goes (host wall clock, medians of 50): the 6 MB reload alone, the Q6 query
alone (host result), and both — plus the same with H2TAP_LOAD_BORROW (no staging copy)."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import numpy as np, torch
import chgen, paper_conf_cidr_appuswamykpa17_b200 as h
t = chgen.generate(1, 2, seed=1)
cols = {"order_line": {c: torch.from_numpy(t["order_line"][c]).pin_memory()
                       for c in ("ol_delivery_d", "ol_quantity", "ol_amount")}}
P = [chgen.ts_us("2007-01-02"), chgen.ts_us("2020-01-01"), 1, 100000]
e = h.h2tap_open(0)
ep = [1]
h.h2tap_load_snapshot(e, cols, 1)
def load(flags=0):
    ep[0] += 1; h.h2tap_load_snapshot(e, cols, ep[0], flags=flags)
    if flags: h.h2tap_sync(e)
def query(flags=0):
    r = h.h2tap_run_query(e, h.H2TAP_Q6, P, flags=flags); v = r.to_numpy() if not flags else None; h.h2tap_free(r)
def med(f, n=50):
    for _ in range(5): f()
    ts = []
    for _ in range(n):
        t0 = time.perf_counter(); f(); ts.append((time.perf_counter() - t0) * 1e3)
    return round(float(np.median(ts)), 4)
print("load 6 MB", med(load))
print("load 6 MB borrow+async+sync", med(lambda: load(h.H2TAP_LOAD_ASYNC | h.H2TAP_LOAD_BORROW)))
print("query (host result)", med(query))
print("query (device result)", med(lambda: query(h.H2TAP_RESULT_DEVICE)))
print("load+query", med(lambda: (load(), query())))
r = h.h2tap_run_query(e, h.H2TAP_Q6, P, flags=h.H2TAP_RESULT_DEVICE); print("device_ms", r.device_ms, "e2e_ms", r.e2e_ms); h.h2tap_free(r)
h.h2tap_close(e)
