"""Phase times of the pipelined incremental e2e loop (refresh, batch, D2H issue, drain wait)."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import numpy as np, torch
import chgen, bench, paper_conf_cidr_appuswamykpa17_b200 as h
t = chgen.generate(1, 101, seed=1)
inc, nolf, nof, rows = bench.incremental_inputs(h, t, 1, 101, 16, 10000, 1000)
e = h.h2tap_open(0)
h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
del t
h.h2tap_reserve(e, "order_line", nolf); h.h2tap_reserve(e, "orders", nof)
Q = [(h.H2TAP_Q6, None, h.H2TAP_RESULT_DEVICE), (h.H2TAP_Q1, None, h.H2TAP_RESULT_DEVICE),
     (h.H2TAP_Q18, None, h.H2TAP_RESULT_DEVICE)]
s2 = torch.cuda.Stream(); bufs = {}; pending = None; ep = 1
ph = {"refresh": [], "batch": [], "issue": [], "drain": [], "step": []}
for k, (delta, upd, first, _) in enumerate(inc):
    t0 = time.perf_counter(); ep += 1
    h.h2tap_refresh(e, delta, upd, ep, first_row=first); t1 = time.perf_counter()
    rs = h.h2tap_run_queries(e, Q); t2 = time.perf_counter()
    with torch.cuda.stream(s2):
        for r in rs:
            if not r.nrows: continue
            for name, c in r.columns.items():
                src = torch.as_tensor(c, device="cuda")
                b = bufs.get(name)
                if b is None or b.numel() < src.numel():
                    b = bufs[name] = torch.empty(int(src.numel() * 1.25) + 1024, dtype=src.dtype, pin_memory=True)
                b[:src.numel()].copy_(src, non_blocking=True)
        ev = torch.cuda.Event(); ev.record(s2)
    t3 = time.perf_counter()
    if pending:
        pending[1].synchronize()
        for r in pending[0]: h.h2tap_free(r)
    t4 = time.perf_counter()
    pending = (rs, ev)
    if k >= 4:
        for n_, v in (("refresh", t1 - t0), ("batch", t2 - t1), ("issue", t3 - t2), ("drain", t4 - t3), ("step", t4 - t0)):
            ph[n_].append(v * 1e3)
print({k: round(float(np.median(v)), 3) for k, v in ph.items()})
h.h2tap_close(e)
