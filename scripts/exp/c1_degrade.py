"""Why does the C1 e2e (6 MB full reload + Q6) slow down over a process's life? Per engine: load
and query host times, medians per 50 iterations, for several engines opened in turn."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import numpy as np
import torch
import chgen
import paper_conf_cidr_appuswamykpa17_b200 as h
t = chgen.generate(1, 2, seed=1)
cols = {"order_line": {c: torch.from_numpy(t["order_line"][c]).pin_memory()
                       for c in ("ol_delivery_d", "ol_quantity", "ol_amount")}}
P = [chgen.ts_us("1999-01-01"), chgen.ts_us("2020-01-01"), 1, 100000]
for k in range(4):
    e = h.h2tap_open(0)
    ld, qq = [], []
    for i in range(200):
        t0 = time.perf_counter()
        h.h2tap_load_snapshot(e, cols, i + 1)
        t1 = time.perf_counter()
        r = h.h2tap_run_query(e, h.H2TAP_Q6, P)
        r.to_numpy()
        h.h2tap_free(r)
        t2 = time.perf_counter()
        ld.append((t1 - t0) * 1e3); qq.append((t2 - t1) * 1e3)
    print(k, "load ms per 50:", [round(float(np.median(ld[j:j + 50])), 3) for j in range(0, 200, 50)],
          "query ms:", [round(float(np.median(qq[j:j + 50])), 3) for j in range(0, 200, 50)], flush=True)
    h.h2tap_close(e)
