"""Config C1 (Q6 at W=1): where the ~40 us per call go — python wall, the library's own wall
(result.e2e_ms), the query's device span (result.device_ms), for device and host results."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import numpy as np
import chgen
import paper_conf_cidr_appuswamykpa17_b200 as h
t = chgen.generate(1, 2, seed=1)
e = h.h2tap_open(0)
h.h2tap_load_snapshot(e, {"order_line": {c: t["order_line"][c] for c in ("ol_delivery_d", "ol_quantity", "ol_amount")}}, 1)
for flags in (h.H2TAP_RESULT_DEVICE, 0):
    for _ in range(50):
        h.h2tap_free(h.h2tap_run_query(e, 6, flags=flags))
    py, cpp, dev, fr = [], [], [], []
    for i in range(200):
        t0 = time.perf_counter()
        r = h.h2tap_run_query(e, 6, flags=flags)
        t1 = time.perf_counter()
        cpp.append(r.e2e_ms); dev.append(r.device_ms)
        h.h2tap_free(r)
        t2 = time.perf_counter()
        py.append((t1 - t0) * 1e3); fr.append((t2 - t1) * 1e3)
    print(f"flags={flags} Q6 W=1: python call {np.median(py)*1e3:.1f} us  library {np.median(cpp)*1e3:.1f} us  "
          f"device {np.median(dev)*1e3:.1f} us  free {np.median(fr)*1e3:.1f} us")
h.h2tap_close(e)
