"""Where does host time go per query? python wall vs C++ wall (e2e_ms) vs device_ms."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import numpy as np
import chgen
import paper_conf_cidr_appuswamykpa17_b200 as h
t = chgen.generate(1, 101, seed=1)
e = h.h2tap_open(0)
h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
for flags in (h.H2TAP_RESULT_DEVICE, h.H2TAP_RESULT_DEVICE | h.H2TAP_QUERY_PROFILE):
    for plan in (6, 1, 18):
        py, cpp, dev = [], [], []
        for i in range(30):
            t0 = time.perf_counter()
            r = h.h2tap_run_query(e, plan, flags=flags)
            t1 = time.perf_counter()
            cpp.append(r.e2e_ms); dev.append(r.device_ms)
            h.h2tap_free(r)
            t2 = time.perf_counter()
            py.append((t2 - t0) * 1e3)
        print(f"flags={flags} Q{plan}: python {np.median(py):.4f} ms  c++ {np.median(cpp):.4f} ms  device {np.median(dev):.4f} ms")
h.h2tap_close(e)
