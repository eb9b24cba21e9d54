"""Config C1 (Q6 at W=1) e2e, repeated: the spread of the host-timed e2e medians (bench.c1_line)."""
import os, sys
ROOT = os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
sys.path.insert(0, ROOT)
sys.argv = [os.path.join(ROOT, "bench.py")]
import bench  # noqa: E402
import paper_conf_cidr_appuswamykpa17_b200 as h  # noqa: E402
a = bench.parse()
for _ in range(4):
    c = bench.c1_line(h, a)
    print({k: c[k] for k in ("device_ms", "call_ms", "e2e_ms", "e2e_zero_copy_ms", "oracle_ms")}, flush=True)
