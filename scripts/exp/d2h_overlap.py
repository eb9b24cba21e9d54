"""Is the result read-back overlapped with the next batch? Times, on the W=100 snapshot: a 120 MB
device->pinned copy alone; the Q6+Q1+Q18 batch alone (device results); both concurrently (the copy on
a second stream while the batch runs)."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.dirname(os.path.abspath(__file__)))))
import numpy as np, torch
import chgen, paper_conf_cidr_appuswamykpa17_b200 as h
t = chgen.generate(1, 101, seed=1)
e = h.h2tap_open(0)
h.h2tap_load_snapshot(e, h.hot_path_tables(t), 1)
del t
Q = [(h.H2TAP_Q6, None, h.H2TAP_RESULT_DEVICE), (h.H2TAP_Q1, None, h.H2TAP_RESULT_DEVICE),
     (h.H2TAP_Q18, None, h.H2TAP_RESULT_DEVICE)]
src = torch.empty(120_000_000, dtype=torch.uint8, device="cuda")
dst = torch.empty(120_000_000, dtype=torch.uint8, pin_memory=True)
s2 = torch.cuda.Stream()
def copy():
    with torch.cuda.stream(s2):
        dst.copy_(src, non_blocking=True)
    ev = torch.cuda.Event(); ev.record(s2); return ev
def batch():
    for r in h.h2tap_run_queries(e, Q): h.h2tap_free(r)
def med(f, n=10):
    for _ in range(3): f()
    ts = []
    for _ in range(n):
        torch.cuda.synchronize(); t0 = time.perf_counter(); f(); torch.cuda.synchronize(); ts.append((time.perf_counter() - t0) * 1e3)
    return round(float(np.median(ts)), 3)
print("copy 120 MB D2H alone ms", med(lambda: copy().synchronize()))
print("batch alone ms", med(batch))
print("copy + batch concurrently ms", med(lambda: (lambda ev: (batch(), ev.synchronize()))(copy())))
x = torch.empty(200_000_000, dtype=torch.float32, device="cuda")
s3 = torch.cuda.Stream()
def torch_work():
    with torch.cuda.stream(s3):
        for _ in range(3): x.mul_(1.0001)
    s3.synchronize()
print("torch elementwise alone ms", med(torch_work))
print("copy + torch elementwise ms", med(lambda: (lambda ev: (torch_work(), ev.synchronize()))(copy())))
# where does the batch's extra time go when a copy runs: device span vs host return
for label, f in (("alone", lambda: None), ("with copy", copy)):
    spans, walls = [], []
    for _ in range(8):
        torch.cuda.synchronize(); ev = f(); t0 = time.perf_counter(); batch(); walls.append((time.perf_counter() - t0) * 1e3)
        spans.append(h.h2tap_last_batch_ms(e))
        if ev is not None: ev.synchronize()
    print("batch", label, "device span ms", round(float(np.median(spans)), 3), "host wall ms", round(float(np.median(walls)), 3))
r = h.h2tap_run_query(e, h.H2TAP_Q18, None)
t0 = time.perf_counter(); r = h.h2tap_run_query(e, h.H2TAP_Q18, None); print("Q18 host result ms", round((time.perf_counter()-t0)*1e3, 3)); r.free()
h.h2tap_close(e)
