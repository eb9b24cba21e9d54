"""Do a device->host and a host->device copy on two streams overlap (separate copy engines)?"""
import time, numpy as np, torch
d = torch.empty(120_000_000, dtype=torch.uint8, device="cuda")
hd = torch.empty(120_000_000, dtype=torch.uint8, pin_memory=True)
hs = torch.ones(5_000_000, dtype=torch.uint8, pin_memory=True)
ds = torch.empty(5_000_000, dtype=torch.uint8, device="cuda")
a, b = torch.cuda.Stream(), torch.cuda.Stream()
def t(f, n=10):
    f(); torch.cuda.synchronize(); ts = []
    for _ in range(n):
        torch.cuda.synchronize(); t0 = time.perf_counter(); r = f(); ts.append((time.perf_counter() - t0) * 1e3)
    return round(float(np.median(ts)), 3)
def d2h():
    with torch.cuda.stream(a): hd.copy_(d, non_blocking=True)
    a.synchronize()
def h2d():
    with torch.cuda.stream(b): ds.copy_(hs, non_blocking=True)
    b.synchronize()
def both():
    with torch.cuda.stream(a): hd.copy_(d, non_blocking=True)
    t0 = time.perf_counter()
    with torch.cuda.stream(b): ds.copy_(hs, non_blocking=True)
    b.synchronize(); t1 = time.perf_counter(); a.synchronize()
    return (t1 - t0) * 1e3
print("D2H 120 MB alone", t(d2h), "ms; H2D 5 MB alone", t(h2d), "ms")
both(); r = [both() for _ in range(10)]
print("H2D 5 MB while a 120 MB D2H runs: H2D done after", round(float(np.median(r)), 3), "ms")
print("props asyncEngineCount", torch.cuda.get_device_properties(0))
