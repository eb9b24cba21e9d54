#!/usr/bin/env python
"""NEXT-3 / NEXT-4 measurement: the paper's layout experiment (§5.3, Fig. 10 / Fig. 11)
on one B200 through the C ABI (h2tap_layout_sum).

  SELECT SUM(col1 + ... + colN) FROM dataset, N = 1, 2, 4, 8, 16, over a table of 16 int32
  attributes stored as DSM, PAX (4 KB pages = 16 minipages x 64 values) or NSM.

Residency:
  hbm  — table in HBM (Fig. 11 is this with a 1 GB table and N = 2; on a B200 the paper's full
         16 GB table fits, so both sizes are run);
  host — table in PINNED host memory, read by the kernel over PCIe with no copy (the paper's UVA
         setting of Fig. 10, Caldera's data-sharing mechanism, L484-490, L568-572).

Per (residency, size, layout, N): K timed kernel runs (CUDA events inside the library), median.
Algorithmic bytes = N x 4 B x rows (the attributes the query reads). Denominators: HBM = the
measured copy peak (MEASURED_PEAKS.json); host = the pinned H2D cudaMemcpy bandwidth measured in
the same run (same PCIe link, DMA engines). The table values follow a closed form (value(r, c) =
(r mod 2^20) * 16 + c), so every run's sum is checked exactly.

Usage: python scripts/layout_bench.py [--rows 270000000] [--host-rows 67108864] [--steps 5] [--out F]
"""
import argparse
import json
import os
import sys

import numpy as np

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
sys.path.insert(0, os.path.join(ROOT, "tests"))


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--rows", type=int, default=270_000_000, help="paper: 16 GB / 270 M records")
    ap.add_argument("--small-rows", type=int, default=16_777_216, help="paper Fig. 11: 1 GB")
    ap.add_argument("--host-rows", type=int, default=67_108_864, help="host-resident rows (4 GB)")
    ap.add_argument("--steps", type=int, default=5)
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    import torch
    import paper_conf_cidr_appuswamykpa17_b200 as h
    from test_gpu_layout import build_closed_form, closed_form
    K, k = 1 << 20, 16
    peaks = json.load(open(os.path.join(ROOT, "MEASURED_PEAKS.json"))) \
        if os.path.exists(os.path.join(ROOT, "MEASURED_PEAKS.json")) else {}
    hbm_peak = peaks.get("hbm_gbs", 6650.0)
    # PCIe denominator: pinned H2D copy bandwidth on this box
    src = torch.empty(1 << 30, dtype=torch.uint8, pin_memory=True)
    dst = torch.empty(1 << 30, dtype=torch.uint8, device="cuda")
    ts = []
    for _ in range(5):
        b, en = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        b.record(); dst.copy_(src, non_blocking=True); en.record(); torch.cuda.synchronize()
        ts.append(b.elapsed_time(en))
    pcie_gbs = (1 << 30) / (np.median(ts[1:]) * 1e-3) / 1e9
    del src, dst
    e = h.h2tap_open(0)
    rows = []
    layouts = (("dsm", h.H2TAP_DSM), ("pax", h.H2TAP_PAX), ("nsm", h.H2TAP_NSM))
    runs = [("hbm", a.rows), ("hbm", a.small_rows), ("host", a.host_rows)]
    for where, n in runs:
        for lay, lid in layouts:
            d = build_closed_form(n, k, K, lay)
            if where == "host":
                hd = torch.empty(d.shape, dtype=torch.int32, pin_memory=True)
                hd.copy_(d)
                del d
                torch.cuda.empty_cache()
                d = hd
            for N in (1, 2, 4, 8, 16):
                cols = list(range(N))
                ms = []
                for i in range(a.steps + 1):
                    got, t = h.h2tap_layout_sum(e, d, lid, n, k, cols)
                    assert got == closed_form(n, k, cols, K), (where, lay, N)
                    if i:
                        ms.append(t)
                med = float(np.median(ms))
                alg = 4 * N * n
                gbs = alg / (med * 1e-3) / 1e9
                peak = hbm_peak if where == "hbm" else pcie_gbs
                rows.append({"residency": where, "rows": n, "table_GB": round(4 * k * n / 1e9, 2),
                             "layout": lay, "N": N, "ms": round(med, 4), "alg_GBps": round(gbs, 1),
                             "frac_of_peak": round(gbs / peak, 3)})
                print(json.dumps(rows[-1]), flush=True)
            del d
            torch.cuda.empty_cache()
    h.h2tap_close(e)
    line = {"what": "NEXT-3/NEXT-4 layout scan SUM(col1+...+colN), one B200 (PAPER.md §5.3)",
            "hbm_peak_GBps": hbm_peak, "pcie_h2d_GBps": round(pcie_gbs, 1), "steps": a.steps, "runs": rows}
    if a.out:
        open(a.out, "w").write(json.dumps(line) + "\n")


if __name__ == "__main__":
    main()
