#!/usr/bin/env python
"""Per-source-line instruction and stall-sample totals of one kernel from an ncu report
(`--page source --print-source cuda,sass`; the kernels must be built with -lineinfo).
usage: python scripts/ncu_lines.py <report.ncu-rep> <kernel regex> [top N]"""
import csv
import io
import subprocess
import sys
from collections import defaultdict

rep, kre = sys.argv[1], sys.argv[2]
top = int(sys.argv[3]) if len(sys.argv) > 3 else 40
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "-k", f"regex:{kre}",
                      "--print-source", "cuda,sass"], capture_output=True, text=True).stdout
agg = defaultdict(lambda: [0.0, 0.0, ""])
fname, hdr = "", None
for r in csv.reader(io.StringIO(out)):
    if not r:
        continue
    if r[0] == "File Path":
        fname = r[1].rsplit("/", 1)[-1]
        continue
    if r[0] == "Line No":
        hdr = r
        continue
    if hdr is None or len(r) < len(hdr) or not r[0].strip().isdigit():
        continue
    ie, iss = hdr.index("Instructions Executed"), hdr.index("Warp Stall Sampling (All Samples)")
    key = (fname, int(r[0]))
    num = lambda x: float(x) if x.replace(".", "", 1).isdigit() else 0.0
    agg[key][0] += num(r[ie])
    agg[key][1] += num(r[iss])
    agg[key][2] = r[1].strip()[:80]
ti = sum(v[0] for v in agg.values()) or 1
ts = sum(v[1] for v in agg.values()) or 1
print(f"total warp instructions {ti:.0f}, stall samples {ts:.0f}")
for (f, ln), (i, s, src) in sorted(agg.items(), key=lambda kv: -kv[1][1])[:top]:
    print(f"{i / ti * 100:5.1f}% instr {s / ts * 100:5.1f}% samples  {f}:{ln}: {src}")
