"""Top SASS lines by warp-stall samples for one kernel of an ncu report.
Usage: python scripts/ncu_hot.py <report> <kernel-regex> [n]"""
import csv
import subprocess
import sys

rep, kre = sys.argv[1], sys.argv[2]
n = int(sys.argv[3]) if len(sys.argv) > 3 else 15
out = subprocess.run(["ncu", "-i", rep, "--page", "source", "--csv", "-k", f"regex:{kre}",
                      "--print-source", "sass"], capture_output=True, text=True).stdout
r = list(csv.reader(out.splitlines()))
hi = next(i for i, x in enumerate(r) if x and x[0] == "Address")
h = r[hi]
rows = [x for x in r[hi + 1:] if len(x) == len(h) and x[0] != "Address"]
si = h.index("Warp Stall Sampling (All Samples)")
cols = [c for c in h if c.startswith("stall_") and "Not Issued" not in c]
def f(v):
    try:
        return float(v)
    except ValueError:
        return 0.0


tot = sum(f(x[si]) for x in rows) or 1
for x in sorted(rows, key=lambda x: -f(x[si]))[:n]:
    d = dict(zip(h, x))
    top = sorted(((f(d[c]), c[6:]) for c in cols), reverse=True)[:2]
    print(f"{f(x[si]) / tot:6.3f}  {x[1].strip()[:70]:70s} {top}")
