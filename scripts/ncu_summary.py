"""Summarise an ncu launch list (--metrics gpu__time_duration.sum csv) and a --set full report
into a markdown table under profiles/. Usage: python scripts/ncu_summary.py <tag>"""
import collections
import csv
import json
import os
import subprocess
import sys

tag = sys.argv[1]
root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
out = []
lp = os.path.join(root, "gpurun_out", f"launches_{tag}.csv")
if os.path.exists(lp):
    rows = list(csv.reader(open(lp)))
    hdr = next(i for i, r in enumerate(rows) if "Kernel Name" in r)
    H = rows[hdr]
    ki, vi = H.index("Kernel Name"), H.index("Metric Value")
    agg = collections.OrderedDict()
    for r in rows[hdr + 1:]:
        if len(r) > vi:
            agg.setdefault(r[ki].split("(")[0].split("::")[-1], []).append(float(r[vi].replace(",", "")))
    tot = sum(sum(v) for v in agg.values())
    out.append(f"## Launch list ({lp.split('/')[-1]}, ncu gpu__time_duration.sum, cold cache, serialised)\n")
    out.append("| kernel | launches | mean us | share of listed time |\n|---|---|---|---|")
    for k, v in agg.items():
        out.append(f"| {k} | {len(v)} | {sum(v)/len(v)/1e3:.1f} | {sum(v)/tot:.3f} |")
rp = os.path.join(root, "gpurun_out", f"prof_{tag}.ncu-rep")
traffic = {}
if os.path.exists(rp):
    raw = subprocess.run(["ncu", "-i", rp, "--page", "raw", "--csv"], capture_output=True, text=True).stdout
    r = list(csv.reader(raw.splitlines()))
    h = r[0]
    want = ["Kernel Name", "gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
            "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed",
            "sm__throughput.avg.pct_of_peak_sustained_elapsed", "launch__registers_per_thread",
            "sm__warps_active.avg.pct_of_peak_sustained_active", "lts__t_sector_hit_rate.pct",
            # SURVEY.md §8(d) timing protocol's list: shared atomics, global load sectors, issue
            "smsp__inst_executed_op_shared_atom.sum", "l1tex__t_sectors_pipe_lsu_mem_global_op_ld.sum",
            "smsp__issue_active.avg.pct_of_peak_sustained_active", "smsp__inst_executed.sum"]
    idx = [h.index(w) for w in want if w in h]
    out.append(f"\n## ncu --set full ({rp.split('/')[-1]})\n")
    out.append("| " + " | ".join(h[i] for i in idx) + " |")
    out.append("|" + "---|" * len(idx))
    out.append("| " + " | ".join(r[1][i] for i in idx) + " |")
    unit = {h[i]: r[1][i] for i in idx}
    for row in r[2:]:
        name = row[h.index("Kernel Name")].split("(")[0].split("::")[-1]
        out.append("| " + " | ".join([name] + [row[i] for i in idx[1:]]) + " |")
        mult = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}
        rd = float(row[h.index("dram__bytes_read.sum")]) * mult[unit["dram__bytes_read.sum"]]
        wr = float(row[h.index("dram__bytes_write.sum")]) * mult[unit["dram__bytes_write.sum"]]
        traffic.setdefault(name, []).append(rd + wr)
md = os.path.join(root, "profiles", f"{tag}_ncu_summary.md")
open(md, "w").write(f"# ncu summary {tag}\n\n" + "\n".join(out) + "\n")
print(open(md).read())
if traffic:
    tj = os.path.join(root, "profiles", f"{tag}_traffic.json")
    per = {k: sum(v) / len(v) for k, v in traffic.items()}
    json.dump(per, open(tj, "w"), indent=1)
    # per-launch DRAM bytes keyed by the engine's profile marks (what bench.py reports)
    marks = {"q6_kernel": "q6_scan_filter_sum", "q1_kernel": "q1_scan_filter_groupby",
             "q6_tma_kernel": "q6_scan_filter_sum", "q1_tma_kernel": "q1_scan_filter_groupby",
             "q18_probe_tma_kernel": "q18_probe_groupjoin",
             "q18_init_kernel": "q18_init", "q18_build_kernel": "q18_build",
             "q18_probe_kernel": "q18_probe_groupjoin", "q18_having_kernel": "q18_having_compact",
             "q18_keys_hist_kernel": "q18_sort_keys_hist", "bucket_scatter_kernel": "q18_bucket_scatter",
             "bucket_local_emit_kernel<2048, 0>": "q18_bucket_sort_emit",
             "bucket_local_emit_kernel<8192, 2048>": "q18_bucket_sort_emit_large",
             "ob_hist_kernel": "q18_sort_hist", "ob_scan_kernel": "q18_sort_scan",
             "ob_scatter_kernel": "q18_bucket_scatter", "ob_local_emit_kernel<2048, 0>": "q18_bucket_sort_emit",
             "ob_local_emit_kernel<8192, 2048>": "q18_bucket_sort_emit_large",
             "q18_probe_kernel<0>": "q18_probe_groupjoin", "q18_having_kernel<2>": "q18_having_compact",
             "bucket_local_emit_kernel<2048, 0, 1>": "q18_bucket_sort_emit",
             "bucket_local_emit_kernel<8192, 2048, 1>": "q18_bucket_sort_emit_large",
             "q18_plan_kernel": "q18_plan", "q1_compact_kernel": "q1_compact",
             "q1_emit_kernel": "q1_emit", "q1_tma_kernel<1>": "q61_shared_scan",
             "q1_tma_kernel<1, 0>": "q61_shared_scan", "q1_tma_kernel<1, 1>": "q6118_full_pass",
             "q18_acc_stats_kernel": "q18_acc_stats", "q18_having_rec_kernel": "q18_having_records",
             "q18_having_rec_kernel<1>": "q18_having_records", "q18_having_rec_kernel<0>": "q18_having_records",
             "q18_acc_hist_kernel": "q18_bucket_count", "q18_plan_hist_kernel": "q18_plan_count",
             "ob_scatter_rec_kernel": "q18_bucket_scatter",
             "bucket_local_emit_kernel<1536, 0, 1>": "q18_bucket_sort_emit",
             "bucket_local_emit_kernel<8192, 1536, 1>": "q18_bucket_sort_emit_large"}
    bymark = {}
    for k, v in per.items():
        m = marks.get(k)
        if m:
            bymark[m] = bymark.get(m, 0.0) + v
    if len(sys.argv) > 2 and sys.argv[2] == "--bench":
        json.dump({"source": f"profiles/{tag}_ncu_summary.md (ncu --set full, per launch, dram read + write)",
                   **{k: int(v) for k, v in bymark.items()}},
                  open(os.path.join(root, "profiles", "ncu_traffic.json"), "w"), indent=1)
