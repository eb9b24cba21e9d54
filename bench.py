#!/usr/bin/env python
"""bench.py — CH-benCHmark OLAP hot path on B200 (H2TAP / Caldera data-parallel archipelago).

One STEP = one pass of the whole hot path over the rank's resident snapshot: CH Q6 (fused
scan-filter-sum), CH Q1 (fused scan-filter-group-by) and CH Q18 (hash build, probe +
group-join, HAVING compaction, customer probe, ORDER BY) through the C ABI, each with its
cross-GPU merge when N > 1. Workload = BASELINE.json configs[1]/[2]: W = 100 TPC-C warehouses
per GPU (~30M order_line rows), synthetic ('spread' population, seed 1).

value  = order_line rows processed per second by the step's three queries, whole job
         (3 x visible order_line rows x N / step time), snapshot resident in HBM.
e2e    = same metric through the public API with host buffers: each step refreshes the snapshot
         from pinned host memory (full reload, H2D inside the timed region) and returns every
         result to host memory.
roofline: the dominant kernel's algorithmic bytes per launch / its CUDA-event duration,
         against MEASURED_PEAKS.json hbm_gbs.

Usage: python bench.py [--gpus N --steps K --warmup W] [--impl ours|reference]
       torchrun --nproc-per-node N bench.py --gpus N ...
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import tempfile
import time

import numpy as np

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

import chgen  # noqa: E402

METRIC = "CH-benCHmark Q1/Q6 order_line rows/s & latency; % of HBM BW, 1/2/4/8 B200"
UNIT = "order_line rows/s"
Q6_P = [chgen.ts_us("1999-01-01"), chgen.ts_us("2020-01-01"), 1, 100000]
Q1_P = [chgen.ts_us("2007-01-02")]
Q18_P = [20000]


def parse():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=10)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", choices=["ours", "reference"], default="ours")
    ap.add_argument("--warehouses", type=int, default=100, help="warehouses per GPU (weak scaling)")
    ap.add_argument("--mode", default="spread", choices=["spread", "strict"])
    ap.add_argument("--e2e-steps", type=int, default=None)
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-flush-l2", action="store_true")
    return ap.parse_args()


# ------------------------------------------------------------------ plumbing --
def dist_env():
    rank = int(os.environ.get("RANK", "0"))
    world = int(os.environ.get("WORLD_SIZE", "1"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return rank, world, local


class Clocks:
    """nvidia-smi sampling during the timed region (B200_PROFILING.md clocks line)."""

    def __init__(self, index):
        self.path = tempfile.mktemp(suffix=".csv")
        q = ("index,clocks.sm,clocks.max.sm,power.draw,clocks_event_reasons.active,"
             "clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
             "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap")
        try:
            self.p = subprocess.Popen(["nvidia-smi", f"--id={index}", f"--query-gpu={q}",
                                       "--format=csv,noheader,nounits", "-lms", "20"],
                                      stdout=open(self.path, "w"), stderr=subprocess.DEVNULL)
        except Exception:
            self.p = None

    def stop(self):
        if not self.p:
            return None
        self.p.terminate()
        self.p.wait()
        sm, mx, reasons = [], 0, set()
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        for line in open(self.path):
            f = [x.strip() for x in line.split(",")]
            if len(f) < 9:
                continue
            try:
                sm.append(float(f[1]))
                mx = max(mx, float(f[2]))
            except ValueError:
                continue
            for n, v in zip(names, f[5:9]):
                if v.lower() == "active":
                    reasons.add(n)
        os.unlink(self.path)
        if not sm:
            return None
        return {"sm_mhz": statistics.median(sm), "sm_max_mhz": mx, "reasons": sorted(reasons),
                "samples": len(sm)}


def peaks():
    p = os.path.join(ROOT, "MEASURED_PEAKS.json")
    if os.path.exists(p):
        d = json.load(open(p))
        return float(d["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs: copy, read+write bytes)"
    return 6650.0, "fallback (B200_PROFILING.md 6.65 TB/s)"


def ncu_traffic():
    """Per-launch DRAM bytes of each kernel from the committed ncu --set full capture."""
    p = os.path.join(ROOT, "profiles", "ncu_traffic.json")
    if os.path.exists(p):
        return {k: v for k, v in json.load(open(p)).items() if k != "source"}
    return {}


# ------------------------------------------------------------- algorithmic bytes --
def key_box(t, cols):
    """Slots of the (w, d, id) min/max box: the perfect-hash join index size."""
    n = 1
    for c in cols:
        v = t[c]
        n *= int(v.max()) - int(v.min()) + 1 if len(v) else 0
    return n


def alg_bytes(kernel, n_ol, n_o, n_c, n_pass, sort_passes, box=None):
    """Bytes the method must move per launch. `box`: the
    (orders, customer) key-box slot counts when the planner chose perfect-hash indexes (4-byte
    slots), else None (open addressing: 16-byte slots, capacity pow2 >= 2n)."""
    if box:
        slots_o, slots_c, slot_b = box[0], box[1], 4
    else:
        slots_o = 1 << max(4, int(np.ceil(np.log2(max(2 * n_o, 16)))))
        slots_c = 1 << max(4, int(np.ceil(np.log2(max(2 * n_c, 16)))))
        slot_b = 16
    return {
        "q6_scan_filter_sum": 20 * n_ol,
        "q1_scan_filter_groupby": 24 * n_ol,
        # shared scan of the batch's Q6 and Q1: Q1's 4 columns once, both queries
        "q61_shared_scan": 24 * n_ol,
        "q18_init": slot_b * (slots_o + slots_c),               # empty the join indexes
        # keys in, accumulators zeroed, one slot written per build row
        "q18_build": 12 * n_o + 12 * n_c + 16 * n_o + slot_b * (n_o + n_c),
        # order_line keys + amounts; per order one index slot and the accumulator read + write
        "q18_probe_groupjoin": 20 * n_ol + slot_b * n_o + 16 * n_o + 16 * n_o,
        # acc + orders columns in; per result row a customer slot + c_last lookup, 40 B out
        "q18_having_compact": 16 * n_o + 28 * n_o + (slot_b + 4) * n_pass + 40 * n_pass,
        # ORDER BY v1 (H2TAP_ORDER=v1): (key, row id) sort, random row gather at emit
        "q18_sort_keys_hist": (32 + 8 + 8 + 4) * n_pass,   # rows + amounts -> keys + row ids
        # ORDER BY v2 (default): count matrix + scatter computing keys + chunked local sort
        "q18_sort_hist": 8 * n_pass,                       # amounts (bucket bits inside field a)
        "q18_bucket_scatter": (40 + 16) * n_pass if sort_passes != "v1" else (12 + 12) * n_pass,
        # carry records (v2 default): 16 B record in, 40 B of result columns out (no row gather);
        # row-id paths: pair in + 32 B row gather + 40 B out
        "q18_bucket_sort_emit": (16 + 40) * n_pass if sort_passes == "carry"
                                else (16 if sort_passes == "v2" else 12) * n_pass + (32 + 40) * n_pass,
    }.get(kernel)


# ------------------------------------------------------------------ reference --
def cpu_oracle_sample(w_lo, sample_w, mode):
    """Oracle (single-threaded C, as it stands) on a bounded sample of the same workload."""
    import oracle
    t = chgen.generate(w_lo, w_lo + sample_w, seed=1, mode=mode)
    n = len(t["order_line"]["ol_w_id"])
    t0 = time.perf_counter()
    oracle.q6(t, *Q6_P)
    oracle.q1(t, *Q1_P)
    oracle.q18(t, *Q18_P)
    dt = time.perf_counter() - t0
    return 3 * n / dt, dt, n


def run_reference(a):
    rank, world, _ = dist_env()
    if rank != 0:
        return 0
    import oracle
    oracle.build()
    sample_w = 10
    t = chgen.generate(1, 1 + sample_w, seed=1, mode=a.mode)
    n = len(t["order_line"]["ol_w_id"])
    for _ in range(a.warmup):
        oracle.q6(t, *Q6_P); oracle.q1(t, *Q1_P); oracle.q18(t, *Q18_P)
    t0 = time.perf_counter()
    for _ in range(a.steps):
        oracle.q6(t, *Q6_P); oracle.q1(t, *Q1_P); oracle.q18(t, *Q18_P)
    dt = time.perf_counter() - t0
    value = 3 * n * a.steps / dt
    sample = (f"each step = oracle Q6+Q1+Q18 over W={sample_w} warehouses ({n} order_line rows, "
              f"'{a.mode}', seed 1), single thread")
    print(json.dumps({
        "impl": "reference", "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": a.gpus,
        "steps": a.steps, "warmup": a.warmup, "ms_per_step": dt / a.steps * 1e3,
        "higher_is_better": True, "scaling": "weak", "vs_baseline": None, "dtype": "int64",
        "data": "synthetic", "config": {"workload": f"CH Q6+Q1+Q18 per step, sample W={sample_w}",
                                        "mode": a.mode},
        "cpu_baseline": {"value": value, "unit": UNIT, "cores": 1, "kind": "oracle", "sample": sample},
        "e2e": {"value": value, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }))
    return 0


# ----------------------------------------------------------------------- ours --
def main():
    a = parse()
    if a.impl == "reference":
        return run_reference(a)
    import torch
    import torch.distributed as dist

    rank, world, local = dist_env()
    if world != a.gpus:
        a.gpus = world if world > 1 else a.gpus
    torch.cuda.set_device(local)
    if world > 1:
        dist.init_process_group("nccl", device_id=torch.device("cuda", local))

    import paper_conf_cidr_appuswamykpa17_b200 as h

    # ---- engine + NCCL bootstrap (ncclUniqueId broadcast over the torch process group)
    nccl_id = None
    if world > 1:
        obj = [h.h2tap_nccl_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(obj, src=0)
        nccl_id = obj[0]
    eng = h.h2tap_open(local, rank, world, nccl_id)

    # ---- this rank's warehouse shard (weak scaling: a.warehouses per GPU)
    W = a.warehouses * world
    lo, hi = chgen.warehouse_ranges(W, world)[rank]
    tables = chgen.generate(lo, hi, seed=1, mode=a.mode)
    hot = h.hot_path_tables(tables)
    n_ol = len(tables["order_line"]["ol_w_id"])
    n_o = len(tables["orders"]["o_id"])
    n_c = len(tables["customer"]["c_id"])
    box = (key_box(tables["orders"], ("o_w_id", "o_d_id", "o_id")),
           key_box(tables["customer"], ("c_w_id", "c_d_id", "c_id")))
    pinned = {t: {c: torch.from_numpy(v).pin_memory() for c, v in cols.items()} for t, cols in hot.items()}
    h2d_bytes = sum(v.numel() * v.element_size() for cols in pinned.values() for v in cols.values())
    epoch = 1
    h.h2tap_load_snapshot(eng, pinned, epoch)

    stream = torch.cuda.ExternalStream(h.h2tap_compute_stream(eng))
    flush = None if a.no_flush_l2 else torch.empty(512 << 20, dtype=torch.uint8, device="cuda")
    flush_rd = None if a.no_flush_l2 else torch.ones(256 << 20, dtype=torch.uint8, device="cuda")

    def barrier():
        if world > 1:
            dist.barrier()
        torch.cuda.synchronize()

    plans = (("q6", h.H2TAP_Q6, Q6_P), ("q1", h.H2TAP_Q1, Q1_P), ("q18", h.H2TAP_Q18, Q18_P))

    def step(flags):
        # one batch on the resident snapshot: the three plans run back to back on the GPU and
        # the library synchronises once (h2tap_run_queries)
        rs = h.h2tap_run_queries(eng, [(plan, p, flags) for _, plan, p in plans])
        out = {}
        for (name, _, _), r in zip(plans, rs):
            out[name] = (r.device_ms, r.kernels if flags & h.H2TAP_QUERY_PROFILE else [], r.nrows,
                         r.kernel_launches)
            if name == "q18":
                dense_seen.append(r.plan_flags == 3)  # both join indexes perfect-hash
            h.h2tap_free(r)
        return out

    dense_seen = []

    dev_flags = h.H2TAP_RESULT_DEVICE
    prof_flags = h.H2TAP_RESULT_DEVICE | h.H2TAP_QUERY_PROFILE
    clocks = Clocks(local)  # sampled from warm-up to the end of the instrumented pass
    time.sleep(0.3)
    for _ in range(a.warmup):
        step(dev_flags)
    barrier()

    def flush_l2():
        if flush is not None:
            with torch.cuda.stream(stream):
                flush.add_(1)            # write 512 MB > 126 MB L2 between steps, outside the events,
                flush_rd.sum(dtype=torch.int64)  # then read 256 MB so L2 holds clean lines

    # ---- timed region: K steps, CUDA events on the engine's stream, no per-kernel instrumentation
    starts = [torch.cuda.Event(enable_timing=True) for _ in range(a.steps)]
    ends = [torch.cuda.Event(enable_timing=True) for _ in range(a.steps)]
    per_query = {"q6": [], "q1": [], "q18": []}
    launches = 0
    n_pass = 0
    barrier()
    for i in range(a.steps):
        flush_l2()
        starts[i].record(stream)
        out = step(dev_flags)
        ends[i].record(stream)
        for q, (ms, ks, nrows, nl) in out.items():
            per_query[q].append(ms)
            launches += nl
        n_pass = out["q18"][2]
    barrier()
    step_ms_local = sum(s.elapsed_time(e) for s, e in zip(starts, ends)) / a.steps

    # ---- instrumented pass (same K steps): per-kernel CUDA events for the roofline; a 30 us gate
    # kernel at each query start keeps host launch latency out of every kernel's event window
    kern = {}
    for i in range(a.steps):
        flush_l2()
        out = step(prof_flags)
        for q, (ms, ks, nrows, nl) in out.items():
            for kname, kms in ks:
                kern.setdefault(kname, []).append(kms)
    barrier()
    clk = clocks.stop()
    t = torch.tensor([step_ms_local], dtype=torch.float64, device="cuda")
    if world > 1:
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
    step_ms = float(t.item())
    nt = torch.tensor([n_ol], dtype=torch.float64, device="cuda")
    if world > 1:  # weak scaling: every rank holds its own shard of W warehouses
        dist.all_reduce(nt, op=dist.ReduceOp.SUM)
    rows_total = 3 * int(nt.item())  # order_line rows all ranks scanned, x3 queries
    value = rows_total / (step_ms / 1e3)

    plan_dense = bool(dense_seen) and all(dense_seen)
    # ---- roofline for the dominant kernel (largest share of the step)
    kavg = {k: float(np.mean(v)) for k, v in kern.items()}
    sort_passes = ("v1" if os.environ.get("H2TAP_ORDER") == "v1"
                   else "v2" if os.environ.get("H2TAP_ORDER_CARRY") == "0" else "carry")
    dominant = max(kavg, key=kavg.get) if kavg else None
    peak, peak_src = peaks()
    roof = None
    if dominant:
        b = alg_bytes(dominant, n_ol, n_o, n_c, n_pass, sort_passes, box if plan_dense else None)
        if b:
            ach = b / (kavg[dominant] / 1e3) / 1e9
            tr = ncu_traffic().get(dominant)
            roof = {"bound": "hbm", "kernel": dominant, "achieved": round(ach, 1), "peak": peak,
                    "unit": "GB/s", "frac": round(ach / peak, 4), "traffic": tr,
                    "algorithmic_bytes_per_launch": int(b), "avg_launch_ms": round(kavg[dominant], 5),
                    "share_of_step": round(kavg[dominant] / step_ms_local, 4), "peak_source": peak_src,
                    "timing": "CUDA events on the engine stream, instrumented pass of the same K steps"}
    kernels_summary = {}
    for k, v in kavg.items():
        b = alg_bytes(k, n_ol, n_o, n_c, n_pass, sort_passes, box if plan_dense else None)
        kernels_summary[k] = {"ms": round(v, 5), "share": round(v / step_ms_local, 4)}
        if b:
            kernels_summary[k]["GB/s"] = round(b / (v / 1e3) / 1e9, 1)
            kernels_summary[k]["frac_hbm"] = round(b / (v / 1e3) / 1e9 / peak, 4)

    # ---- e2e: host buffers through the public API (H2D refresh + queries + D2H results)
    e2e_steps = a.e2e_steps or max(5, min(a.steps, 10))
    for _ in range(2):  # warm the reload path (spare buffers) and the host result pool
        epoch += 1
        h.h2tap_load_snapshot(eng, pinned, epoch)
        for r in h.h2tap_run_queries(eng, [(plan, p, 0) for _, plan, p in plans]):
            h.h2tap_free(r)
    barrier()
    d2h = 0
    t0 = time.perf_counter()
    for _ in range(e2e_steps):
        epoch += 1
        h.h2tap_load_snapshot(eng, pinned, epoch)
        d2h = 0
        for r in h.h2tap_run_queries(eng, [(plan, p, 0) for _, plan, p in plans]):
            for c in r.columns.values():
                d2h += c.nbytes
            _ = r.columns[next(iter(r.columns))][:1].sum() if r.nrows else 0  # host read
            h.h2tap_free(r)
    barrier()
    e2e_serial_s = (time.perf_counter() - t0) / e2e_steps
    # pipelined: the same calls with H2TAP_LOAD_ASYNC | H2TAP_LOAD_BORROW (the pinned buffers are
    # lent to the DMA and not modified), so step k's 1.2 GB upload (copy stream)
    # overlaps step k-1's result read-back (D2H, the other PCIe direction) and the queries; each
    # batch runs on the latest PUBLISHED epoch (k or k-1, reported per step) — double buffering
    # (one rank only: with world > 1 the ranks could publish different epochs and a collective
    # query must see one epoch everywhere)
    h.h2tap_sync(eng)
    barrier()
    lag = []
    e2e_pipe_s = float("inf")
    if world == 1:
        for _ in range(3):  # warm-up: grows the device pool to the in-flight snapshot copies
            epoch += 1
            h.h2tap_load_snapshot(eng, pinned, epoch, flags=h.H2TAP_LOAD_ASYNC | h.H2TAP_LOAD_BORROW)
            for r in h.h2tap_run_queries(eng, [(plan, p, 0) for _, plan, p in plans]):
                h.h2tap_free(r)
        h.h2tap_sync(eng)
        t0 = time.perf_counter()
        for _ in range(e2e_steps):
            epoch += 1
            h.h2tap_load_snapshot(eng, pinned, epoch, flags=h.H2TAP_LOAD_ASYNC | h.H2TAP_LOAD_BORROW)
            for r in h.h2tap_run_queries(eng, [(plan, p, 0) for _, plan, p in plans]):
                _ = r.columns[next(iter(r.columns))][:1].sum() if r.nrows else 0  # host read
                lag.append(epoch - r.epoch)
                h.h2tap_free(r)
        h.h2tap_sync(eng)  # the last upload is inside the timed region too
        e2e_pipe_s = (time.perf_counter() - t0) / e2e_steps
    barrier()
    te = torch.tensor([e2e_serial_s, e2e_pipe_s], dtype=torch.float64, device="cuda")
    if world > 1:
        dist.all_reduce(te, op=dist.ReduceOp.MAX)
    e2e_serial_s, e2e_pipe_s = (float(x) for x in te.tolist())
    e2e_s = min(e2e_serial_s, e2e_pipe_s)

    # ---- CPU oracle baseline (rank 0, N = 1 only, bounded sample)
    cpu = None
    if rank == 0 and world == 1 and not a.no_cpu_baseline:
        sample_w = 20
        v, dt, n = cpu_oracle_sample(lo, sample_w, a.mode)
        cpu = {"value": v, "unit": UNIT, "cores": 1, "kind": "oracle",
               "sample": f"oracle Q6+Q1+Q18 once over W={sample_w} of the same warehouses "
                         f"({n} order_line rows, {dt:.1f} s, single thread)"}

    if rank == 0:
        line = {
            "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": a.steps,
            "warmup": a.warmup, "ms_per_step": step_ms, "higher_is_better": True,
            "scaling": "weak", "vs_baseline": None, "dtype": "int64", "data": "synthetic",
            "config": {"workload": f"CH Q6+Q1+Q18 per step over W={a.warehouses} warehouses per GPU "
                                   f"('{a.mode}' TPC-C population, seed 1)",
                       "warehouses_per_gpu": a.warehouses, "order_line_rows_per_gpu": n_ol,
                       "orders_rows_per_gpu": n_o, "customer_rows_per_gpu": n_c,
                       "queries_per_step": 3, "parallelism": f"row-sharded by warehouse x{world}",
                       "scan_sharing": ("Q6 and Q1 of the batch share one pass over order_line "
                                        "(latency_ms q6 includes it, q1 is its finalize; DESIGN.md "
                                        "§4.5); every query computes its full result"
                                        if os.environ.get("H2TAP_SHARED_SCAN", "1") != "0" else "off"),
                       "l2": ("inputs > L2; between steps (outside events) 512 MB written then 256 MB read to flush L2"
                              if flush is not None else "inputs > L2 (no flush)")},
            "latency_ms": {q: round(float(np.median(v)), 4) for q, v in per_query.items()},
            "rows_per_s": {q: rows_total / 3 / (float(np.median(v)) / 1e3) for q, v in per_query.items()},
            "q18_result_rows": n_pass,
            "roofline": roof,
            "kernels": kernels_summary,
            "cpu_baseline": cpu,
            "e2e": {"value": rows_total / e2e_s, "unit": UNIT, "h2d_bytes_per_step": int(h2d_bytes),
                    "d2h_bytes_per_step": int(d2h), "ms_per_step": e2e_s * 1e3, "steps": e2e_steps,
                    "mode": "pipelined" if e2e_pipe_s <= e2e_serial_s else "serial",
                    "serial_ms_per_step": e2e_serial_s * 1e3,
                    "pipelined_ms_per_step": e2e_pipe_s * 1e3 if world == 1 else None,
                    "pipelined_epoch_lag": sorted(set(lag)),
                    "how": "every step: full snapshot upload of the step's inputs from pinned host "
                           "buffers (h2tap_load_snapshot) + Q6/Q1/Q18 batch (h2tap_run_queries) + "
                           "results copied to host; serial = load then queries; pipelined = "
                           "H2TAP_LOAD_ASYNC|H2TAP_LOAD_BORROW, queries on the latest published "
                           "epoch (lag in epochs listed)"},
            "gpu_launches": int(launches),
            "clocks": clk,
        }
        print(json.dumps(line))
    h.h2tap_close(eng)
    if world > 1:
        dist.destroy_process_group()
    return 0


if __name__ == "__main__":
    sys.exit(main())
