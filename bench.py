#!/usr/bin/env python
"""bench.py — CH-benCHmark OLAP hot path on B200 (H2TAP / Caldera data-parallel archipelago).

One STEP = one pass of the whole hot path over the rank's resident snapshot: CH Q6 (fused
scan-filter-sum), CH Q1 (fused scan-filter-group-by) and CH Q18 (hash build, probe +
group-join, HAVING compaction, customer probe, ORDER BY) through the C ABI, each with its
cross-GPU merge when N > 1. Workload = BASELINE.json configs[1]/[2]: W = 100 TPC-C warehouses
per GPU (~30M order_line rows), synthetic ('spread' population, seed 1).

value  = order_line rows per second through one full pass of the hot path, whole job: every
         rank's visible order_line rows (each counted ONCE per step, although Q6, Q1 and Q18 all
         read them) / step time (max over ranks), snapshot resident in HBM. Step time = the
         batch's GPU span from the library's CUDA events on its stream (h2tap_last_batch_ms:
         before the first kernel, after the last); ms_per_step_host_return adds the host's
         wake-up and return path (the bench's own events around the synchronous call).
e2e    = same metric through the public API with host buffers: each step refreshes the snapshot
         from pinned host memory (full reload, H2D inside the timed region), runs the batch and
         returns every result to host memory; the serial figure (queries read that step's upload).
         e2e_incremental: the snapshot stays resident, each step refreshes it with that step's
         NewOrder appends + Delivery updates only (the paper's fresh-snapshot loop).
roofline: the dominant kernel's algorithmic bytes per launch / its CUDA-event duration,
         against MEASURED_PEAKS.json hbm_gbs (copy) and the live read-stream peak.
c1     = BASELINE configs[0]: Q6 at W=1 on one GPU, device and e2e latency, oracle beside it.

Usage: python bench.py [--gpus N --steps K --warmup W] [--impl ours|reference]
       [--total-warehouses T]   (strong scaling: T warehouses split over the N GPUs, config C4)
With --gpus N > 1 and no torchrun environment, bench.py launches its N ranks itself
(torch.distributed.run, 127.0.0.1); under torchrun WORLD_SIZE must equal --gpus.
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
    ap.add_argument("--total-warehouses", type=int, default=None,
                    help="strong scaling: this many warehouses split over the GPUs (config C4)")
    ap.add_argument("--peer-heap-mb", type=int, default=0, help="world > 1: peer heap per rank (0 = 1 GiB)")
    ap.add_argument("--no-c1", action="store_true", help="skip the config C1 line (Q6 at W=1)")
    ap.add_argument("--share-device", action="store_true",
                    help="functional check of the N-rank path on ONE GPU: every rank on cuda:0 (CUDA IPC between "
                         "the processes), gloo for the plumbing; timings meaningless, never a bench line")
    ap.add_argument("--sleep-cycles", type=int, default=200_000,
                    help="sleep kernel queued before each timed step (the host enqueues meanwhile)")
    ap.add_argument("--plans", default="q6,q1,q18",
                    help="the step's queries (config C4 is Q1 + Q6: --plans q6,q1)")
    ap.add_argument("--mode", default="spread", choices=["spread", "strict"])
    ap.add_argument("--e2e-steps", type=int, default=None)
    ap.add_argument("--inc-neworders", type=int, default=10_000,
                    help="e2e_incremental: NewOrder transactions appended per step and GPU (0: skip)")
    ap.add_argument("--inc-deliveries", type=int, default=1_000,
                    help="e2e_incremental: Delivery transactions (10 orders each) per step and GPU")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-flush-l2", action="store_true")
    return ap.parse_args()


# ------------------------------------------------------------------ plumbing --
def dist_env():
    rank = int(os.environ.get("RANK", "0"))
    world = int(os.environ.get("WORLD_SIZE", "1"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    return rank, world, local


def spawn_ranks(a):
    """--gpus N > 1 outside torchrun: launch the N ranks here (one process per GPU)."""
    import socket
    import torch
    have = torch.cuda.device_count()
    if have < a.gpus and not (a.share_device and have >= 1):
        print(json.dumps({"error": f"--gpus {a.gpus} but {have} CUDA device(s) visible"}), flush=True)
        return 2
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    cmd = [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={a.gpus}",
           "--master-addr=127.0.0.1", f"--master-port={port}", os.path.abspath(__file__)] + sys.argv[1:]
    return subprocess.call(cmd)


def host_cpu():
    model = "unknown"
    try:
        for line in open("/proc/cpuinfo"):
            if line.startswith("model name"):
                model = line.split(":", 1)[1].strip()
                break
    except OSError:
        pass
    return {"nproc": os.cpu_count(), "cpu_model": model}


class pinned_core:
    """Run the oracle on one host core (taskset -c 1 equivalent: sched_setaffinity)."""

    def __init__(self, core=1):
        self.core = core
        self.old = None

    def __enter__(self):
        try:
            self.old = os.sched_getaffinity(0)
            core = self.core if self.core in self.old else min(self.old)
            os.sched_setaffinity(0, {core})
            self.used = core
        except (AttributeError, OSError):
            self.used = None
        return self

    def __exit__(self, *exc):
        if self.old:
            os.sched_setaffinity(0, self.old)


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


def alg_bytes(kernel, n_ol, n_o, n_c, n_pass, sort_passes, box=None, clustered=False):
    """Bytes the method must move per launch. `box`: the
    (orders, customer) key-box slot counts when the planner chose perfect-hash indexes (4-byte
    slots), else None (open addressing: 16-byte slots, capacity pow2 >= 2n). `clustered`: both
    build sides verified in key order, indexes positional: the verify pass reads
    the keys and zeroes the accumulators, nothing is built, no slot is read."""
    if clustered:
        return {"q61_shared_scan": 24 * n_ol, "q6_scan_filter_sum": 20 * n_ol, "q1_scan_filter_groupby": 24 * n_ol,
                # the batch's full pass: Q1's 4 columns + Q18's 3 keys once, the probe's
                # accumulator read + write per order
                "q6118_full_pass": 36 * n_ol + 16 * n_o + 16 * n_o,
                "q18_init": 12 * (n_o + n_c) + 16 * n_o,            # verify: keys in, acc zeroed
                "q18_probe_groupjoin": 20 * n_ol + 16 * n_o + 16 * n_o,
                # one GPU: o_entry_d's bounds come from the snapshot's zone map, acc[] alone is read
                "q18_acc_stats": 16 * n_o,
                "q18_having_records": 16 * n_o + 12 * n_o + (4 + 16 + 16) * n_pass,
                "q18_bucket_scatter": (16 + 16) * n_pass,
                # direct ORDER BY (default): bucket counts from the accumulators alone
                "q18_bucket_count": 16 * n_o,
                "q18_plan_count": 16 * n_o,  # plan + counts in one kernel: acc[] once (L2 re-read)
                "q18_bucket_sort_emit": (16 + 40) * n_pass}.get(kernel)
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
        # full pass: + Q18's keys; per order one index slot and the accumulator read + write
        "q6118_full_pass": 36 * n_ol + slot_b * n_o + 16 * n_o + 16 * n_o,
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
        "q18_bucket_count": 16 * n_o,                      # direct ORDER BY: counts from acc[]
        "q18_plan_count": 16 * n_o,                        # plan + counts, one kernel
        "q18_bucket_scatter": (16 + 16) * n_pass if sort_passes == "carry"
                              else (40 + 16) * n_pass if sort_passes != "v1" else (12 + 12) * n_pass,
        # v3 (default): the accumulators for the plan's amount bounds (o_entry_d: zone map)
        "q18_acc_stats": 16 * n_o,
        # v3: acc + orders keys in, per result row a customer slot + c_last + (o_id, o_ol_cnt,
        # o_entry_d) and the 16 B carry record out
        "q18_having_records": 16 * n_o + 12 * n_o + (slot_b + 4 + 16 + 16) * n_pass,
        # carry records (v2 default): 16 B record in, 40 B of result columns out (no row gather);
        # row-id paths: pair in + 32 B row gather + 40 B out
        "q18_bucket_sort_emit": (16 + 40) * n_pass if sort_passes == "carry"
                                else (16 if sort_passes == "v2" else 12) * n_pass + (32 + 40) * n_pass,
    }.get(kernel)


# ------------------------------------------------------------------ reference --
def incremental_inputs(h, tables, lo, hi, n_steps, n_neworder, n_delivery):
    """The per-step inputs of ``e2e_incremental``: TPC-C NewOrder appends (``chgen.neworder_batch``)
    plus Delivery row updates (``chgen.delivery_batch``: ol_delivery_d of the delivered orders'
    lines; o_carrier_id and the new_order DELETE touch no hot-path column) for ``n_steps`` epochs,
    generated before the timed region into pinned host buffers. Returns ([(delta, updates,
    first_row, h2d_bytes)], final order_line rows, final orders rows, rows per step)."""
    import torch

    def pin(a):
        a = np.ascontiguousarray(a)
        if a.dtype == np.uint32:
            a = a.view(np.int32)
        return torch.from_numpy(a).pin_memory()
    item = tables.get("item") or chgen.generate_item(1)
    no_state = chgen.NewOrderState(lo, hi)
    dl = chgen.DeliveryState()
    dl.add(tables["orders"], 0, 0)
    n_o, n_ol = len(tables["orders"]["o_id"]), len(tables["order_line"]["ol_o_id"])
    clock = chgen.TS_2025 + 30 * chgen.DAY_US
    hot_cols = {}
    for plan in h.HOT_PATH_PLANS:
        for t, cols in h.plan_columns()[plan].items():
            hot_cols.setdefault(t, set()).update(cols)
    out, rows = [], []
    for b in range(n_steps):
        d = chgen.neworder_batch(no_state, n_neworder, seed=1, batch=1000 + b, item=item)
        dl.add(d["orders"], n_o, n_ol)
        w, carrier = chgen.delivery_inputs(n_delivery, seed=1, batch=1000 + b, w_lo=lo, w_hi=hi)
        upd = chgen.delivery_batch(dl, w, carrier, clock)
        clock += (n_delivery + 1) * 1000
        delta = {t: {c: pin(v) for c, v in cols.items() if c in hot_cols.get(t, ())}
                 for t, cols in d.items() if t in hot_cols}
        updates = {t: {c: (pin(r), pin(v)) for c, (r, v) in cols.items() if c in hot_cols.get(t, ())}
                   for t, cols in upd.items() if t in hot_cols}
        updates = {t: c for t, c in updates.items() if c}
        nbytes = sum(v.numel() * v.element_size() for cols in delta.values() for v in cols.values())
        nbytes += sum(x.numel() * x.element_size() for cols in updates.values() for p in cols.values() for x in p)
        out.append((delta, updates, {"orders": n_o, "order_line": n_ol}, nbytes))
        n_o += len(d["orders"]["o_id"])
        n_ol += len(d["order_line"]["ol_o_id"])
        rows.append(n_ol)
    return out, n_ol, n_o, rows


def cpu_oracle_steps(t, min_s=10.0, max_reps=4):
    """The oracle (single-threaded C, as it stands, one pinned core) running the bench's step —
    Q6 + Q1 + Q18 over the rank's whole table set — repeated until about min_s seconds of CPU work
    (at most max_reps steps): rows/s of the median step."""
    import oracle
    n = len(t["order_line"]["ol_w_id"])
    dts = []
    with pinned_core(1) as pc:
        while len(dts) < max_reps and sum(dts) < min_s:
            t0 = time.perf_counter()
            oracle.q6(t, *Q6_P)
            oracle.q1(t, *Q1_P)
            oracle.q18(t, *Q18_P)
            dts.append(time.perf_counter() - t0)
    dt = float(np.median(dts))
    return n / dt, dt, n, pc.used, len(dts), sum(dts)


def workload_name(a, world):
    """The `config.workload` string of a run (both arms print the same one)."""
    qs = "+".join(x.strip().upper() for x in a.plans.split(",") if x.strip())
    if a.total_warehouses is not None:
        w = f"CH {qs} per step over W={a.total_warehouses} warehouses split over {world} GPU(s)"
    else:
        w = f"CH {qs} per step over W={a.warehouses} warehouses per GPU"
    return w + f" ('{a.mode}' TPC-C population, seed 1)"


def rows_counted(a):
    qs = " + ".join(x.strip().upper() for x in a.plans.split(",") if x.strip())
    return f"each visible order_line row counted once per step; one step = CH {qs} over the snapshot"


def run_reference(a):
    rank, world, _ = dist_env()
    if rank != 0:
        return 0
    import oracle
    oracle.build()
    sample_w = 10
    t = chgen.generate(1, 1 + sample_w, seed=1, mode=a.mode)
    n = len(t["order_line"]["ol_w_id"])
    want = [x.strip() for x in a.plans.split(",") if x.strip()]
    fns = [f for q, f in (("q6", lambda: oracle.q6(t, *Q6_P)), ("q1", lambda: oracle.q1(t, *Q1_P)),
                          ("q18", lambda: oracle.q18(t, *Q18_P))) if q in want]
    with pinned_core(1) as pc:
        for _ in range(a.warmup):
            for f in fns:
                f()
        t0 = time.perf_counter()
        for _ in range(a.steps):
            for f in fns:
                f()
        dt = time.perf_counter() - t0
    value = n * a.steps / dt
    sample = (f"each step = oracle {'+'.join(q.upper() for q in want)} over W={sample_w} warehouses ({n} order_line rows, "
              f"'{a.mode}', seed 1), single thread pinned to core {pc.used}")
    print(json.dumps({
        "impl": "reference", "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": a.gpus,
        "steps": a.steps, "warmup": a.warmup, "ms_per_step": dt / a.steps * 1e3,
        "higher_is_better": True, "scaling": "weak", "vs_baseline": None, "dtype": "int64",
        "data": "synthetic", "config": {"workload": workload_name(a, a.gpus), "rows_counted": rows_counted(a),
                                        "reference_sample": f"W={sample_w} of the workload's warehouses per "
                                                            "step (rows/s is size-independent for the "
                                                            "row-at-a-time oracle)"},
        "cpu_baseline": dict({"value": value, "unit": UNIT, "cores": 1, "kind": "oracle", "sample": sample,
                              "pinned_core": pc.used}, **host_cpu()),
        "e2e": {"value": value, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }))
    return 0



# ----------------------------------------------------------------------- ours --
def event_ms(stream, fn, reps, flush=None):
    """Median CUDA-event time of fn() on `stream` over `reps` runs (L2 flushed before each)."""
    import torch
    out = []
    for _ in range(reps):
        if flush:
            flush()
        a, b = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        a.record(stream)
        fn()
        b.record(stream)
        b.synchronize()
        out.append(a.elapsed_time(b))
    return float(np.median(out))


def read_stream_peak(h, eng, stream):
    """Live read-only HBM stream rate: the library's DSM layout kernel (one int32 column, pure
    coalesced reads, NEXT-3) over 4 GiB — the read ceiling next to the copy peak of MEASURED_PEAKS."""
    import torch
    n = 1 << 30
    col = torch.ones(n, dtype=torch.int32, device="cuda")
    torch.cuda.synchronize()
    best = 0.0
    for _ in range(5):
        _, ms = h.h2tap_layout_sum(eng, col, h.H2TAP_DSM, n, 1, [0])
        best = max(best, 4.0 * n / (ms / 1e3) / 1e9)
    del col
    torch.cuda.empty_cache()
    return round(best, 1)


def c1_line(h, a):
    """BASELINE configs[0]: CH Q6 at W=1 (~300 k order_line rows, 6 MB) on one GPU vs the oracle:
    device latency (CUDA events around the query on the resident snapshot), e2e latency (the W=1
    Q6 columns uploaded from pinned host memory + the query + the result on the host) and the
    oracle's latency on one pinned host core, medians."""
    import torch
    import oracle
    t = chgen.generate(1, 2, seed=1, mode=a.mode)
    n = len(t["order_line"]["ol_w_id"])
    cols = {"order_line": {c: torch.from_numpy(t["order_line"][c]).pin_memory()
                           for c in ("ol_delivery_d", "ol_quantity", "ol_amount")}}
    e = h.h2tap_open(0)
    try:
        h.h2tap_load_snapshot(e, cols, 1)
        stream = torch.cuda.ExternalStream(h.h2tap_compute_stream(e))
        got = None

        own = []

        def q():
            nonlocal got
            r = h.h2tap_run_query(e, h.H2TAP_Q6, Q6_P, flags=h.H2TAP_RESULT_DEVICE)
            got = r.nrows
            own.append(r.device_ms)  # the query's own CUDA events around its kernels
            h.h2tap_free(r)
        for _ in range(20):
            q()
        own.clear()
        dev_ms = event_ms(stream, q, 100)  # events around the host call: launch latency included
        own_ms = float(np.median(own))
        epoch = [1]

        def e2e():
            epoch[0] += 1
            h.h2tap_load_snapshot(e, cols, epoch[0])
            r = h.h2tap_run_query(e, h.H2TAP_Q6, Q6_P)
            v = r.to_numpy()
            h.h2tap_free(r)
            return v
        for _ in range(5):
            res = e2e()
        e2e_ms = []
        for _ in range(50):
            t0 = time.perf_counter()
            res = e2e()
            e2e_ms.append((time.perf_counter() - t0) * 1e3)
        want = oracle.q6(t, *Q6_P)
        assert int(res["revenue"][0]) == want["revenue"] and int(res["count_rows"][0]) == want["count"]
        # zero-copy (NEXT-4, the paper's UVA design): the columns stay in pinned host memory, a new
        # epoch publishes them without a copy and the query's kernel reads them over PCIe
        zc_cols = h.pinned_tables({"order_line": {c: t["order_line"][c]
                                                  for c in ("ol_delivery_d", "ol_quantity", "ol_amount")}})

        def e2e_zc():
            epoch[0] += 1
            h.h2tap_load_snapshot(e, zc_cols, epoch[0], flags=h.H2TAP_LOAD_ZERO_COPY)
            r = h.h2tap_run_query(e, h.H2TAP_Q6, Q6_P)
            v = r.to_numpy()
            h.h2tap_free(r)
            return v
        for _ in range(5):
            res = e2e_zc()
        zc_ms = []
        for _ in range(50):
            t0 = time.perf_counter()
            res = e2e_zc()
            zc_ms.append((time.perf_counter() - t0) * 1e3)
        assert int(res["revenue"][0]) == want["revenue"] and int(res["count_rows"][0]) == want["count"]
        ora = []
        with pinned_core(1) as pc:
            for _ in range(5):
                t0 = time.perf_counter()
                oracle.q6(t, *Q6_P)
                ora.append((time.perf_counter() - t0) * 1e3)
        dev, ee, om = own_ms, float(np.median(e2e_ms)), float(np.median(ora))
        zz = float(np.median(zc_ms))
        return {"workload": "CH Q6 at W=1 (BASELINE configs[0]), 1 GPU, parity vs the oracle checked",
                "order_line_rows": n, "device_ms": round(dev, 4), "device_rows_per_s": n / (dev / 1e3),
                "device_how": "the query's own CUDA events around its kernels (result.device_ms), median of 100",
                "call_ms": round(dev_ms, 4),
                "call_how": "CUDA events on the engine stream around the synchronous h2tap_run_query call "
                            "(host launch latency inside), median of 100",
                "e2e_zero_copy_ms": round(zz, 4), "e2e_zero_copy_rows_per_s": n / (zz / 1e3),
                "e2e_zero_copy_how": "per run: the 3 Q6 columns published in place from pinned host memory "
                                     "(H2TAP_LOAD_ZERO_COPY, no copy) + h2tap_run_query reading them over "
                                     "PCIe + result on the host; host wall clock, median of 50",
                "e2e_ms": round(ee, 4), "e2e_rows_per_s": n / (ee / 1e3),
                "e2e_how": "per run: full reload of the 3 Q6 columns (6 MB) from pinned host memory + "
                           "h2tap_run_query + result on the host; host wall clock, median of 50",
                "oracle_ms": round(om, 3), "oracle_rows_per_s": n / (om / 1e3), "oracle_cores": 1,
                "oracle_pinned_core": pc.used,
                "note": "6 MB is L2-resident and launch-bound; % of HBM is not meaningful here"}
    finally:
        h.h2tap_close(e)


def main():
    a = parse()
    if a.impl == "reference":
        return run_reference(a)
    rank, world, local = dist_env()
    if "WORLD_SIZE" not in os.environ and a.gpus > 1:
        return spawn_ranks(a)
    if world != a.gpus:
        print(json.dumps({"error": f"WORLD_SIZE={world} but --gpus {a.gpus}"}), flush=True)
        return 2
    import torch
    import torch.distributed as dist

    if a.share_device:
        local = 0
    torch.cuda.set_device(local)
    pg_dev = "cpu" if a.share_device else "cuda"  # gloo reduces host tensors, NCCL device tensors
    if world > 1:  # plumbing only: peer-handle exchange, barriers, max-over-ranks timing
        if a.share_device:
            dist.init_process_group("gloo")
        else:
            dist.init_process_group("nccl", device_id=torch.device("cuda", local))

    import paper_conf_cidr_appuswamykpa17_b200 as h

    eng = h.h2tap_open(local, rank, world, a.peer_heap_mb << 20)
    if world > 1:
        h.connect_torch_group(eng)

    # ---- this rank's warehouse shard: weak scaling (a.warehouses per GPU) or strong (C4)
    strong = a.total_warehouses is not None
    W = a.total_warehouses if strong else a.warehouses * world
    lo, hi = chgen.warehouse_ranges(W, world)[rank]
    tables = chgen.generate(lo, hi, seed=1, mode=a.mode)
    hot = h.hot_path_tables(tables)
    n_ol = len(tables["order_line"]["ol_w_id"])
    n_o = len(tables["orders"]["o_id"])
    n_c = len(tables["customer"]["c_id"])
    box = (key_box(tables["orders"], ("o_w_id", "o_d_id", "o_id")),
           key_box(tables["customer"], ("c_w_id", "c_d_id", "c_id")))
    e2e_steps = a.e2e_steps or max(5, min(a.steps, 10))
    inc = None
    if a.inc_neworders > 0:  # generated before any timing; tables are dropped right after
        # two runs of 2 + K steps each (serial, then pipelined), one continuous OLTP history
        inc = incremental_inputs(h, tables, lo, hi, 2 * (2 + e2e_steps), a.inc_neworders, a.inc_deliveries)
    del tables
    pinned = {t: {c: torch.from_numpy(v).pin_memory() for c, v in cols.items()} for t, cols in hot.items()}
    del hot
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

    def max_over_ranks(vals):
        t = torch.tensor(vals, dtype=torch.float64, device=pg_dev)
        if world > 1:
            dist.all_reduce(t, op=dist.ReduceOp.MAX)
        return [float(x) for x in t.tolist()]

    want = [x.strip() for x in a.plans.split(",") if x.strip()]
    plans = tuple(p for p in (("q6", h.H2TAP_Q6, Q6_P), ("q1", h.H2TAP_Q1, Q1_P), ("q18", h.H2TAP_Q18, Q18_P))
                  if p[0] in want)

    def run_batch(sel, flags, end_event=None):
        rs = h.h2tap_run_queries(eng, [(plan, p, flags) for name, plan, p in plans if name in sel])
        if end_event is not None:  # right after the call returns (the batch is complete on the
            end_event.record(stream)  # device): the Python bookkeeping below stays outside
        out = {}
        for name, r in zip([n for n, _, _ in plans if n in sel], rs):
            out[name] = (r.device_ms, r.kernels if flags & h.H2TAP_QUERY_PROFILE else [], r.nrows,
                         r.kernel_launches, r.total_rows)
            if name == "q18":
                dense_seen.append(r.plan_flags & 3 == 3)  # both join indexes perfect-hash
                clustered_seen.append(r.plan_flags >> 3 == 3)  # ... and positional (§4.3)
            h.h2tap_free(r)
        return out

    dense_seen, clustered_seen = [], []
    dev_flags = h.H2TAP_RESULT_DEVICE
    prof_flags = h.H2TAP_RESULT_DEVICE | h.H2TAP_QUERY_PROFILE
    ALL = tuple(p[0] for p in plans)
    clocks = Clocks(local)  # sampled from warm-up to the end of the instrumented pass
    time.sleep(0.3)
    for _ in range(a.warmup):
        run_batch(ALL, dev_flags)
    barrier()

    def flush_l2():
        if flush is not None:
            with torch.cuda.stream(stream):
                flush.add_(1)            # write 512 MB > 126 MB L2 between steps, outside the events,
                flush_rd.sum(dtype=torch.int64)  # then read 256 MB so L2 holds clean lines

    # ---- timed region: K steps, CUDA events on the engine's stream, no per-kernel instrumentation
    starts = [torch.cuda.Event(enable_timing=True) for _ in range(a.steps)]
    ends = [torch.cuda.Event(enable_timing=True) for _ in range(a.steps)]
    per_query = {q: [] for q in ALL}
    batch_dev = []  # the library's own events around each batch's GPU work (h2tap_last_batch_ms)
    launches = 0
    n_pass = n_pass_total = 0
    barrier()
    for i in range(a.steps):
        flush_l2()
        with torch.cuda.stream(stream):  # ~50 us sleep outside the events: the host enqueues the
            torch.cuda._sleep(a.sleep_cycles)  # batch while the GPU sleeps (no launch gap inside)
        starts[i].record(stream)
        out = run_batch(ALL, dev_flags, ends[i])
        batch_dev.append(h.h2tap_last_batch_ms(eng))
        for q, (ms, ks, nrows, nl, tot) in out.items():
            per_query[q].append(ms)
            launches += nl
        if "q18" in out:
            n_pass, n_pass_total = out["q18"][2], out["q18"][4]
    barrier()
    # the step = the batch's GPU span: CUDA events on the engine stream before its first kernel and
    # after its last (h2tap_last_batch_ms); the bench's own events around the call (end recorded
    # when the synchronous call has returned to Python) add the host's wake-up + return path and
    # are reported next to it
    step_host_ms_local = sum(s.elapsed_time(e) for s, e in zip(starts, ends)) / a.steps
    step_ms_local = float(np.mean(batch_dev))

    # ---- the scans alone (not sharing a pass): Q6 by itself, Q1 by itself (C2 = Q1 at W=100).
    # The query's own CUDA events (result.device_ms, recorded on the engine stream around its
    # kernels); a ~50 us sleep kernel queued first lets the host enqueue the whole query before the
    # GPU reaches it, so no launch latency lands inside the window
    alone, alone_p99 = {}, {}
    for q in [x for x in ("q6", "q1", "q18") if x in ALL]:  # (Q18 alone: config C3)
        for _ in range(2):
            run_batch((q,), dev_flags)
        barrier()
        ms = []
        for _ in range(a.steps):
            flush_l2()
            with torch.cuda.stream(stream):
                torch.cuda._sleep(a.sleep_cycles)
            ms.append(run_batch((q,), dev_flags)[q][0])
        alone[q] = float(np.median(ms))
        alone_p99[q] = float(np.percentile(ms, 99))
    barrier()
    # C3 end to end: Q18 alone with its result rows copied to host memory (the D2H of the result
    # columns is inside; its bytes are reported), host wall clock around the call, median
    c3_e2e_ms = c3_d2h = None
    if "q18" in ALL:
        c3 = []
        for k in range(3 + min(a.steps, 10)):
            flush_l2()
            torch.cuda.synchronize()
            t0 = time.perf_counter()
            r = h.h2tap_run_query(eng, h.H2TAP_Q18, Q18_P)  # host result: columns in host memory
            _ = r.columns["amount_sum"][:1].sum() if r.nrows else 0  # host read
            dt = (time.perf_counter() - t0) * 1e3
            c3_d2h = int(sum(v.nbytes for v in r.columns.values()))
            h.h2tap_free(r)
            if k >= 3:
                c3.append(dt)
        c3_e2e_ms = float(np.median(c3))
    barrier()

    # ---- instrumented pass (same K steps): per-kernel CUDA events for the roofline; a 30 us gate
    # kernel at each query start keeps host launch latency out of every kernel's event window
    kern = {}
    for i in range(a.steps):
        flush_l2()
        out = run_batch(ALL, prof_flags)
        for q, (ms, ks, nrows, nl, tot) in out.items():
            for kname, kms in ks:
                kern.setdefault(kname, []).append(kms)
    barrier()
    clk = clocks.stop()
    step_ms, step_host_ms, q6_alone_ms, q1_alone_ms, q18_alone_ms, step_p50, step_p99 = max_over_ranks(
        [step_ms_local, step_host_ms_local, alone.get("q6", float("nan")), alone.get("q1", float("nan")),
         alone.get("q18", float("nan")), float(np.median(batch_dev)), float(np.percentile(batch_dev, 99))])
    lat = {q: float(np.median(v)) for q, v in per_query.items()}
    lat_max = dict(zip(lat, max_over_ranks(list(lat.values()))))
    nt = torch.tensor([n_ol], dtype=torch.float64, device=pg_dev)
    if world > 1:
        dist.all_reduce(nt, op=dist.ReduceOp.SUM)
    rows_total = int(nt.item())  # order_line rows of all ranks, each counted once per step
    value = rows_total / (step_ms / 1e3)

    plan_dense = bool(dense_seen) and all(dense_seen)
    plan_clustered = plan_dense and bool(clustered_seen) and all(clustered_seen)
    # ---- roofline for the dominant kernel (largest share of the step)
    kavg = {k: float(np.mean(v)) for k, v in kern.items()}
    sort_passes = ("v1" if os.environ.get("H2TAP_ORDER") == "v1"
                   else "v2" if os.environ.get("H2TAP_ORDER_CARRY") == "0" else "carry")
    # the dominant kernel: the largest share of the step among the kernels with a byte model (at
    # W = 100 the shared scan; on tiny snapshots a launch-bound kernel could otherwise win)
    modeled = [k for k in kavg if alg_bytes(k, n_ol, n_o, n_c, n_pass, sort_passes, box if plan_dense else None,
                                            plan_clustered and sort_passes == "carry")]
    dominant = max(modeled, key=kavg.get) if modeled else None
    peak, peak_src = peaks()
    rpeak = read_stream_peak(h, eng, stream) if rank == 0 else None
    roof = None
    if dominant:
        b = alg_bytes(dominant, n_ol, n_o, n_c, n_pass, sort_passes, box if plan_dense else None,
                      plan_clustered and sort_passes == "carry")
        if b:
            ach = b / (kavg[dominant] / 1e3) / 1e9
            tr = ncu_traffic().get(dominant)
            roof = {"bound": "hbm", "kernel": dominant, "achieved": round(ach, 1), "peak": peak,
                    "unit": "GB/s", "frac": round(ach / peak, 4), "traffic": tr,
                    "algorithmic_bytes_per_launch": int(b), "avg_launch_ms": round(kavg[dominant], 5),
                    "share_of_step": round(kavg[dominant] / step_ms_local, 4), "peak_source": peak_src,
                    "read_stream_peak_gbs": rpeak,
                    "frac_of_read_stream_peak": round(ach / rpeak, 4) if rpeak else None,
                    "timing": "CUDA events on the engine stream, instrumented pass of the same K steps"}
    kernels_summary = {}
    full_pass = "q6118_full_pass" in kavg  # Q18's probe ran inside the batch's shared pass
    # C3 runs Q18 alone (its own probe kernel): its byte model includes the probe's bytes
    q18_alg = int(alg_bytes("q18_probe_groupjoin", n_ol, n_o, n_c, n_pass, sort_passes,
                            box if plan_dense else None, plan_clustered and sort_passes == "carry") or 0) if full_pass else 0
    for k, v in kavg.items():
        b = alg_bytes(k, n_ol, n_o, n_c, n_pass, sort_passes, box if plan_dense else None,
                      plan_clustered and sort_passes == "carry")
        kernels_summary[k] = {"ms": round(v, 5), "share": round(v / step_ms_local, 4)}
        if b and k.startswith("q18"):
            q18_alg += int(b)
        if b:
            kernels_summary[k]["GB/s"] = round(b / (v / 1e3) / 1e9, 1)
            kernels_summary[k]["frac_hbm"] = round(b / (v / 1e3) / 1e9 / peak, 4)

    # ---- e2e: host buffers through the public API (H2D refresh + queries + D2H results)
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
    # pipelined (reported separately): the same calls with H2TAP_LOAD_ASYNC | H2TAP_LOAD_BORROW, so
    # step k's upload overlaps step k-1's result read-back and queries; each batch runs on the
    # latest PUBLISHED epoch (lag reported) — one rank only (a collective batch must see one epoch
    # on every rank)
    h.h2tap_sync(eng)
    barrier()
    lag = []
    e2e_pipe_s = float("nan")
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
    e2e_serial_s, = max_over_ranks([e2e_serial_s])

    # incremental (reported separately, weak #11 of round 1): the snapshot stays resident and each
    # step refreshes it with that step's committed OLTP changes only — NewOrder appends + Delivery
    # updates (copy-on-write pages) from pinned host buffers — then runs the batch on
    # the new epoch and reads the results back: the paper's fresh-snapshot loop
    e2e_inc = None
    if inc is not None:
        steps_all, n_ol_final, n_o_final, rows_all = inc
        half = len(steps_all) // 2
        steps_in, inc_rows = steps_all[:half], rows_all[:half]
        h.h2tap_sync(eng)
        h.h2tap_reserve(eng, "order_line", n_ol_final)
        h.h2tap_reserve(eng, "orders", n_o_final)
        st0 = None
        inc_d2h = 0
        barrier()
        t_inc = 0.0
        for k, (delta, updates, first, _) in enumerate(steps_in):
            if k == 2:
                barrier()
                st0 = h.h2tap_get_store_stats(eng)
                t0 = time.perf_counter()
            epoch += 1
            h.h2tap_refresh(eng, delta, updates, epoch, first_row=first)
            inc_d2h = 0
            for r in h.h2tap_run_queries(eng, [(plan, p, 0) for _, plan, p in plans]):
                assert r.epoch == epoch
                for c in r.columns.values():
                    inc_d2h += c.nbytes
                _ = r.columns[next(iter(r.columns))][:1].sum() if r.nrows else 0  # host read
                h.h2tap_free(r)
        barrier()
        t_inc = (time.perf_counter() - t0) / e2e_steps
        st1 = h.h2tap_get_store_stats(eng)
        t_inc, = max_over_ranks([t_inc])
        rows_inc = float(np.mean(inc_rows[2:]))
        if world > 1:
            t = torch.tensor([rows_inc], dtype=torch.float64, device=pg_dev)
            dist.all_reduce(t)
            rows_inc = float(t.item())
        e2e_inc = {"value": rows_inc / t_inc, "unit": UNIT, "ms_per_step": t_inc * 1e3, "steps": e2e_steps,
                   "h2d_bytes_per_step": int(np.mean([x[3] for x in steps_in[2:]])),
                   "d2h_bytes_per_step": int(inc_d2h),
                   "neworders_per_step_per_gpu": a.inc_neworders, "deliveries_per_step_per_gpu": a.inc_deliveries,
                   "order_line_rows_appended_per_step_per_gpu": int((inc_rows[-1] - inc_rows[1]) / e2e_steps),
                   "cow_pages_copied_per_step": (st1["cow_pages_copied"] - st0["cow_pages_copied"]) / e2e_steps,
                   "last_update_ms": round(st1["last_update_ms"], 4),
                   "how": "every step: h2tap_refresh of that step's NewOrder appends + Delivery "
                          "ol_delivery_d updates (pinned host buffers, copy-on-write epoch) + the "
                          "Q6/Q1/Q18 batch on the new epoch + results copied to host"}
        # pipelined: the same loop with device-resident results whose copy to pinned host buffers
        # (a second stream) overlaps the next step's refresh and batch; each step's results are
        # on the host before the step after next starts; every batch reads its own step's epoch
        d2h_stream = torch.cuda.Stream()
        host_bufs = {}
        pending = None

        def drain(p):
            rs_prev, ev_prev = p
            ev_prev.synchronize()
            for r in rs_prev:
                for name, c in r.columns.items():
                    if r.nrows:
                        _ = host_bufs[name][:1].sum()  # host read
                h.h2tap_free(r)
        steps_p, rows_p = steps_all[half:], rows_all[half:]
        d2h_p = 0
        for k, (delta, updates, first, _) in enumerate(steps_p):
            if k == 2:
                if pending is not None:
                    drain(pending)
                    pending = None
                barrier()
                t0 = time.perf_counter()
            epoch += 1
            h.h2tap_refresh(eng, delta, updates, epoch, first_row=first)
            rs = h.h2tap_run_queries(eng, [(plan, p, h.H2TAP_RESULT_DEVICE) for _, plan, p in plans])
            d2h_p = 0
            with torch.cuda.stream(d2h_stream):
                for r in rs:
                    assert r.epoch == epoch
                    if not r.nrows:
                        continue
                    for name, c in r.columns.items():
                        src = torch.as_tensor(c, device="cuda")
                        buf = host_bufs.get(name)
                        if buf is None or buf.numel() < src.numel() or buf.dtype != src.dtype:
                            buf = host_bufs[name] = torch.empty(int(src.numel() * 1.25) + 1024, dtype=src.dtype,
                                                                pin_memory=True)
                        buf[:src.numel()].copy_(src, non_blocking=True)
                        d2h_p += src.numel() * src.element_size()
                ev = torch.cuda.Event()
                ev.record(d2h_stream)
            if pending is not None:
                drain(pending)
            pending = (rs, ev)
        drain(pending)
        barrier()
        t_p = (time.perf_counter() - t0) / e2e_steps
        t_p, = max_over_ranks([t_p])
        rows_p_mean = float(np.mean(rows_p[2:]))
        if world > 1:
            t = torch.tensor([rows_p_mean], dtype=torch.float64, device=pg_dev)
            dist.all_reduce(t)
            rows_p_mean = float(t.item())
        e2e_inc["pipelined"] = {
            "value": rows_p_mean / t_p, "unit": UNIT, "ms_per_step": t_p * 1e3, "d2h_bytes_per_step": int(d2h_p),
            "how": "same steps with device-resident results (H2TAP_RESULT_DEVICE) copied to pinned host "
                   "buffers on a second stream, overlapping the next step's refresh and batch; every batch "
                   "reads its own step's epoch; results on the host one step later"}

    # ---- CPU oracle baseline (rank 0, N = 1 only, bounded sample) and config C1
    cpu = c1 = None
    if rank == 0 and world == 1 and not a.no_cpu_baseline:
        # the step's own inputs: numpy views of the pinned host columns the e2e runs upload
        v, dt, n, core, reps, tot = cpu_oracle_steps({t: {c: x.numpy() for c, x in cols.items()}
                                                      for t, cols in pinned.items()})
        cpu = dict({"value": v, "unit": UNIT, "cores": 1, "kind": "oracle", "pinned_core": core,
                    "sample": f"the bench's step itself: oracle Q6+Q1+Q18 over this rank's whole W={hi - lo} "
                              f"table set ({n} order_line rows), {reps} steps in {tot:.1f} s of CPU work, "
                              f"median step {dt:.2f} s, single thread on core {core}"},
                   **host_cpu())
    if rank == 0 and world == 1 and not a.no_c1:
        c1 = c1_line(h, a)

    if rank == 0:
        line = {
            "metric": METRIC, "value": value, "unit": UNIT, "n_gpus": world, "steps": a.steps,
            "warmup": a.warmup, "ms_per_step": step_ms, "higher_is_better": True,
            "ms_per_step_host_return": round(step_host_ms, 5),
            "scaling": "strong" if strong else "weak", "vs_baseline": None, "dtype": "int64",
            "data": "synthetic",
            "config": {"workload": workload_name(a, world),
                       "warehouses_total": W, "warehouses_per_gpu": W / world,
                       "order_line_rows_total": rows_total, "order_line_rows_rank0": n_ol,
                       "orders_rows_rank0": n_o, "customer_rows_rank0": n_c,
                       "rows_counted": rows_counted(a),
                       "queries_per_step": len(ALL),
                       **({"shared_device": "FUNCTIONAL CHECK ONLY: all ranks on one GPU"} if a.share_device else {}), "parallelism": f"row-sharded by warehouse x{world}",
                       "merge": ("peer-memory kernels over NVLink (Q6 allreduce, Q1 group lists, Q18 "
                                 "range-partitioned ORDER BY; DESIGN.md §6)" if world > 1 else "none (1 GPU)"),
                       "scan_sharing": (("the batch's full pass: Q6, Q1 and Q18's probe + group-join share one "
                                         "read of order_line (latency_ms.q6_in_batch includes Q18's join-index "
                                         "verify/build and the pass, q1_in_batch is Q1's finalize, q18_in_batch "
                                         "starts after its probe; DESIGN.md §4.5)" if full_pass else
                                         "Q6 and Q1 of the batch share one pass over order_line "
                                         "(latency_ms.q6 includes it, q1 is its finalize; DESIGN.md §4.5)")
                                        + "; every query computes its full result; the scans alone are in "
                                          "latency_ms.q6_alone / q1_alone, Q18 alone in c3"
                                        if os.environ.get("H2TAP_SHARED_SCAN", "1") != "0" else "off"),
                       "timing": "ms_per_step: the batch's GPU span, CUDA events recorded by the library on its "
                                 "stream around the batch (h2tap_last_batch_ms), per step, mean; "
                                 "ms_per_step_host_return: bench events around the call, end recorded "
                                 "after it returned to Python",
                       "l2": ("inputs > L2; between steps (outside events) 512 MB written then 256 MB read to flush L2"
                              if flush is not None else "inputs > L2 (no flush)")},
            "latency_ms": dict({f"{q}_in_batch": round(v, 4) for q, v in lat_max.items()},
                               q6_alone=round(q6_alone_ms, 4), q1_alone=round(q1_alone_ms, 4),
                               **({("q6_q1_q18probe_full_pass_batch" if full_pass else "q6_q1_shared_scan_batch"):
                                   round(lat_max["q6"] + lat_max["q1"], 4)}
                                  if "q6" in lat_max and "q1" in lat_max else {})),
            "step_ms_median": round(step_p50, 5), "step_ms_p99": round(step_p99, 5),
            "c2": ({"workload": "CH Q1 alone at W=100 per GPU (BASELINE configs[1]), device time (query's own events), "
                               "median / p99 of the K steps", "latency_ms": round(q1_alone_ms, 4),
                    "latency_p99_ms": round(alone_p99.get("q1", float("nan")), 4),
                    "rows_per_s": rows_total / (q1_alone_ms / 1e3),
                    "GB/s": round(24 * n_ol / (q1_alone_ms / 1e3) / 1e9, 1),
                    "frac_of_8TBps": round(24 * n_ol / (q1_alone_ms / 1e3) / 8.0e12, 4),
                    "frac_of_measured_peak": round(24 * n_ol / (q1_alone_ms / 1e3) / 1e9 / peak, 4),
                    "target": "kernel <= 129 us (>= 70 % of 8 TB/s), SURVEY.md §8(d)"} if "q1" in ALL else None),
            "c3": ({"workload": "CH Q18 alone at W=100 per GPU (BASELINE configs[2]), 1 GPU",
                    "device_ms": round(q18_alone_ms, 4), "device_p99_ms": round(alone_p99.get("q18", float("nan")), 4),
                    "e2e_ms": round(c3_e2e_ms, 3) if c3_e2e_ms else None, "e2e_d2h_bytes": c3_d2h,
                    "e2e_how": "h2tap_run_query with a host result (the result columns' D2H inside), host wall "
                               "clock around the call, median",
                    "result_rows": n_pass_total,
                    "algorithmic_bytes": q18_alg,
                    "GB/s_on_algorithmic_bytes": round(q18_alg / (q18_alone_ms / 1e3) / 1e9, 1) if q18_alg else None,
                    "frac_of_measured_peak": round(q18_alg / (q18_alone_ms / 1e3) / 1e9 / peak, 4) if q18_alg else None,
                    "frac_of_8TBps": round(q18_alg / (q18_alone_ms / 1e3) / 8.0e12, 4) if q18_alg else None,
                    "bytes_model": "sum of the Q18 kernels' algorithmic bytes (bench.py alg_bytes, DESIGN.md §5)"}
                   if "q18" in ALL and world == 1 else None),
            "rows_per_s": dict({f"{q}_in_batch": rows_total / (v / 1e3) for q, v in lat_max.items()},
                               q6_alone=rows_total / (q6_alone_ms / 1e3), q1_alone=rows_total / (q1_alone_ms / 1e3)),
            "q18_result_rows_total": n_pass_total, "q18_result_rows_rank0": n_pass,
            "q18_join_indexes": ("positional: orders / customer verified in key order on the device (DESIGN.md §4.3)"
                                 if plan_clustered else "perfect hash" if plan_dense else "hash tables"),
            "roofline": roof,
            "kernels": kernels_summary,
            "cpu_baseline": cpu,
            "c1": c1,
            "e2e": {"value": rows_total / e2e_serial_s, "unit": UNIT, "h2d_bytes_per_step": int(h2d_bytes),
                    "d2h_bytes_per_step": int(d2h), "ms_per_step": e2e_serial_s * 1e3, "steps": e2e_steps,
                    "mode": "serial: each step's queries read that step's upload",
                    "how": "every step: full snapshot upload of the step's inputs from pinned host "
                           "buffers (h2tap_load_snapshot) + Q6/Q1/Q18 batch (h2tap_run_queries) + "
                           "results copied to host"},
            "e2e_pipelined": ({"value": rows_total / e2e_pipe_s, "unit": UNIT, "ms_per_step": e2e_pipe_s * 1e3,
                               "epoch_lag": sorted(set(lag)),
                               "how": "H2TAP_LOAD_ASYNC|H2TAP_LOAD_BORROW: uploads overlap the previous "
                                      "step's queries and read-back; each batch reads the latest "
                                      "published epoch (lag in epochs listed)"} if world == 1 else None),
            "e2e_incremental": e2e_inc,
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
