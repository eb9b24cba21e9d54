"""GPU parity of the multi-GPU path (§8 a7 / e) on ONE device: N logical ranks,
one engine each, connected with h2tap_peer_connect_local, so every world > 1 code path of the
library runs — the peer allreduce (Q6, Q14), the group-list push + merge (Q1, Q12, Q4), the
distributed ORDER BY with its record exchange (Q18, Q3) — exactly as across GPUs, the merges
going through one device's memory instead of NVLink. Each rank loads its warehouse range
(chgen.warehouse_ranges, R15); results are compared with the CPU oracle over ALL
warehouses: Q6/Q1/Q14/Q12/Q4 on every rank, and the rank slices of Q18/Q3 concatenated in rank
order equal the oracle's globally ordered result (rows bit-exact, order exact).
A second part runs two PROCESSES on the one GPU (CUDA IPC handles exchanged over gloo), the
multi-process bootstrap bench.py uses."""
import math
import os
import socket
import subprocess
import sys

import numpy as np
import pytest

import chgen
import oracle
from chref import Q1_CUTOFF, Q6_D_HI, Q6_D_LO, Q18_HAVING
from test_oracle_next2 import Q4_HI, Q4_LO, Q12_HI, Q14_HI, Q14_LO
from test_oracle_q3 import Q3_LO

pytestmark = pytest.mark.gpu
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
Q18_NAMES = ["c_last", "c_id", "o_id", "o_entry_d", "o_ol_cnt", "amount_sum", "o_w_id", "o_d_id"]
Q3_NAMES = ["ol_o_id", "ol_w_id", "ol_d_id", "revenue", "o_entry_d"]
HEAP = 64 << 20  # per-rank peer heap (records of the ORDER BY exchange): plenty at these sizes


@pytest.fixture(scope="module")
def h():
    import paper_conf_cidr_appuswamykpa17_b200 as mod
    return mod


def all_plans(h):
    return (h.H2TAP_Q1, h.H2TAP_Q6, h.H2TAP_Q18, h.H2TAP_Q14, h.H2TAP_Q12, h.H2TAP_Q4, h.H2TAP_Q3)


def shards(total_w, world, seed, mode="spread", empty_rank=None):
    """Per-rank tables of a warehouse-range split (an optional rank gets no warehouse), and the
    whole table set the oracle evaluates."""
    ranges = chgen.warehouse_ranges(total_w, world if empty_rank is None else world - 1)
    if empty_rank is not None:
        ranges.insert(empty_rank, (ranges[empty_rank - 1][1] if empty_rank else 1,) * 2)
    parts = [chgen.generate(lo, hi, seed=seed, mode=mode) for lo, hi in ranges]
    whole = chgen.generate(1, total_w + 1, seed=seed, mode=mode)
    return parts, whole


def load_all(h, engines, parts, epoch=1, plans=None):
    for e, t in zip(engines, parts):
        h.h2tap_load_snapshot(e, h.hot_path_tables(t, plans or all_plans(h)), epoch)


def batch(h, engines, queries):
    """One collective batch on every rank (one thread each); per rank a list of dicts."""
    def run(e):
        rs = h.h2tap_run_queries(e, queries)
        out = []
        for r in rs:
            d = r.to_numpy()
            d["_nulls"] = dict(r.nulls)
            d["_meta"] = (r.nrows, r.row_offset, r.total_rows, r.kernel_launches)
            out.append(d)
            h.h2tap_free(r)
        return out
    return h.run_collective(engines, run)


def concat_slices(per_rank, idx, names):
    out = {}
    for k in names:
        out[k] = np.concatenate([per_rank[r][idx][k] for r in range(len(per_rank))])
    return out


def check_ordered_slices(per_rank, idx, want, names):
    """Rank slices in rank order == the oracle's ordered result; offsets/totals consistent."""
    got = concat_slices(per_rank, idx, names)
    for k in names:
        assert np.array_equal(got[k], want[k]), (k, got[k][:6], want[k][:6])
    total = len(want[names[0]])
    off = 0
    for r in range(len(per_rank)):
        nrows, row_offset, total_rows, _ = per_rank[r][idx]["_meta"]
        assert (row_offset, total_rows) == (off, total), (r, row_offset, off, total_rows, total)
        off += nrows


def assert_q1(got, want):
    for k in ("ol_number", "sum_qty", "sum_amount", "count_order"):
        assert np.array_equal(got[k], want[k]), k
    for k in ("avg_qty", "avg_amount"):
        for a, b in zip(got[k].tolist(), want[k].tolist()):
            assert math.isclose(a, b, rel_tol=1e-9, abs_tol=0.0), (k, a, b)


def assert_q6(got, want):
    assert int(got["count_rows"][0]) == want["count"]
    if want["revenue"] is None:
        assert got["_nulls"]["revenue"][0] == 1
    else:
        assert int(got["revenue"][0]) == want["revenue"]


def hot_batch(h, cut=Q1_CUTOFF, d=(Q6_D_LO, Q6_D_HI, 1, 100000), having=Q18_HAVING, flags=0):
    return [(h.H2TAP_Q6, list(d), flags), (h.H2TAP_Q1, [cut], flags), (h.H2TAP_Q18, [having], flags)]


@pytest.mark.parametrize("world,total_w", [(2, 3), (4, 5), (8, 8)])
def test_hot_path_batch_matches_whole_oracle(h, world, total_w):
    """The bench's step (Q6 + Q1 shared scan, Q18) on N logical ranks, repeated three times with
    different parameters (both mailbox / heap parities), vs the oracle over all warehouses."""
    parts, whole = shards(total_w, world, seed=31 + world)
    engines = h.open_local_group(world, 0, HEAP)
    try:
        load_all(h, engines, parts)
        rng = np.random.default_rng(world)
        cases = [(Q1_CUTOFF, (Q6_D_LO, Q6_D_HI, 1, 100000), Q18_HAVING)]
        for _ in range(2):
            lo = int(rng.integers(chgen.TS_1995, chgen.TS_2025))
            cases.append((int(rng.integers(chgen.TS_1995, chgen.TS_2025)),
                          (lo, int(rng.integers(lo, chgen.TS_2025)), 2, 8), int(rng.integers(0, 3_000_000))))
        for cut, d, having in cases:
            res = batch(h, engines, hot_batch(h, cut, d, having))
            w6, w1, w18 = oracle.q6(whole, *d), oracle.q1(whole, cut), oracle.q18(whole, having)
            for r in range(world):
                assert_q6(res[r][0], w6)
                assert_q1(res[r][1], w1)
            check_ordered_slices(res, 2, w18, Q18_NAMES)
            # the range partition is balanced to within a bucket
            sizes = [res[r][2]["_meta"][0] for r in range(world)]
            assert max(sizes) - min(sizes) <= 2048 + len(w18["o_id"]) // world, sizes
    finally:
        for e in engines:
            h.h2tap_close(e)


def test_next2_queries_distributed(h):
    """Q14 (allreduce), Q12 / Q4 (group tables), Q3 (distributed ORDER BY) on 3 logical ranks,
    hash and perfect-hash join indexes."""
    world = 3
    parts, whole = shards(4, world, seed=44)
    engines = h.open_local_group(world, 0, HEAP)
    try:
        load_all(h, engines, parts)
        for flags in (0, 4):
            q = [(h.H2TAP_Q14, [Q14_LO, Q14_HI, 0x5052], flags), (h.H2TAP_Q12, [Q12_HI], flags),
                 (h.H2TAP_Q4, [Q4_LO, Q4_HI], flags), (h.H2TAP_Q3, [Q3_LO, 0x4100], flags)]
            res = batch(h, engines, q)
            w14, w12, w4 = oracle.q14(whole, Q14_LO, Q14_HI), oracle.q12(whole, Q12_HI), oracle.q4(whole, Q4_LO, Q4_HI)
            for r in range(world):
                g = res[r][0]
                assert (int(g["sum_promo"][0]), int(g["sum_amount"][0]), int(g["count_rows"][0])) == \
                    (w14["sum_promo"], w14["sum_amount"], w14["count"])
                assert math.isclose(float(g["promo_revenue"][0]), w14["promo_revenue"], rel_tol=1e-9)
                for k in w12:
                    assert np.array_equal(res[r][1][k], w12[k]), k
                for k in w4:
                    assert np.array_equal(res[r][2][k], w4[k]), k
            check_ordered_slices(res, 3, oracle.q3(whole, Q3_LO, b"A"), Q3_NAMES)
    finally:
        for e in engines:
            h.h2tap_close(e)


def test_empty_rank_sparse_keys_and_device_results(h):
    """A rank with no warehouse (empty tables), Q1 keys outside the dense range on some ranks
    only, results left on the device, the ORDER BY's output capacity exceeded on purpose
    (re-emitted into exact columns), and HAVING at an exact group sum."""
    world = 4
    parts, whole = shards(3, world, seed=52, empty_rank=2)
    rng = np.random.default_rng(52)
    for r in (0, 3):  # sparse ol_number keys on two ranks, consistently in the whole table set
        ol = parts[r]["order_line"]
        pick = rng.random(len(ol["ol_number"])) < 0.3
        ol["ol_number"] = ol["ol_number"].copy()
        ol["ol_number"][pick] = rng.integers(-500, 500, int(pick.sum()), dtype=np.int32)
    whole = chgen.concat_tables([p for p in parts if len(p["order_line"]["ol_w_id"])])
    whole["item"] = parts[0]["item"]
    engines = h.open_local_group(world, 0, HEAP)
    try:
        load_all(h, engines, parts)
        sums = oracle.q18(whole, -1)["amount_sum"]
        having = int(sums[len(sums) // 3])
        os.environ["H2TAP_DIST_OUT_CAP"] = "100"
        try:
            res = batch(h, engines, hot_batch(h, having=having, flags=1))  # H2TAP_RESULT_DEVICE
        finally:
            del os.environ["H2TAP_DIST_OUT_CAP"]
        w18 = oracle.q18(whole, having)
        assert having not in w18["amount_sum"].tolist()
        for r in range(world):
            assert_q6(res[r][0], oracle.q6(whole, Q6_D_LO, Q6_D_HI, 1, 100000))
            assert_q1(res[r][1], oracle.q1(whole, Q1_CUTOFF))
        check_ordered_slices(res, 2, w18, Q18_NAMES)
        assert res[2][2]["_meta"][0] >= 0
    finally:
        for e in engines:
            h.h2tap_close(e)


def test_errors_are_collective(h):
    """A duplicate orders key on ONE rank fails Q18 with EDUPKEY on EVERY rank; a peer heap too
    small for a rank's share fails with ENOMEM on every rank; the group stays usable after both."""
    world = 2
    parts, whole = shards(2, world, seed=61)
    dup = {k: v.copy() for k, v in parts[1]["orders"].items()}
    for k in dup:
        dup[k] = np.concatenate([dup[k], dup[k][:1]])
    bad = dict(parts[1])
    bad["orders"] = dup
    engines = h.open_local_group(world, 0, 1 << 18)  # 128 KB per parity: 8192 records
    try:
        load_all(h, engines, [parts[0], bad])

        def q18(e):
            try:
                r = h.h2tap_run_query(e, h.H2TAP_Q18, [-1])
                r.free()
                return 0
            except h.H2tapError as x:
                return x.status
        assert h.run_collective(engines, q18) == [h.H2TAP_EDUPKEY] * world
        load_all(h, engines, parts, epoch=2)
        assert h.run_collective(engines, q18) == [h.H2TAP_ENOMEM] * world  # 60k rows: ~30k per rank
        thr = int(oracle.q18(whole, -1)["amount_sum"][4000])                # ~2k rows per rank: fits
        res = batch(h, engines, hot_batch(h, having=thr))
        check_ordered_slices(res, 2, oracle.q18(whole, thr), Q18_NAMES)
        for r in range(world):
            assert_q1(res[r][1], oracle.q1(whole, Q1_CUTOFF))
    finally:
        for e in engines:
            h.h2tap_close(e)


def test_missing_peer_times_out(h, monkeypatch):
    """A rank that never joins the collective: the others fail with EPEER after the timeout
    (no hang), and the group is reported broken afterwards."""
    monkeypatch.setenv("H2TAP_PEER_TIMEOUT_MS", "1500")
    parts, _ = shards(2, 2, seed=71)
    engines = h.open_local_group(2, 0, HEAP)
    try:
        load_all(h, engines, parts)
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_run_query(engines[0], h.H2TAP_Q6)  # rank 1 never calls
        assert ei.value.status == h.H2TAP_EPEER
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_run_query(engines[0], h.H2TAP_Q6)
        assert ei.value.status == h.H2TAP_EPEER and "failed earlier" in str(ei.value)
    finally:
        for e in engines:
            h.h2tap_close(e)


def test_unconnected_and_bad_connect(h):
    e = h.h2tap_open(0, 0, 2)
    try:
        h.h2tap_load_snapshot(e, h.hot_path_tables(chgen.generate(1, 2, seed=1)), 1)
        with pytest.raises(h.H2tapError) as ei:
            h.h2tap_run_query(e, h.H2TAP_Q6)
        assert ei.value.status == h.H2TAP_EPEER
        with pytest.raises(h.H2tapError):
            h.h2tap_peer_connect_local([e])          # one engine is not a group
        assert len(h.h2tap_peer_handle(e)) == 64
    finally:
        h.h2tap_close(e)


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def test_two_processes_one_gpu_ipc(h, tmp_path):
    """Two processes, ranks 0 and 1, both on cuda:0: peer segments mapped with CUDA IPC handles
    exchanged over a gloo process group (the multi-process bootstrap of bench.py); each process
    checks its results against the whole-table oracle."""
    port = _free_port()
    script = os.path.join(ROOT, "tests", "mp_rank.py")
    env = dict(os.environ, MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port), WORLD_SIZE="2",
               H2TAP_PEER_TIMEOUT_MS="60000", PYTHONPATH=ROOT + os.pathsep + os.path.join(ROOT, "tests"))
    procs = [subprocess.Popen([sys.executable, script, str(tmp_path)], env=dict(env, RANK=str(r)),
                              stdout=subprocess.PIPE, stderr=subprocess.STDOUT, text=True) for r in range(2)]
    outs = []
    for p in procs:
        try:
            out, _ = p.communicate(timeout=300)
        except subprocess.TimeoutExpired:
            p.kill()
            out, _ = p.communicate()
        outs.append(out)
    for r, p in enumerate(procs):
        assert p.returncode == 0, f"rank {r}:\n{outs[r][-3000:]}"
        assert "RANK_OK" in outs[r], outs[r][-2000:]


def test_bench_two_ranks_functional():
    """bench.py's N-rank path end to end (it spawns its ranks, maps the peer segments over the
    process group, takes the max over ranks, sums the rows): --share-device puts both ranks on the
    one GPU (CUDA IPC between processes, gloo plumbing). Functional only: the line says so."""
    import json as _json
    env = {k: v for k, v in os.environ.items() if k not in ("RANK", "WORLD_SIZE", "LOCAL_RANK")}
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--gpus", "2", "--share-device",
                        "--steps", "2", "--warmup", "3", "--warehouses", "2", "--no-cpu-baseline", "--no-c1",
                        "--e2e-steps", "2"], capture_output=True, text=True, env=env, timeout=600)
    assert r.returncode == 0, r.stderr[-3000:]
    line = _json.loads([x for x in r.stdout.splitlines() if x.startswith("{")][-1])
    assert line["n_gpus"] == 2 and line["config"]["shared_device"]
    whole = chgen.generate(1, 5, seed=1)
    assert line["config"]["order_line_rows_total"] == len(whole["order_line"]["ol_w_id"])
    assert line["q18_result_rows_total"] == len(oracle.q18(whole, Q18_HAVING)["o_id"])
    assert line["gpu_launches"] > 0 and line["value"] > 0
