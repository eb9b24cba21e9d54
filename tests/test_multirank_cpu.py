"""World-size-2 CPU (gloo) coverage of the N>1 path's host logic: warehouse sharding and the
merge semantics the library implements:
  Q6  -> allreduce(sum) of {revenue, count}
  Q1  -> allgather of per-rank group lists, merge by key (integer sums)
  Q18 -> groups are warehouse-local: the union of the shards' rows, ordered, is the whole result
         (the library then range-partitions that order over the ranks)
Each rank computes its partials with the oracle on its own shard; rank 0 checks the merged
result against the oracle over all warehouses. This pins the DEFINITION of the merges (that they
are exact under re-partitioning); the library's own world > 1 kernels run in
tests/test_gpu_multirank.py (N logical ranks on one GPU, and two processes over CUDA IPC).
bench.py's multi-rank launcher is checked here too (it refuses to run N ranks without N GPUs)."""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import chgen

W = 4
SEED = 23


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, q):
    import sys
    sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
    import oracle
    from chref import Q1_CUTOFF, Q6_D_HI, Q6_D_LO, Q18_HAVING
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        lo, hi = chgen.warehouse_ranges(W, world)[rank]
        part = chgen.generate(lo, hi, seed=SEED, with_item=False)
        # Q6
        p6 = oracle.q6(part, Q6_D_LO, Q6_D_HI, 1, 100000)
        t6 = torch.tensor([p6["revenue"] or 0, p6["count"]], dtype=torch.int64)
        dist.all_reduce(t6)
        # Q1: allgather group lists (key, qty, amt, cnt), merge by key
        p1 = oracle.q1(part, Q1_CUTOFF)
        mine = np.stack([p1["ol_number"].astype(np.int64), p1["sum_qty"], p1["sum_amount"],
                         p1["count_order"]], axis=1)
        lists = [None] * world
        dist.all_gather_object(lists, mine)
        merged = {}
        for arr in lists:
            for k, qty, amt, cnt in arr.tolist():
                m = merged.setdefault(k, [0, 0, 0])
                m[0] += qty; m[1] += amt; m[2] += cnt
        # Q18: groups are warehouse-local, so the union of the shards' result rows in the global
        # ORDER BY is the whole result (the library range-partitions that order over the ranks)
        p18 = oracle.q18(part, Q18_HAVING)
        rows = list(zip(*[p18[n].tolist() for n, _ in oracle.Q18_COLUMNS]))
        gathered = [None] * world if rank == 0 else None
        dist.gather_object(rows, gathered, dst=0)
        if rank == 0:
            whole = chgen.generate(1, W + 1, seed=SEED, with_item=False)
            w6 = oracle.q6(whole, Q6_D_LO, Q6_D_HI, 1, 100000)
            w1 = oracle.q1(whole, Q1_CUTOFF)
            w18 = oracle.q18(whole, Q18_HAVING)
            ok = t6.tolist() == [w6["revenue"], w6["count"]]
            ok &= sorted(merged) == w1["ol_number"].tolist()
            for i, k in enumerate(w1["ol_number"].tolist()):
                ok &= merged[k] == [int(w1["sum_qty"][i]), int(w1["sum_amount"][i]),
                                    int(w1["count_order"][i])]
            allrows = [r for g in gathered for r in g]
            # ORDER BY amount_sum DESC, o_entry_d, o_w_id, o_d_id, o_id (columns 5, 3, 6, 7, 2)
            allrows.sort(key=lambda r: (-r[5], r[3], r[6], r[7], r[2]))
            want = list(zip(*[w18[n].tolist() for n, _ in oracle.Q18_COLUMNS]))
            ok &= allrows == want
            q.put(bool(ok))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world", [2])
def test_gloo_sharded_merge_equals_whole(world):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    for p in procs:
        p.join(timeout=300)
        assert p.exitcode == 0
    assert q.get(timeout=10) is True


def test_bench_refuses_more_ranks_than_gpus():
    """bench.py --gpus 2 without a torchrun environment spawns its ranks itself only when two
    GPUs are visible; otherwise it reports the error and exits non-zero (never a silent N=1)."""
    import subprocess
    import sys
    root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
    env = {k: v for k, v in os.environ.items() if k not in ("RANK", "WORLD_SIZE", "LOCAL_RANK")}
    env["CUDA_VISIBLE_DEVICES"] = ""
    r = subprocess.run([sys.executable, os.path.join(root, "bench.py"), "--gpus", "2", "--steps", "1"],
                       capture_output=True, text=True, env=env, timeout=600)
    assert r.returncode != 0
    assert "error" in r.stdout and "--gpus 2" in r.stdout
    env.update(RANK="0", WORLD_SIZE="1", LOCAL_RANK="0")
    r = subprocess.run([sys.executable, os.path.join(root, "bench.py"), "--gpus", "2", "--steps", "1"],
                       capture_output=True, text=True, env=env, timeout=600)
    assert r.returncode != 0 and "WORLD_SIZE=1" in r.stdout
