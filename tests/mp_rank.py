"""One rank of tests/test_gpu_multirank.py::test_two_processes_one_gpu_ipc (not collected by
pytest): opens an engine with world 2 on cuda:0, exchanges CUDA IPC handles of the peer
segments over a gloo process group, loads its warehouse range, runs the hot-path batch twice and
checks it against the oracle over all warehouses. Prints RANK_OK on success."""
import os
import sys

import numpy as np
import torch.distributed as dist

import chgen
import oracle
import paper_conf_cidr_appuswamykpa17_b200 as h
from chref import Q1_CUTOFF, Q6_D_HI, Q6_D_LO, Q18_HAVING

NAMES = ["c_last", "c_id", "o_id", "o_entry_d", "o_ol_cnt", "amount_sum", "o_w_id", "o_d_id"]


def main():
    rank, world = int(os.environ["RANK"]), int(os.environ["WORLD_SIZE"])
    dist.init_process_group("gloo", rank=rank, world_size=world)
    total_w = 3
    lo, hi = chgen.warehouse_ranges(total_w, world)[rank]
    part = chgen.generate(lo, hi, seed=81)
    whole = chgen.generate(1, total_w + 1, seed=81)
    e = h.h2tap_open(0, rank, world, 64 << 20)
    try:
        h.connect_torch_group(e)
        h.h2tap_load_snapshot(e, h.hot_path_tables(part), 1)
        for having in (Q18_HAVING, 1_000_000):
            rs = h.h2tap_run_queries(e, [(h.H2TAP_Q6, [Q6_D_LO, Q6_D_HI, 1, 100000], 0),
                                         (h.H2TAP_Q1, [Q1_CUTOFF], 0), (h.H2TAP_Q18, [having], 0)])
            g6, g1, g18 = (r.to_numpy() for r in rs)
            off, total = rs[2].row_offset, rs[2].total_rows
            for r in rs:
                h.h2tap_free(r)
            w6 = oracle.q6(whole, Q6_D_LO, Q6_D_HI, 1, 100000)
            assert int(g6["revenue"][0]) == w6["revenue"] and int(g6["count_rows"][0]) == w6["count"]
            w1 = oracle.q1(whole, Q1_CUTOFF)
            for k in ("ol_number", "sum_qty", "sum_amount", "count_order"):
                assert np.array_equal(g1[k], w1[k]), k
            w18 = oracle.q18(whole, having)
            assert total == len(w18["o_id"])
            n = len(g18["o_id"])
            for k in NAMES:  # this rank's slice of the global order
                assert np.array_equal(g18[k], w18[k][off:off + n]), k
            sizes = [None] * world
            dist.all_gather_object(sizes, (off, n))
            assert sorted(sizes)[0][0] == 0 and sum(s[1] for s in sizes) == total
        print("RANK_OK", rank, flush=True)
    finally:
        h.h2tap_close(e)
        dist.destroy_process_group()


if __name__ == "__main__":
    sys.exit(main())
