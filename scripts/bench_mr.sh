#!/bin/bash
# bench.py smoke: N=1 default line, then --gpus 2 must fail cleanly on a 1-GPU box
mkdir -p gpurun_out
timeout 900 python bench.py --steps 10 --warmup 3 2>&1 | tail -3 | tee gpurun_out/bench.txt
timeout 120 python bench.py --gpus 2 --steps 2 --warmup 3; echo "gpus2 rc=$?"
