#!/bin/bash
# config C4 on one GPU (strong-scaling N=1 point): Q6 + Q1 over W=1000, and the Q18 step at W=1000
mkdir -p gpurun_out
timeout 1500 python bench.py --total-warehouses 1000 --plans q6,q1 --steps 10 --warmup 3 --e2e-steps 3 --no-c1 --no-cpu-baseline 2>gpurun_out/c4.err | tail -1 > gpurun_out/bench_c4_q61_w1000.json
tail -c 300 gpurun_out/c4.err
python -c "
import json; d=json.loads(open('gpurun_out/bench_c4_q61_w1000.json').read())
print('step', d['ms_per_step'], d['latency_ms'], d['roofline']['frac'], d['roofline']['achieved'])"
