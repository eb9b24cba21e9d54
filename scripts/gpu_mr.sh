#!/bin/bash
# Multi-rank (loopback + two-process) GPU tests, then the rest of the GPU suite
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv,noheader
timeout 900 python -m pytest tests/test_gpu_multirank.py -q --timeout 300 -rf -x "$@" 2>&1 | tail -40 | tee gpurun_out/pytest_mr.txt
