#!/bin/bash
# config C5 with the native driver: parity test, then W=100 and W=1000 runs (epoch 100 ms)
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_c5_native.py -q -x 2>&1 | tail -3
timeout 300 python tools/c5_native.py --out gpurun_out/c5_native_w100.json -- --warehouses 100 --seconds 20 --epoch-ms 100 --tps 400000 --threads 4
timeout 900 python tools/c5_native.py --out gpurun_out/c5_native_w1000.json -- --warehouses 1000 --seconds 30 --epoch-ms 100 --tps 400000 --threads 8
