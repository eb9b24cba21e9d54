#!/bin/bash
# config C5 (native driver) at W=1000 on one GPU for the three epoch periods SURVEY.md §8(d) names
# (E = 10, 100, 1000 ms): the freshness / throughput trade-off of the snapshot period
mkdir -p gpurun_out
for E in 10 100 1000; do
  timeout 900 python tools/c5_native.py --out gpurun_out/c5_native_w1000_e${E}.json -- --warehouses 1000 \
      --seconds 30 --epoch-ms $E --tps 400000 --threads 8 > /dev/null 2>&1
  echo "E=$E rc=$?"
done
