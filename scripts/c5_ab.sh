#!/bin/bash
# A/B of config C5 (native driver, W=1000, E=100 ms, 20 s) over engine knobs / build variants
mkdir -p gpurun_out
for cfg in "$@"; do
  env $cfg timeout 600 python tools/c5_native.py --out gpurun_out/c5ab.json -- --warehouses 1000 --seconds 20 \
      --epoch-ms 100 --tps 400000 --threads 8 > /dev/null 2>&1
  python -c "
import json; d=json.load(open('gpurun_out/c5ab.json'))
print('$cfg', 'refresh', d['refresh_ms_per_epoch_mean'], 'batches/s', d['query_batches_per_s'], 'lag p50/p99/max', d['freshness_lag_ms_p50'], d['freshness_lag_ms_p99'], d['freshness_lag_ms_max'])"
done
