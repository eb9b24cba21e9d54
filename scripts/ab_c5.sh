# C5 A/B (mixed HTAP): knob settings, 15 s each
mkdir -p gpurun_out
for v in "H2TAP_PDL=1" "H2TAP_PDL=0" "H2TAP_PDL=1" "H2TAP_PDL=0"; do
  env $v timeout 600 python scripts/htap_mixed.py --warehouses 100 --seconds 15 --epoch-ms 100 --out gpurun_out/c5.json > /dev/null 2>&1
  python -c "
import json; d=json.load(open('gpurun_out/c5.json'))
print('$v', {k: round(d[k],1) for k in ('epochs_published','refresh_ms_per_epoch_mean','query_batches_per_s','batch_latency_ms_p50','batch_latency_ms_p99','freshness_lag_ms_p50','freshness_lag_ms_p99')})"
done
