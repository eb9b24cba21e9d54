#!/bin/bash
for c in 200000 600000 1200000; do
  timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu-baseline --no-c1 --sleep-cycles $c 2>/dev/null | tail -1 | python -c "
import json,sys
d=json.loads(sys.stdin.read()); print('sleep $c step', round(d['ms_per_step'],4), {k: v for k, v in d['latency_ms'].items()})"
done
