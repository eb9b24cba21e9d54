#!/bin/bash
# compute-sanitizer over every plan (scripts/exp/sanitize_all.py) and the Q18 ORDER BY paths
# (scripts/exp/race_q18.py); logs under gpurun_out/
mkdir -p gpurun_out
CS=/usr/local/cuda/bin/compute-sanitizer
$CS --tool memcheck python scripts/exp/sanitize_all.py > gpurun_out/memcheck_all.txt 2>&1; echo "memcheck all rc=$?"
$CS --tool racecheck --racecheck-report all --print-limit 100 python scripts/exp/sanitize_all.py > gpurun_out/racecheck_all.txt 2>&1; echo "racecheck all rc=$?"
bash scripts/race.sh
for f in gpurun_out/memcheck_all.txt gpurun_out/racecheck_all.txt; do echo "== $f"; tail -n 2 $f; done
