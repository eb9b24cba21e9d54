#!/bin/bash
mkdir -p gpurun_out
CS=/usr/local/cuda/bin/compute-sanitizer
$CS --tool racecheck --racecheck-report all --print-limit 200 python scripts/exp/race_q18.py > gpurun_out/racecheck_v3.txt 2>&1; echo "racecheck rc=$?"
H2TAP_ORDER_CARRY=0 $CS --tool racecheck --racecheck-report all --print-limit 100 python scripts/exp/race_q18.py > gpurun_out/racecheck_rowid.txt 2>&1; echo "racecheck rowid rc=$?"
$CS --tool memcheck python scripts/exp/race_q18.py > gpurun_out/memcheck_v3.txt 2>&1; echo "memcheck rc=$?"
for f in gpurun_out/racecheck_v3.txt gpurun_out/racecheck_rowid.txt gpurun_out/memcheck_v3.txt; do echo "== $f"; tail -n 3 $f; done
