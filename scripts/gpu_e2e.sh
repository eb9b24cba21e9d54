# refresh back-pressure: snapshot/refresh GPU tests + bench e2e (serial vs pipelined), twice
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_updates.py tests/test_gpu_mixed.py tests/test_gpu_zero_copy.py -q -x --timeout 400 2>&1 | tail -2
for v in 1 2; do
  timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu-baseline 2>&1 | tail -1 > gpurun_out/bench_e2e.json
  python -c "import json; d=json.load(open('gpurun_out/bench_e2e.json')); e=d['e2e']; print('run$v', d['ms_per_step'], e['serial_ms_per_step'], e['pipelined_ms_per_step'], e['pipelined_epoch_lag'])"
done
