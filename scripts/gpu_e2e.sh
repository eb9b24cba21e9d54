# async borrowed loads: parity test + bench (e2e serial vs pipelined)
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -q -x --timeout 300 -k "async_borrowed or snapshot or concurrent" 2>&1 | tail -3
timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu-baseline 2>&1 | tail -1 > gpurun_out/bench_e2e.json
python -c "import json; d=json.load(open('gpurun_out/bench_e2e.json')); print(d['ms_per_step'], d['e2e'])"
