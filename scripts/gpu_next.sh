# NEXT-2/3/4 round evidence: GPU parity of Q3, layout scans and zero-copy snapshots; NEXT-2 bench,
# layout bench, zero-copy bench; ncu of the layout kernels (1 GB table).
mkdir -p gpurun_out
TAG=${1:-r01}
timeout 900 python -m pytest tests/test_gpu_q3.py tests/test_gpu_layout.py tests/test_gpu_zero_copy.py -q --timeout 600 2>&1 | tail -15 | tee gpurun_out/pytest_next_${TAG}.txt
timeout 600 python scripts/ch_bench.py --out gpurun_out/ch_bench_${TAG}.json > /dev/null 2>&1; tail -c 300 gpurun_out/ch_bench_${TAG}.json
timeout 900 python scripts/layout_bench.py --out gpurun_out/layout_bench_${TAG}.json > gpurun_out/layout_bench_${TAG}.log 2>&1; tail -2 gpurun_out/layout_bench_${TAG}.log
timeout 900 python scripts/zero_copy_bench.py --out gpurun_out/zero_copy_${TAG}.json 2>&1 | tail -3
if [ "${NCU:-1}" = 1 ]; then
timeout 600 ncu --set full --clock-control none -k regex:'dsm_sum|pax_sum|nsm_sum' -c 15 -o gpurun_out/layout_${TAG} -f \
    python scripts/layout_bench.py --rows 16777216 --small-rows 16777216 --host-rows 4194304 --steps 1 > gpurun_out/layout_ncu_${TAG}.log 2>&1
fi
echo done
