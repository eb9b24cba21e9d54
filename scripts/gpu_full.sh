mkdir -p gpurun_out
TAG=${1:-r01}
timeout 900 python -m pytest tests -m gpu -q --timeout 400 -rf -x 2>&1 | tail -5 | tee gpurun_out/pytest_gpu.txt
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -2
timeout 600 python bench.py 2>&1 | tail -3 | tee gpurun_out/bench.txt
bash scripts/ncu_round.sh $TAG
