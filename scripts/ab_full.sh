# the batch's full pass (Q6 + Q1 + Q18 probe in one order_line read): A/B of variants / knobs.
# args: tag[=lib][,ENV=V...]  e.g.  on  off  pg2a  pg2a,H2TAP_Q1_SIDE=0
mkdir -p gpurun_out
[ -z "$NOTEST" ] && timeout 900 python -m pytest tests/test_gpu_parity.py -q -x --timeout 400 -k "full_pass or shared or w100_bench" 2>&1 | tail -3
for spec in "$@"; do
  IFS=, read -ra parts <<< "$spec"
  tag=${parts[0]}; envs=("${parts[@]:1}")
  case $tag in
    off) envs+=(H2TAP_FULL_PASS=0) ;;
    on) ;;
    *) envs+=(H2TAP_LIB=variants/libh2tap_$tag.so) ;;
  esac
  name=$(echo "$spec" | tr ',=' '__')
  env "${envs[@]}" timeout 300 python bench.py --no-cpu-baseline --no-c1 --steps 20 --e2e-steps 2 --inc-neworders 0 2>&1 | tail -1 > gpurun_out/full_$name.json
  python -c "
import json; d=json.load(open('gpurun_out/full_$name.json'))
print('$spec', round(d['ms_per_step'],4), d['roofline']['kernel'], d['roofline']['frac'], {k: round(v['ms']*1000,1) for k, v in d['kernels'].items()})" || tail -5 gpurun_out/full_$name.json
done
