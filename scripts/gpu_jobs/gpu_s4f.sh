# cutcp register cap sweep, repeated C2 bench runs (noise): min CTAs/SM 9, 10, 8
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
for mb in 9 10 8; do
  ACCEL_NVCC_EXTRA="-DCUTCP_MINB=$mb" python -m paper_conf_cgo_margiolaso16_b200.build --force > /dev/null 2>&1 || echo "build fail minb=$mb"
  echo "minb=$mb"
  timeout 120 python scripts/isolated.py cutcp --reps 5 2>&1 | python -c "
import sys,json
for l in sys.stdin:
  if l.startswith('cutcp'): d=json.loads(l[6:]); print('  isolated native %.3f pers %.3f res %.3f ovh %.3f regs %s occ %s' % (d['native']['elapsed_ms'], d['persistent']['elapsed_ms'], d['persistent_resolve']['elapsed_ms'], d['overhead'], d['regs'], d['occ']))"
  for rep in 1 2 3; do
  timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu-baseline > gpurun_out/bench_minb${mb}_$rep.log 2>&1
  python -c "
import json; d=json.loads(open('gpurun_out/bench_minb${mb}_$rep.log').read().strip().splitlines()[-1]); s=d['sharing']
print('  U', round(s['unfairness_shared'],3), 'Unat', round(s['unfairness_native'],3), 'STPr', round(s['stp_ratio'],3), 'thr', round(s['throughput_speedup'],3), 'mixes/s', round(d['value'],1), {k: round(s['T_s_ms_shared'][k]/s['T_a_ms'][k],2) for k in s['T_a_ms']}, s['quotas_last_step']['cutcp'])"
  done
done
