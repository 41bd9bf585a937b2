# tpacf: float4 Q tile + first two binary-search levels in registers: parity, isolated timing, C2 bench x2
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python -m paper_conf_cgo_margiolaso16_b200.build --force > /dev/null 2>&1
timeout 600 python -m pytest tests -m gpu -q -x -k "tpacf or config2 or fig2 or mix" 2>&1 | tail -2
timeout 120 python scripts/isolated.py tpacf --reps 5 2>&1 | python -c "
import sys,json
for l in sys.stdin:
  if l.startswith('tpacf'): d=json.loads(l[6:]); print('  isolated native %.3f pers %.3f res %.3f ovh %.3f regs %s occ %s' % (d['native']['elapsed_ms'], d['persistent']['elapsed_ms'], d['persistent_resolve']['elapsed_ms'], d['overhead'], d['regs'], d['occ']))"
for rep in 1 2; do
  timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu-baseline > gpurun_out/bench_s4k_$rep.log 2>&1
  python -c "
import json; d=json.loads(open('gpurun_out/bench_s4k_$rep.log').read().strip().splitlines()[-1]); s=d['sharing']
print('  U', round(s['unfairness_shared'],3), 'Unat', round(s['unfairness_native'],3), 'STPr', round(s['stp_ratio'],3), 'thr', round(s['throughput_speedup'],3), 'mixes/s', round(d['value'],1), {k: round(s['T_s_ms_shared'][k]/s['T_a_ms'][k],2) for k in s['T_a_ms']}, s['T_a_ms']['tpacf'])"
done
