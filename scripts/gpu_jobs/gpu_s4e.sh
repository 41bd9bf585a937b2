# cutcp register cap (min CTAs/SM 8 -> 10, 62 -> <=48 regs): parity, isolated timing, C2 bench (U, STP, throughput)
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
for mb in 10 8; do
  ACCEL_NVCC_EXTRA="-DCUTCP_MINB=$mb" python -m paper_conf_cgo_margiolaso16_b200.build --force > /dev/null 2>&1 || echo "build fail minb=$mb"
  echo "minb=$mb"
  timeout 600 python -m pytest tests -m gpu -q -x -k "cutcp or config2 or fig2" 2>&1 | tail -2
  timeout 120 python scripts/isolated.py cutcp --reps 5 2>&1 | cut -c1-900
  timeout 600 python bench.py --steps 10 --warmup 3 --no-cpu-baseline --out gpurun_out/bench_minb$mb.json > gpurun_out/bench_minb$mb.log 2>&1
  python -c "
import json; d=json.loads(open('gpurun_out/bench_minb$mb.log').read().strip().splitlines()[-1]); s=d['sharing']
print('U', round(s['unfairness_shared'],3), 'Unat', round(s['unfairness_native'],3), 'STPr', round(s['stp_ratio'],3), 'thr', round(s['throughput_speedup'],3), 'mixes/s', round(d['value'],1), {k: round(s['T_s_ms_shared'][k]/s['T_a_ms'][k],2) for k in s['T_a_ms']}, s['quotas_last_step']['cutcp'])"
done
