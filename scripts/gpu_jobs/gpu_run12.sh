timeout 1200 python -m pytest tests -m gpu -q -x 2>&1 | tail -4
timeout 600 python scripts/isolated.py stencil histo bfs cutcp tpacf spmv sgemm mriq --reps 3 2>&1 | tail -12
timeout 900 python bench.py --steps 5 --warmup 3 --no-cpu-baseline --out gpurun_out/bench_c2_r12.json 2>&1 | tail -1 | python -c "
import sys,json; j=json.loads(sys.stdin.read()); print(json.dumps({k:j[k] for k in ('value','ms_per_step')})); s=j['sharing']; print({k:s[k] for k in ('unfairness_shared','unfairness_native','stp_shared','stp_native','throughput_speedup','dispatch_overhead','T_s_ms_shared','T_a_ms','quotas_last_step')}); print(s['other_policy']); print(j['roofline'])"
