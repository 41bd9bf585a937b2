timeout 1200 python -m pytest tests -m gpu -q -x 2>&1 | tail -2
for i in 1 2; do timeout 300 python -m pytest tests/test_gpu_resolve.py -q -x 2>&1 | tail -1; done
python scripts/isolated.py stencil histo bfs cutcp tpacf spmv sgemm mriq --reps 3 2>&1 | python -c "
import sys,json
for line in sys.stdin:
    t,j=line.split(' ',1); j=json.loads(j); print(t, 'ovh static %.3f resolve %.3f'%(j['overhead'], j.get('overhead_resolve',0)), 'occ', j['occ'])"
timeout 900 python bench.py --steps 5 --warmup 3 --out gpurun_out/bench_c2_r18.json 2>&1 | tail -1 | python -c "
import sys,json; j=json.loads(sys.stdin.read()); print(json.dumps({k:j[k] for k in ('value','ms_per_step','e2e','gpu_launches')})); s=j['sharing']; print({k:s[k] for k in ('unfairness_shared','unfairness_native','stp_shared','stp_native','throughput_speedup','dispatch_overhead','T_s_ms_shared','T_a_ms')}); print(s['other_policy']); print(j['roofline'])"
