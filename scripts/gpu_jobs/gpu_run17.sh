timeout 1200 python -m pytest tests -m gpu -q -x 2>&1 | tail -2
python scripts/isolated.py stencil histo bfs cutcp tpacf spmv sgemm mriq --reps 3 2>&1 | python -c "
import sys,json
for line in sys.stdin:
    t,j=line.split(' ',1); j=json.loads(j); print(t, 'ovh static %.3f resolve %.3f'%(j['overhead'], j.get('overhead_resolve',0)), 'occ', j['occ'], {k:round(v.get('GBps_mean', v.get('TFLOPs_mean',0)),1) for k,v in j.items() if isinstance(v,dict)})"
timeout 900 python bench.py --steps 5 --warmup 3 --out gpurun_out/bench_c2_r17.json 2>&1 | tail -1 | python -c "
import sys,json; j=json.loads(sys.stdin.read()); print(json.dumps({k:j[k] for k in ('value','ms_per_step','e2e','gpu_launches')})); s=j['sharing']; print({k:s[k] for k in ('unfairness_shared','unfairness_native','stp_shared','stp_native','throughput_speedup','dispatch_overhead','T_s_ms_shared','T_a_ms')}); print(s['other_policy']); print(j['roofline'])"
