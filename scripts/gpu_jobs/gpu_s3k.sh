# session 3k: static first chunks for main grids -- suite, isolated overhead, VG trace, C2 bench
export ACCEL_DEBUG_OFF=1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite5.log 2>&1; tail -3 gpurun_out/gpu_suite5.log; grep FAILED gpurun_out/gpu_suite5.log
timeout 600 python scripts/isolated.py stencil histo bfs spmv sgemm mriq cutcp tpacf --reps 5 --policy both > gpurun_out/iso5.log 2>&1
python - <<'PY'
import json
for line in open("gpurun_out/iso5.log"):
    if " {" not in line: print(line[:200]); continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print(t, {k: round(v, 4) for k, v in j.items() if k.startswith("overhead")}, {k: round(v["elapsed_ms"], 3) for k, v in j.items() if isinstance(v, dict)})
PY
timeout 300 python scripts/vg_trace.py stencil --policy resolve 2>&1 | grep -E "launches|gap_us" | cut -c1-400
timeout 600 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1; tail -c 200 gpurun_out/bench_c2.log
