# session 3: GPU suite, RESOLVE admission overlap (isolated overhead), default bench, FAIR hang probe
export ACCEL_DEBUG_OFF=1
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -6
timeout 600 python scripts/isolated.py stencil histo bfs spmv cutcp tpacf --reps 3 --policy all > gpurun_out/iso2.log 2>&1
python - <<'PY'
import json
for line in open("gpurun_out/iso2.log"):
    if " {" not in line: print(line[:300]); continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print(t, {k: round(v, 3) for k, v in j.items() if k.startswith("overhead")})
PY
timeout 600 python bench.py --steps 5 --warmup 3 --calib-reps 3 --no-cpu-baseline --out gpurun_out/bench_res2.json > gpurun_out/bench_res2.log 2>&1; tail -c 200 gpurun_out/bench_res2.log
ACCEL_DEBUG=1 timeout 300 python bench.py --policy fair --steps 3 --warmup 3 --calib-reps 2 --no-cpu-baseline --hang-dump-s 150 > gpurun_out/bench_fairdbg.log 2>&1; echo "fair rc=$?"; tail -c 3000 gpurun_out/bench_fairdbg.log
