# session 3c: Ctl line split -> RESOLVE overhead; GPU suite; default bench; f1 weight sweep on C2
export ACCEL_DEBUG_OFF=1
for ab in 0 4; do
  ACCEL_ABLATE=$ab timeout 300 python scripts/isolated.py stencil spmv histo bfs tpacf cutcp --reps 5 --policy both > gpurun_out/ablc_$ab.log 2>&1
  python - "$ab" <<'PY'
import json, sys
for line in open(f"gpurun_out/ablc_{sys.argv[1]}.log"):
    if " {" not in line: print(line[:200]); continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print("ablate", sys.argv[1], t, {k: round(v, 4) for k, v in j.items() if k.startswith("overhead")}, {k: round(v["elapsed_ms"], 3) for k, v in j.items() if isinstance(v, dict)})
PY
done
timeout 1500 python -m pytest tests -m gpu -q -rf > gpurun_out/gpu_suite.log 2>&1; tail -4 gpurun_out/gpu_suite.log
timeout 600 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1; tail -c 300 gpurun_out/bench_c2.log
timeout 900 python scripts/weights.py --reps 5 --out gpurun_out/weights_c2.json > gpurun_out/weights_c2.log 2>&1; cat gpurun_out/weights_c2.log | cut -c1-250
