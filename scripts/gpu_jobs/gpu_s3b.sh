# session 3b: RESOLVE ablations (isolated), GPU suite with per-test timeouts (verbose), default bench
export ACCEL_DEBUG_OFF=1
for ab in 0 1 2 4 7; do
  ACCEL_ABLATE=$ab timeout 300 python scripts/isolated.py stencil spmv --reps 5 --policy both > gpurun_out/abl_$ab.log 2>&1
  python - "$ab" <<'PY'
import json, sys
for line in open(f"gpurun_out/abl_{sys.argv[1]}.log"):
    if " {" not in line: print(line[:200]); continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print("ablate", sys.argv[1], t, {k: round(v, 4) for k, v in j.items() if k.startswith("overhead")}, {k: round(v["elapsed_ms"], 3) for k, v in j.items() if isinstance(v, dict)})
PY
done
timeout 2000 python -m pytest tests -m gpu -q -rf --durations=15 > gpurun_out/gpu_suite.log 2>&1; tail -40 gpurun_out/gpu_suite.log
timeout 600 python bench.py --steps 5 --warmup 3 --calib-reps 3 --no-cpu-baseline --out gpurun_out/bench_res3.json > gpurun_out/bench_res3.log 2>&1; tail -c 300 gpurun_out/bench_res3.log
