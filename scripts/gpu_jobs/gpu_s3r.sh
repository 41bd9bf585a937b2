# session 3r: idle top-up stream selection -- suite, C4, C2 bench
export ACCEL_DEBUG_OFF=1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite9.log 2>&1; tail -2 gpurun_out/gpu_suite9.log; grep FAILED gpurun_out/gpu_suite9.log
for i in 1 2; do timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve --out gpurun_out/c4_r$i.json > gpurun_out/c4_r$i.log 2>&1; grep -E "^resolve " gpurun_out/c4_r$i.log | cut -c1-330; done
timeout 600 python bench.py --steps 10 --warmup 3 --calib-reps 3 --no-cpu-baseline --out gpurun_out/bench_r.json > gpurun_out/bench_r.log 2>&1
python - <<'PY'
import json
j = json.load(open("gpurun_out/bench_r.json")); s = j["sharing"]
print(j["value"], {k: round(s[k], 3) for k in ["unfairness_shared", "unfairness_native", "stp_ratio", "throughput_speedup"]}, {k: round(v, 2) for k, v in s["T_s_ms_shared"].items()})
PY
