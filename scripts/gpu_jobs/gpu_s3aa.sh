# session 3aa: FAIR with device-time elapsed and cost-weighted progress
export ACCEL_DEBUG_OFF=1 ACCEL_SYNC_TIMEOUT_S=60
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite14.log 2>&1; tail -2 gpurun_out/gpu_suite14.log; grep -E "FAILED|STUCK" gpurun_out/gpu_suite14.log | head
for i in 1 2; do
  timeout 400 python bench.py --policy fair --steps 10 --warmup 3 --calib-reps 3 --no-cpu-baseline --out gpurun_out/bench_fair$i.json > gpurun_out/bench_fair$i.log 2>&1; echo "rc=$?"
  python - $i <<'PY'
import json, sys
j = json.load(open(f"gpurun_out/bench_fair{sys.argv[1]}.json")); s = j["sharing"]
print("fair", j["value"], {k: round(s[k], 3) for k in ["unfairness_shared", "unfairness_native", "stp_ratio", "throughput_speedup"]}, {k: round(v, 2) for k, v in s["T_s_ms_shared"].items()},
      "resolve", {k: round(v, 3) for k, v in s["other_policies"]["resolve"].items() if not isinstance(v, dict)})
PY
done
timeout 600 python scripts/mixes.py --config c3 --reps 3 --modes resolve,fair --out gpurun_out/c3_fair.json > gpurun_out/c3_fair.log 2>&1; echo "c3 rc=$?"; grep SUMMARY gpurun_out/c3_fair.log | cut -c1-900
timeout 600 python scripts/mixes.py --config f2 --k 4 --n 40 --reps 3 --modes resolve,fair --out gpurun_out/f2_fair.json > gpurun_out/f2_fair.log 2>&1; echo "f2 rc=$?"; grep SUMMARY gpurun_out/f2_fair.log | cut -c1-900
