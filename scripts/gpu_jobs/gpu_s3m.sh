# session 3m: interleaved group enqueue -- suite, C2 bench, timeline, C3, C4
export ACCEL_DEBUG_OFF=1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite6.log 2>&1; tail -2 gpurun_out/gpu_suite6.log; grep FAILED gpurun_out/gpu_suite6.log
timeout 600 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1
python - <<'PY'
import json
j = json.load(open("gpurun_out/bench_c2.json")); s = j["sharing"]
print(j["value"], {k: round(s[k], 3) for k in ["unfairness_shared", "unfairness_native", "stp_shared", "stp_native", "stp_ratio", "throughput_speedup"]},
      {k: round(v, 2) for k, v in s["T_s_ms_shared"].items()}, {k: round(v, 2) for k, v in s["T_s_ms_native"].items()}, s["other_policies"]["static"]["unfairness"], s["other_policies"]["static"]["stp"])
PY
timeout 120 python scripts/timeline.py resolve c2 2>&1 | grep "T(s)"
timeout 120 python scripts/timeline.py native c2 2>&1 | grep "T(s)"
timeout 900 python scripts/mixes.py --config c3 --reps 3 --modes resolve,static --out gpurun_out/c3_pairs.json > gpurun_out/c3.log 2>&1; grep SUMMARY gpurun_out/c3.log
timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve,static --out gpurun_out/c4.json > gpurun_out/c4.log 2>&1; grep SUMMARY gpurun_out/c4.log | cut -c1-300
