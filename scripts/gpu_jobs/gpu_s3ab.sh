# session 3ab: final check -- suite, smoke, default bench (the driver's command)
export ACCEL_DEBUG_OFF=1
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite15.log 2>&1; tail -2 gpurun_out/gpu_suite15.log; grep -E "FAILED" gpurun_out/gpu_suite15.log | head
timeout 300 python -c "import __graft_entry__ as g; g.smoke()" 2>&1 | tail -1
SECONDS=0; timeout 900 python bench.py > gpurun_out/bench_default.log 2>&1; tail -1 gpurun_out/bench_default.log | cut -c1-100; echo "bench wall $SECONDS s"
python - <<'PY'
import json
line = [l for l in open("gpurun_out/bench_default.log") if l.startswith("{")][-1]
j = json.loads(line); s = j["sharing"]
print(j["value"], j["e2e"]["value"], {k: round(s[k], 3) for k in ["unfairness_shared", "unfairness_native", "stp_ratio", "throughput_speedup"]}, j["roofline"]["frac"], j["cpu_baseline"]["value"], j["clocks"])
json.dump(j, open("gpurun_out/bench_default.json", "w"))
PY
