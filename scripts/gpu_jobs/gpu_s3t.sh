# session 3t: early GEMM capped at half the device -- suite, C3 (self-pair sgemm), f2, C2 bench
export ACCEL_DEBUG_OFF=1 ACCEL_SYNC_TIMEOUT_S=60
timeout 1200 python -m pytest tests -m gpu -q > gpurun_out/gpu_suite11.log 2>&1; tail -2 gpurun_out/gpu_suite11.log; grep -E "FAILED|STUCK" gpurun_out/gpu_suite11.log | head
timeout 600 python scripts/mixes.py --config c3 --reps 3 --modes resolve,static --out gpurun_out/c3_pairs.json > gpurun_out/c3.log 2>&1; echo "c3 rc=$?"; grep SUMMARY gpurun_out/c3.log | cut -c1-420
timeout 600 python scripts/mixes.py --config f2 --k 4 --n 40 --reps 3 --modes resolve,static --out gpurun_out/f2_k4.json > gpurun_out/f2.log 2>&1; echo "f2 rc=$?"; grep SUMMARY gpurun_out/f2.log | cut -c1-420
timeout 600 python scripts/mixes.py --config c4 --reps 5 --modes resolve,static --out gpurun_out/c4.json > gpurun_out/c4.log 2>&1; echo "c4 rc=$?"; grep -E "^(native|resolve|static) " gpurun_out/c4.log | cut -c1-120
timeout 600 python bench.py --steps 10 --warmup 3 --out gpurun_out/bench_c2.json > gpurun_out/bench_c2.log 2>&1; echo "bench rc=$?"
python - <<'PY'
import json
j = json.load(open("gpurun_out/bench_c2.json")); s = j["sharing"]
print(j["value"], j["e2e"]["value"], {k: round(s[k], 3) for k in ["unfairness_shared", "unfairness_native", "stp_ratio", "throughput_speedup"]}, {k: round(v, 2) for k, v in s["T_s_ms_shared"].items()})
PY
