# session 3g: which RESOLVE piece costs per launch (isolated, measurement-only ablations)
export ACCEL_DEBUG_OFF=1
for ab in 0 8 16 31; do
  ACCEL_ABLATE=$ab timeout 300 python scripts/isolated.py stencil spmv --reps 7 --policy both > gpurun_out/ablg_$ab.log 2>&1
  python - "$ab" <<'PY'
import json, sys
for line in open(f"gpurun_out/ablg_{sys.argv[1]}.log"):
    if " {" not in line: print(line[:200]); continue
    t, j = line.split(" ", 1); j = json.loads(j)
    print("ablate", sys.argv[1], t, {k: round(v, 4) for k, v in j.items() if k.startswith("overhead")}, {k: round(v["elapsed_ms"], 3) for k, v in j.items() if isinstance(v, dict)})
PY
done
for mix in sgemm,spmv spmv,sgemm sgemm,cutcp; do
  for m in native resolve; do echo "== $mix $m"; timeout 120 python scripts/timeline.py $m $mix 2>&1 | tail -40; done
done
