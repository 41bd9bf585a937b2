#!/bin/bash
# Confirmation of the committed build: GPU suite, smoke(), bench line, and an
# lbm dequeue-chunk sweep (RESOLVE overhead on very short VGs).
cd "$GRAFT_REPO_ROOT"; O=gpurun_out/confirm; mkdir -p $O
timeout 900 python -m pytest tests -m gpu -q --timeout 600 -p no:cacheprovider > $O/gputest.log 2>&1; echo "pytest rc=$?" >> $O/gputest.log
timeout 300 python -c "import __graft_entry__ as g; g.smoke(); print('smoke ok')" > $O/smoke.log 2>&1; echo "smoke rc=$?" >> $O/smoke.log
timeout 600 python bench.py --out $O/bench_c2.json > $O/bench_c2.log 2>&1; echo "bench rc=$?" >> $O/bench_c2.log
for c in 1 2 4; do
  echo "== chunk $c" >> $O/lbm_chunk.log
  ACCEL_CHUNK_OVERRIDE=lbm:$c timeout 300 python scripts/isolated.py --reps 8 --chunk $c lbm >> $O/lbm_chunk.log 2>&1
done
tail -2 $O/gputest.log; tail -1 $O/smoke.log; tail -c 300 $O/bench_c2.log
