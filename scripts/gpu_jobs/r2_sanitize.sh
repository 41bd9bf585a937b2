#!/bin/bash
# compute-sanitizer memcheck / racecheck / synccheck over a tiny mix of
# mop, bfs, stencil (cp.async and TMA), histo (16 K bins), tpacf and the
# one-step tcgen05 sgemm, NATIVE / STATIC / RESOLVE (scripts/sanitize.py)
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for t in memcheck racecheck synccheck; do
  timeout 1500 compute-sanitizer --tool $t python scripts/sanitize.py > gpurun_out/san_$t.log 2>&1
  echo "$t rc=$?" >> gpurun_out/san_$t.log
done
