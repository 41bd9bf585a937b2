#!/bin/bash
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
for L in ${LIBS:-default}; do
  if [ "$L" = default ]; then unset ACCEL_LIB; else export ACCEL_LIB=$PWD/$L; fi
  tag=$(basename $L .so)
  ACCEL_DEBUG=1 timeout 300 python scripts/c4_debug.py > gpurun_out/c4dbg_$tag.log 2>&1
  echo "== $tag"; grep -A9 "rep 2" gpurun_out/c4dbg_$tag.log | grep "T_s"
done
