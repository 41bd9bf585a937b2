#!/bin/bash
# one compute-sanitizer tool per call (TOOL=memcheck|racecheck|synccheck) over scripts/sanitize.py
cd "$GRAFT_REPO_ROOT"; mkdir -p gpurun_out
timeout 1500 compute-sanitizer --tool ${TOOL:-memcheck} python scripts/sanitize.py > gpurun_out/san_${TOOL:-memcheck}.log 2>&1
echo "${TOOL:-memcheck} rc=$?" >> gpurun_out/san_${TOOL:-memcheck}.log
tail -4 gpurun_out/san_${TOOL:-memcheck}.log
