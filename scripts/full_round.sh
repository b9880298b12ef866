#!/bin/bash
# full bench line + ncu launch list and full capture for both engines
set -u
mkdir -p gpurun_out
TAG=${1:-r01}
echo "== bench"; timeout 900 python bench.py > gpurun_out/bench_${TAG}.log 2>&1; echo "rc=$?"; tail -c 3000 gpurun_out/bench_${TAG}.log
bash scripts/profile.sh ${TAG} tc
bash scripts/profile.sh ${TAG} ffma
