#!/bin/bash
# quick GPU iteration: parity tests + tcgen05 experiments (+ optional ncu)
set -u
mkdir -p gpurun_out
TAG=${1:-x}
echo "== tests"; timeout 900 python -m pytest tests -q -m gpu --timeout 600 -x > gpurun_out/tests_${TAG}.log 2>&1; echo "rc=$?"; tail -3 gpurun_out/tests_${TAG}.log
NCU=${NCU:-1} bash scripts/tc_exp.sh $TAG
