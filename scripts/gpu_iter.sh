#!/bin/bash
# one iteration on the GPU: GPU parity tests, quick bench + per-role trace of each tcgen05 variant
set -u
mkdir -p gpurun_out
TAG=${1:-x}
python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > gpurun_out/build_${TAG}.log 2>&1
echo "== tests"; timeout 1200 python -m pytest tests -q -m gpu --timeout 600 -x ${PYTEST_K:-} > gpurun_out/tests_${TAG}.log 2>&1; echo "rc=$?"; tail -3 gpurun_out/tests_${TAG}.log
B="python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu-baseline --no-alt --engine tc ${EXTRA:-}"
G='"value": [0-9.]*\|"launch_ms": [0-9.]*\|"executed_frac": [0-9.]*\|fallback_rotations": [0-9]*\|"kernel": "[^"]*"'
for V in ${VARIANTS:-1 2}; do
  echo "== V$V"; timeout 300 $B --tc-variant $V > gpurun_out/bench_${TAG}_v${V}.log 2>&1; grep -o "$G" gpurun_out/bench_${TAG}_v${V}.log | tr '\n' ' '; echo
  DOCK_TC_TRACE=1 timeout 300 python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --no-alt --engine tc --tc-variant $V ${EXTRA:-} > gpurun_out/trace_${TAG}_v${V}.log 2>&1
  grep TCTRACE gpurun_out/trace_${TAG}_v${V}.log | tail -1
done
