#!/bin/bash
# occupancy-schedule iteration: new + tcgen05 parity tests, prod bench per schedule mode, trace
set -u
mkdir -p gpurun_out
TAG=${1:-s}
python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > gpurun_out/build_${TAG}.log 2>&1
echo "== tests"
timeout 900 python -m pytest tests/test_gpu_parity.py -q -m gpu --timeout 600 -x -k "${TESTS:-occupancy or dynamic_scheduler or fallback_path or invariance or prod_config or poses_mid or integer}" > gpurun_out/tests_${TAG}.log 2>&1; echo "rc=$?"; tail -3 gpurun_out/tests_${TAG}.log
B="python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-alt --engine tc"
G='"value": [0-9.]*\|"launch_ms": [0-9.]*\|"executed_frac": [0-9.]*\|"ksteps_per_row_executed": [0-9.]*'
for S in ${SCHEDS:-2 1 0}; do
  echo "== prod sched $S"
  timeout 300 $B --tc-schedule $S > gpurun_out/bench_${TAG}_s$S.log 2>&1
  grep -o "$G" gpurun_out/bench_${TAG}_s$S.log | tr '\n' ' '; echo
  DOCK_TC_TRACE=1 timeout 300 python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu-baseline --no-alt --engine tc --tc-schedule $S > gpurun_out/trace_${TAG}_s$S.log 2>&1
  grep TCTRACE gpurun_out/trace_${TAG}_s$S.log | tail -1
done
