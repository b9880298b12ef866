#!/bin/bash
# tcgen05 engine timeline decomposition: per-role cycle counters (DOCK_TC_TRACE) (the round-1 epilogue ablations were removed from the product kernels)
set -u
mkdir -p gpurun_out
TAG=${1:-x}
python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > gpurun_out/build_${TAG}.log 2>&1
B="python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --no-alt --engine tc"
G='"value": [0-9.]*\|"launch_ms": [0-9.]*\|"executed_frac": [0-9.]*'
for V in ${VARIANTS:-1 4}; do for D in 0 1 2; do
  echo "== V$V dbg$D"
  DOCK_TC_TRACE=1 timeout 300 $B --tc-variant $V > gpurun_out/trace_${TAG}_v${V}_d${D}.log 2>&1
  grep -o "$G" gpurun_out/trace_${TAG}_v${V}_d${D}.log | tr '\n' ' '; echo
  grep TCTRACE gpurun_out/trace_${TAG}_v${V}_d${D}.log | tail -1
done; done
