#!/bin/bash
# compile-time variants of k_corr_tc (DOCK_NVCC_DEFS) timed on the prod bench (kernel ms); experiments only
set -u
mkdir -p gpurun_out
TAG=${1:-v}
B="python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-alt --engine tc"
G='"value": [0-9.]*\|"launch_ms": [0-9.]*\|"ksteps_per_row_executed": [0-9.]*\|"ms_per_step": [0-9.]*'
for V in "${VARIANTS[@]:-}"; do :; done
IFS=';' read -ra VS <<< "${DEFS:-}"
for D in "${VS[@]}"; do
  echo "== defs [$D]"
  DOCK_NVCC_DEFS="$D" python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > gpurun_out/build_${TAG}.log 2>&1 || { tail -5 gpurun_out/build_${TAG}.log; continue; }
  for S in ${SCHEDS:-0}; do
    DOCK_NVCC_DEFS="$D" timeout 300 $B --tc-schedule $S > gpurun_out/bench_${TAG}.log 2>&1
    echo -n "sched $S: "; grep -o "$G" gpurun_out/bench_${TAG}.log | tr '\n' ' '; echo
  done
done
