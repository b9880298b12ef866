#!/bin/bash
# scheduler segment cost sweep (prod, tcgen05 variant 1, occupancy schedule) + trace
set -u
mkdir -p gpurun_out
TAG=${1:-x}
python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > gpurun_out/build_${TAG}.log 2>&1
B="python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-alt --engine tc"
G='"value": [0-9.]*\|"launch_ms": [0-9.]*\|"ksteps_per_row_executed": [0-9.]*\|"ms_per_step": [0-9.]*'
for E in ${COSTS:-12}; do
  echo "== cost $E"
  DOCK_TC_SEG_COST=$E timeout 300 $B > gpurun_out/bench_${TAG}_e$E.log 2>&1
  grep -o "$G" gpurun_out/bench_${TAG}_e$E.log | tr '\n' ' '; echo
  DOCK_TC_SEG_COST=$E DOCK_TC_TRACE=1 timeout 300 python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu-baseline --no-alt --engine tc > gpurun_out/trace_${TAG}_e$E.log 2>&1
  grep TCTRACE gpurun_out/trace_${TAG}_e$E.log | tail -1 | grep -o '"mma_wait[a-z_]*": [0-9]*\|"inserts_per_tile_lane": [0-9.]*\|"epi_wait_tm_full": [0-9]*\|"epi_total": [0-9]*' | tr '\n' ' '; echo
done
