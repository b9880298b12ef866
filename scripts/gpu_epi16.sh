#!/bin/bash
B="python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-alt --engine tc"
G='"value": [0-9.]*\|"launch_ms": [0-9.]*'
DOCK_NVCC_DEFS="-DDOCK_TC_NEPI_MAX=16" python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > gpurun_out/build_epi.log 2>&1 || tail -5 gpurun_out/build_epi.log
for E in 8 16; do echo -n "epi $E: "; DOCK_NVCC_DEFS="-DDOCK_TC_NEPI_MAX=16" timeout 300 $B --tc-epi $E 2>&1 | grep -o "$G" | tr '\n' ' '; echo; done
DOCK_NVCC_DEFS="-DDOCK_TC_NEPI_MAX=16" DOCK_TC_TRACE=1 timeout 300 python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu-baseline --no-alt --engine tc --tc-epi 16 2>&1 | grep TCTRACE | tail -1 | grep -o '"mma_wait[a-z_]*": [0-9]*\|"epi_wait_tm_full": [0-9]*\|"epi_total": [0-9]*' | tr '\n' ' '
