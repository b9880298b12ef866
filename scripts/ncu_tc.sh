#!/bin/bash
# one ncu --set full capture of k_corr_tc (variant ${V:-1}) with source-level stall sampling, exported to CSV
set -u
mkdir -p gpurun_out
TAG=${1:-x}
B="python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu-baseline --no-alt --engine tc --tc-variant ${V:-1}"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_corr_tc -s 1 -c 1 \
    -o gpurun_out/ncu_${TAG} -f $B > gpurun_out/ncu_${TAG}.log 2>&1
echo "ncu rc=$?"
ncu -i gpurun_out/ncu_${TAG}.ncu-rep --page raw --csv > gpurun_out/ncu_${TAG}_raw.csv 2>/dev/null
ncu -i gpurun_out/ncu_${TAG}.ncu-rep --page source --csv > gpurun_out/ncu_${TAG}_source.csv 2>/dev/null
rm -f gpurun_out/ncu_${TAG}.ncu-rep
