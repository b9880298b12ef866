#!/bin/bash
# tcgen05 engine experiments: Q=4/NBUF=1 vs Q=2/NBUF=2, then one ncu capture of k_corr_tc.
set -u
mkdir -p gpurun_out
TAG=${1:-x}
B="python bench.py --steps 3 --warmup 2 --no-e2e --no-cpu-baseline --no-alt --engine tc"
G='"value": [0-9.]*\|"launch_ms": [0-9.]*\|"executed_frac": [0-9.]*\|fallback_rotations": [0-9]*'
echo "== V1"; timeout 300 $B --tc-variant 1 > gpurun_out/tc_${TAG}_q4.log 2>&1; grep -o "$G" gpurun_out/tc_${TAG}_q4.log
echo "== V1 epi8"; timeout 300 $B --tc-variant 1 --tc-epi 8 > gpurun_out/tc_${TAG}_e8.log 2>&1; grep -o "$G" gpurun_out/tc_${TAG}_e8.log
echo "== V2"; timeout 300 $B --tc-variant 2 > gpurun_out/tc_${TAG}_q2.log 2>&1; grep -o "$G" gpurun_out/tc_${TAG}_q2.log
echo "== FFMA"; timeout 300 python bench.py --steps 3 --warmup 2 --no-e2e --no-cpu-baseline --no-alt --engine ffma > gpurun_out/ffma_${TAG}.log 2>&1; grep -o '"value": [0-9.]*\|"launch_ms": [0-9.]*\|"frac": [0-9.]*' gpurun_out/ffma_${TAG}.log
if [ "${NCU:-1}" = "1" ]; then
timeout 900 ncu --set full --clock-control none --import-source on -k regex:${KRE:-k_corr_tc} -s 1 -c 1 \
    -o gpurun_out/tc_${TAG} -f $B ${NCU_ARGS:-} > gpurun_out/tc_${TAG}_ncu.log 2>&1
echo "ncu rc=$?"
ncu -i gpurun_out/tc_${TAG}.ncu-rep --page raw --csv > gpurun_out/tc_${TAG}_raw.csv 2>/dev/null
ncu -i gpurun_out/tc_${TAG}.ncu-rep --page source --csv > gpurun_out/tc_${TAG}_source.csv 2>/dev/null
ncu -i gpurun_out/tc_${TAG}.ncu-rep --page details --csv > gpurun_out/tc_${TAG}_details.csv 2>/dev/null
fi
