#!/bin/bash
# ncu evidence for the dominant kernel (run under gpurun, one GPU).
#   1. launch list of the bench command (cold-cache, serialised: compare SHARES)
#   2. one --set full capture of k_corr (the top kernel) from the same command
# Outputs land in gpurun_out/ (scratch); summaries are copied into profiles/ by hand.
set -u
mkdir -p gpurun_out
TAG=${1:-r01}
CMD="python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv \
    --log-file gpurun_out/launches_${TAG}.csv $CMD > gpurun_out/launches_${TAG}.log 2>&1
echo "launch list rc=$?"
timeout 1500 ncu --set full --clock-control none --import-source on -k regex:k_corr -s 1 -c 1 \
    -o gpurun_out/corr_${TAG} -f $CMD > gpurun_out/corr_${TAG}.log 2>&1
echo "full capture rc=$?"
ncu -i gpurun_out/corr_${TAG}.ncu-rep --page raw --csv > gpurun_out/corr_${TAG}_raw.csv 2>/dev/null
ncu -i gpurun_out/corr_${TAG}.ncu-rep --page details --csv > gpurun_out/corr_${TAG}_details.csv 2>/dev/null
ncu -i gpurun_out/corr_${TAG}.ncu-rep --page source --csv > gpurun_out/corr_${TAG}_source.csv 2>/dev/null
echo done
