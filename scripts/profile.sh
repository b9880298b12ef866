#!/bin/bash
# ncu evidence for the dominant kernel (run under gpurun, one GPU).
#   1. launch list of the bench command (cold-cache, serialised: compare SHARES)
#   2. one --set full capture of the correlation kernel from the same command
# The .ncu-rep stays in /tmp (gpurun copies back <= 64 MiB); its raw/details/source pages come back as CSV.
# usage: profile.sh TAG ENGINE(ffma|tc|auto) [extra bench args]
set -u
mkdir -p gpurun_out
TAG=${1:-r01}
ENGINE=${2:-auto}
shift 2 || true
KRE=k_corr; [ "$ENGINE" = "tc" ] && KRE=k_corr_tc
CMD="python bench.py --steps 2 --warmup 1 --no-e2e --no-cpu-baseline --no-alt --engine $ENGINE $*"
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv \
    --log-file gpurun_out/launches_${TAG}_${ENGINE}.csv $CMD > gpurun_out/launches_${TAG}_${ENGINE}.log 2>&1
echo "launch list rc=$?"
timeout 1500 ncu --set full --clock-control none --import-source on -k regex:$KRE -s 1 -c 1 \
    -o /tmp/corr_${TAG}_${ENGINE} -f $CMD > gpurun_out/corr_${TAG}_${ENGINE}.log 2>&1
echo "full capture rc=$?"
ncu -i /tmp/corr_${TAG}_${ENGINE}.ncu-rep --page raw --csv > gpurun_out/corr_${TAG}_${ENGINE}_raw.csv 2>/dev/null
ncu -i /tmp/corr_${TAG}_${ENGINE}.ncu-rep --page details --csv > gpurun_out/corr_${TAG}_${ENGINE}_details.csv 2>/dev/null
ncu -i /tmp/corr_${TAG}_${ENGINE}.ncu-rep --page source --csv > gpurun_out/corr_${TAG}_${ENGINE}_source.csv 2>/dev/null
gzip -f gpurun_out/corr_${TAG}_${ENGINE}_source.csv
du -sh gpurun_out
echo done
