#!/bin/bash
# One ncu --set full capture of one kernel launch from a short bench command (run under gpurun, 1 GPU).
# usage: ncu_kernel.sh TAG KERNEL_REGEX [bench args...]
set -u
mkdir -p gpurun_out
TAG=$1; KRE=$2; shift 2
python -c "import __graft_entry__ as e; e.build()" > /dev/null || exit 1
CMD="python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu-baseline --no-alt $*"
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:$KRE -s ${SKIP:-1} -c 1 \
    -o /tmp/prof_${TAG} -f $CMD > gpurun_out/ncu_${TAG}.log 2>&1
echo "capture rc=$?"
ncu -i /tmp/prof_${TAG}.ncu-rep --page raw --csv > gpurun_out/ncu_${TAG}_raw.csv 2>/dev/null
ncu -i /tmp/prof_${TAG}.ncu-rep --page details --csv > gpurun_out/ncu_${TAG}_details.csv 2>/dev/null
ncu -i /tmp/prof_${TAG}.ncu-rep --page source --csv > gpurun_out/ncu_${TAG}_source.csv 2>/dev/null
gzip -f gpurun_out/ncu_${TAG}_source.csv
tail -3 gpurun_out/ncu_${TAG}.log
