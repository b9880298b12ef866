#!/bin/bash
# tuning sweep: bench each prebuilt library variant (paper_conf_ipps_sukhwanih10_b200/build/exp/libdock_TAG.so)
set -u
mkdir -p gpurun_out
PK=paper_conf_ipps_sukhwanih10_b200
G='"value": [0-9.]*\|"launch_ms": [0-9.]*\|fallback_rotations": [0-9]*'
for f in $PK/build/exp/libdock_*.so; do
  tag=$(basename $f .so); cp $f $PK/libdock.so; touch $PK/libdock.so
  for E in ${EPIS:-0}; do
    echo -n "$tag epi=$E: "; timeout 300 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-alt --engine tc --tc-variant 1 --tc-epi $E ${EXTRA:-} > gpurun_out/sweep_${tag}_$E.log 2>&1; grep -o "$G" gpurun_out/sweep_${tag}_$E.log | tr '\n' ' '; echo
  done
done
