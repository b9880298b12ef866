#!/bin/bash
# tcgen05 variant-1 chunk size sweep (tiles per dynamically scheduled chunk) at prod and at a 1008-unit launch
python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > /dev/null 2>&1
B="python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-alt --engine tc"
G='"value": [0-9.]*\|"launch_ms": [0-9.]*'
for C in ${CHUNKS:-4 8 16 32 64}; do
  echo -n "prod chunk $C: "; timeout 300 $B --tc-chunk $C 2>&1 | grep -o "$G" | tr '\n' ' '; echo
  echo -n "1008 units chunk $C: "; timeout 300 $B --tc-chunk $C --rotations 63 2>&1 | grep -o "$G" | tr '\n' ' '; echo
done
