#!/bin/bash
# sparse engine: columns between global-bound refreshes (DOCK_SP_BOUND_EVERY; 0 = off), c64 and the large shard
python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > /dev/null 2>&1
G='"launch_ms": [0-9.]*'
for E in ${EVERY:-0 1 2 4 8 16}; do
  echo -n "every $E c64: "; DOCK_SP_BOUND_EVERY=$E python bench.py --config c64 --no-cpu-baseline --no-alt --no-e2e --steps 5 --warmup 3 2>&1 | grep -o "$G" | tr '\n' ' '
  echo -n " large: "; DOCK_SP_BOUND_EVERY=$E python bench.py --config large --rotations 8750 --steps 3 --warmup 2 --no-cpu-baseline --no-e2e --no-alt 2>&1 | grep -o "$G" | tr '\n' ' '; echo
done
