#!/bin/bash
# full bench line + ncu launch lists and full captures (prod: both engines; large slice: tcgen05 variant 2)
set -u
mkdir -p gpurun_out
TAG=${1:-r01}
python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > gpurun_out/build_${TAG}.log 2>&1
echo "== bench"; timeout 900 python bench.py > gpurun_out/bench_${TAG}.log 2>&1; echo "rc=$?"; tail -c 600 gpurun_out/bench_${TAG}.log
echo "== bench c64"; timeout 600 python bench.py --config c64 --no-cpu-baseline > gpurun_out/bench_${TAG}_c64.log 2>&1; echo "rc=$?"
echo "== bench large: one rank's shard of the 8-GPU config (70000 / 8 = 8750 rotations)"; timeout 900 python bench.py --config large --rotations 8750 --steps 2 --warmup 1 --no-cpu-baseline --no-alt --no-e2e > gpurun_out/bench_${TAG}_large.log 2>&1; echo "rc=$?"
bash scripts/profile.sh ${TAG} tc
bash scripts/profile.sh ${TAG} ffma
bash scripts/profile.sh ${TAG}_large tc --config large --rotations 512
