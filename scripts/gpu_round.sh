#!/bin/bash
# One gpurun session: microbenchmarks, GPU parity tests, smoke, bench, (optional) ncu.
set -u
mkdir -p gpurun_out
nvidia-smi > gpurun_out/smi.txt 2>&1
python -c "from paper_conf_ipps_sukhwanih10_b200 import build; build.build_native()" > gpurun_out/build.log 2>&1



echo "== tests"; timeout 1500 python -m pytest tests -q -m gpu --timeout 600 > gpurun_out/tests_gpu.log 2>&1; echo "rc=$?"; tail -15 gpurun_out/tests_gpu.log
echo "== smoke"; timeout 300 python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/smoke.log 2>&1; echo "rc=$?"; tail -3 gpurun_out/smoke.log
echo "== bench"; timeout 900 python bench.py > gpurun_out/bench.log 2>&1; echo "rc=$?"; tail -3 gpurun_out/bench.log
if [ "${PROFILE:-0}" = "1" ]; then echo "== profile"; bash scripts/profile.sh ${TAG:-r01} ffma; bash scripts/profile.sh ${TAG:-r01} tc; fi
