set -x
mkdir -p gpurun_out
nvidia-smi > gpurun_out/smi.txt 2>&1
timeout 300 python -m pytest tests/test_gpu_parity.py -x -q -m gpu -k "voxelize or delta or shift or score_grid" > gpurun_out/t1.log 2>&1
echo "t1 rc=$?"
timeout 900 python -m pytest tests/test_gpu_parity.py -q -m gpu -k "not prod" > gpurun_out/t2.log 2>&1
echo "t2 rc=$?"
timeout 300 python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/smoke.log 2>&1
echo "smoke rc=$?"
timeout 600 python bench.py --steps 3 --warmup 2 --cpu-seconds 5 > gpurun_out/bench.log 2>&1
echo "bench rc=$?"
tail -3 gpurun_out/t1.log gpurun_out/t2.log gpurun_out/smoke.log gpurun_out/bench.log
