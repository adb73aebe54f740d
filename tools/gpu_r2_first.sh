set -x
nvidia-smi --query-gpu=name,memory.total --format=csv
free -g | head -2; nproc
timeout 2400 python -m pytest tests -m gpu -x -q -p no:cacheprovider --durations=15 > gpurun_out/r2_pytest_gpu.txt 2>&1; echo "pytest rc=$?" >> gpurun_out/r2_pytest_gpu.txt
tail -30 gpurun_out/r2_pytest_gpu.txt
timeout 600 python bench.py --config heat3d --steps 5 --warmup 3 --no-cpu > gpurun_out/r2_bench_heat3d_before.json 2>&1
cat gpurun_out/r2_bench_heat3d_before.json
