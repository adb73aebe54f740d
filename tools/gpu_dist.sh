set -x
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -p no:cacheprovider --timeout 300 -k "dist" > gpurun_out/dist_pytest.txt 2>&1; echo "rc=$?" >> gpurun_out/dist_pytest.txt
tail -5 gpurun_out/dist_pytest.txt
timeout 900 python bench.py --config heat3d1024 --steps 3 --warmup 3 --no-cpu > gpurun_out/bench_heat3d1024_n1.json 2> gpurun_out/bench_heat3d1024_n1.err
cat gpurun_out/bench_heat3d1024_n1.json; tail -3 gpurun_out/bench_heat3d1024_n1.err
