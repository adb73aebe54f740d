mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -k "3d" > gpurun_out/pytest_3d.log 2>&1; echo "rc=$?" >> gpurun_out/pytest_3d.log
timeout 200 python bench.py --config heat3d --no-cpu > gpurun_out/bench_heat3d.json 2> gpurun_out/bench_heat3d.err
for t in "1,7" "3,7" "2,5"; do timeout 200 python bench.py --config heat3d --no-cpu --tile $t >> gpurun_out/bench_3d_sweep.json 2>> gpurun_out/bench_heat3d.err; done
timeout 300 ncu --set full --clock-control none --import-source on -k regex:fast3d_kernel -s 10 -c 1 -o gpurun_out/fast3d_v6 python tools/run_once.py heat3d 1 > gpurun_out/ncu_fast3d.log 2>&1
