mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -k "fdtd" > gpurun_out/pytest_fdtd.log 2>&1; echo "rc=$?" >> gpurun_out/pytest_fdtd.log
rm -f gpurun_out/bench_fdtd_sweep.json
for t in "5,10" "8,7" "8,5" "11,5" "11,8" "14,5"; do timeout 200 python bench.py --config fdtd2d --no-cpu --tile $t >> gpurun_out/bench_fdtd_sweep.json 2>> gpurun_out/bench_fdtd2d.err; done
