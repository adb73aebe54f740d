# quick GPU check of the streaming 3D kernel: parity, then a bench line
set -x
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -p no:cacheprovider -k "stream3d or test_3d" > gpurun_out/s3_pytest.txt 2>&1; echo "rc=$?" >> gpurun_out/s3_pytest.txt
tail -15 gpurun_out/s3_pytest.txt
timeout 600 python bench.py --config heat3d --steps 5 --warmup 3 --no-cpu > gpurun_out/s3_bench.json 2> gpurun_out/s3_bench.err
cat gpurun_out/s3_bench.json; tail -5 gpurun_out/s3_bench.err
