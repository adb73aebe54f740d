set -x
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -p no:cacheprovider --timeout 60 -k "stream3d" > gpurun_out/s3_pytest.txt 2>&1; echo "rc=$?" >> gpurun_out/s3_pytest.txt
tail -4 gpurun_out/s3_pytest.txt
timeout 120 python tools/s3_sweep.py star3d7 512 128 > gpurun_out/s3_sweep.json 2>&1
cat gpurun_out/s3_sweep.json
timeout 300 ncu --set full --clock-control none --import-source on -k regex:stream3d -s 8 -c 1 -o gpurun_out/s3_full -f python tools/s3_sweep.py star3d7 512 16 > gpurun_out/s3_ncu.log 2>&1
tail -2 gpurun_out/s3_ncu.log
