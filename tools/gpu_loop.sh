mkdir -p gpurun_out/loop
timeout 600 python -m pytest tests/test_gpu_parity.py -q -m gpu -k "loopback or dist_plan" -p no:cacheprovider > gpurun_out/loop/pytest.txt 2>&1; echo "rc=$?" >> gpurun_out/loop/pytest.txt
tail -6 gpurun_out/loop/pytest.txt
