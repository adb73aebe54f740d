export CUDA_MODULE_LOADING=EAGER
HEXS_DIST_FUSED=1 timeout 150 compute-sanitizer --tool memcheck --print-limit 5 python tools/loop_check.py box3d27 30,52,64 13 2 1 2>&1 | grep -v "^=========     \(Host\|Saved\|     \)" | head -40
