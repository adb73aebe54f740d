CUDA_MODULE_LOADING=EAGER timeout 90 python tools/loop_debug.py star2d5 300,512 29 2 -1 2>&1 | grep -v "^[0-9]* \[False" | tail -8
