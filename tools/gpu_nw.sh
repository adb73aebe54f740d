mkdir -p gpurun_out/nw
python tools/nw_sweep.py star2d5 3 7 512 1024 1536 > gpurun_out/nw/sweep.jsonl 2>&1
python tools/nw_sweep.py star2d5 2 7 512 1024 >> gpurun_out/nw/sweep.jsonl 2>&1
python tools/nw_sweep.py box2d9 2 7 512 1024 >> gpurun_out/nw/sweep.jsonl 2>&1
python tools/nw_sweep.py box2d9 3 7 512 1024 >> gpurun_out/nw/sweep.jsonl 2>&1
cat gpurun_out/nw/sweep.jsonl
