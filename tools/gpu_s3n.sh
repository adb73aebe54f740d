timeout 600 ncu --set full --clock-control none --import-source on -k regex:stream3d -s 8 -c 1 -o gpurun_out/s3_full -f python tools/s3_sweep.py star3d7 512 16 > gpurun_out/s3_ncu.log 2>&1
tail -2 gpurun_out/s3_ncu.log
