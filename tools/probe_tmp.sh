mkdir -p gpurun_out
for c in heat2d5:fast2d_kernel heat2d9:fast2d_kernel fdtd2d:fdtd_kernel heat3d:fast3d_kernel gradient3d:fast3d_kernel; do
  cfg=${c%%:*}; k=${c##*:}
  timeout 600 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k regex:$k --csv --log-file gpurun_out/launches_$cfg.csv python tools/run_once.py $cfg 1 > gpurun_out/ncu_launches_$cfg.log 2>&1
done
timeout 300 ncu --set full --clock-control none --import-source on -k regex:fdtd_kernel -s 20 -c 1 -o gpurun_out/fdtd_v4 python tools/run_once.py fdtd2d 1 > gpurun_out/ncu_fdtd.log 2>&1
timeout 300 python bench.py > gpurun_out/bench_default.json 2> gpurun_out/bench_default.err
timeout 300 python bench.py --config fdtd2d --no-cpu > gpurun_out/bench_fdtd2d.json 2> gpurun_out/bench_fdtd2d.err
