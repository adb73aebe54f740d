# round-2 evidence: per-config ncu launch lists (DRAM, L2, time, CTAs per launch) of one run
mkdir -p gpurun_out/ev
M=dram__bytes_read.sum,dram__bytes_write.sum,lts__t_bytes.sum,gpu__time_duration.sum,launch__grid_size
for c in heat2d5 heat2d9 gradient2d jacobi2d fdtd2d heat3d gradient3d heat3d27 heat3d1024; do
  timeout 1200 ncu --metrics $M --clock-control none -k regex:"fast2d|fdtd|fast3d|stream3d|generic|naive" --csv --log-file gpurun_out/ev/launches_$c.csv python tools/run_once.py $c 1 > gpurun_out/ev/run_$c.log 2>&1
  python tools/ncu_traffic.py $c gpurun_out/ev/launches_$c.csv > /dev/null 2> gpurun_out/ev/tr_$c.err && echo "$c ok" || echo "$c FAIL"
done
cp profiles/round2/traffic_*.json gpurun_out/ev/ 2>/dev/null
