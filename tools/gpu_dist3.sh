mkdir -p gpurun_out/r2
for t in 2,7 2,5 1,7 1,3 3,7 3,5; do
  for P in 1 8; do
    r=$((P/2))
    if [ $P = 1 ]; then env=""; else env="HEXS_DIST_EMULATE_RANK=$r/$P"; fi
    env $env timeout 600 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu --tile $t > gpurun_out/r2/tile_${t}_P$P.json 2>/dev/null
    python -c "
import json
d=json.loads(open('gpurun_out/r2/tile_${t}_P$P.json').read().strip().splitlines()[-1])
print('$t', $P, round(d['ms_per_step'],1), round(d['value'],1))"
  done
done
