for t in 2,7 1,7; do
HEXS_STREAM3D=1 timeout 600 python bench.py --config gradient3d --steps 3 --warmup 3 --no-cpu --tile $t 2>/dev/null | python -c "
import json,sys
d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('s3 gradient3d $t', round(d['value'],1), d['roofline']['kernel'], d['naive_gups'])"
done
HEXS_STREAM3D=1 timeout 600 python bench.py --config heat3d --steps 3 --warmup 3 --no-cpu 2>/dev/null | python -c "
import json,sys
d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('s3 heat3d', round(d['value'],1), d['roofline']['kernel'], d['config']['tile'])"
