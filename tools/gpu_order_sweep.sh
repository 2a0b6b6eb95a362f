# delete ordering on/off across batch sizes (cfg2, cfg3)
D=gpurun_out/order_sweep; mkdir -p $D
for c in ${SWEEP_CFGS:-cfg2 cfg3}; do for b in ${SWEEP_B:-20 21 22 23}; do for v in off on; do
  if [ $v = off ]; then export DG_ORDER_MIN_OPS=0; else export DG_ORDER_MIN_OPS=1; fi
  timeout 600 python bench.py --config $c --batch-log2 $b --steps 10 --warmup 3 --no-e2e --no-cpu-baseline --no-vdel --no-sorted-build > $D/${c}_b${b}_$v.json 2>$D/${c}_b${b}_$v.err
  python -c "
import json;d=json.loads(open('$D/${c}_b${b}_$v.json').read().strip().splitlines()[-1])
print('$c b$b $v', round(d['value']), 'delete ms', round(d['ops']['delete']['ms_per_batch'],4))" || tail -2 $D/${c}_b${b}_$v.err
done; done; done
unset DG_ORDER_MIN_OPS
