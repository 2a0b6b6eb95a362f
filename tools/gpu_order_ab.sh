# locality-ordered delete/query: parity (forced on small cases, full-size cfg2/cfg3) and bench A/B
D=gpurun_out/order; mkdir -p $D
timeout 1500 python -m pytest tests/test_gpu_order.py tests/test_gpu_fullsize.py -m gpu -q -x -k "order or config2 or config3" > $D/pytest.log 2>&1; echo pytest rc=$?; tail -4 $D/pytest.log
for v in off on; do
  if [ $v = off ]; then export DG_ORDER_MIN_OPS=0; else unset DG_ORDER_MIN_OPS; fi
  timeout 600 python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline --no-vdel --no-sorted-build ${BENCH_ARGS} > $D/$v.json 2>$D/$v.err
  python -c "
import json;d=json.loads(open('$D/$v.json').read().strip().splitlines()[-1])
print('$v', round(d['value']), {k:(round(v['M_edges_s']),round(v['kernel_ms_per_batch'],4), round(v['ms_per_batch'],4)) for k,v in d['ops'].items()}, 'frac', round(d['roofline']['frac'],3))" || tail -3 $D/$v.err
done
unset DG_ORDER_MIN_OPS
for c in cfg3 cfg4; do
timeout 900 python bench.py --config $c --steps 10 --warmup 3 --no-e2e --no-cpu-baseline > $D/on_$c.json 2>$D/on_$c.err
python -c "
import json;d=json.loads(open('$D/on_$c.json').read().strip().splitlines()[-1])
print('$c on', round(d['value']), d.get('ops'))" || tail -3 $D/on_$c.err
done
