# A/B of library variants on the cfg2 bench (kernel times per op)
D=gpurun_out/ab_r2; mkdir -p $D
for v in base ${VARIANTS}; do
  if [ $v = base ]; then unset DG_LIB_PATH; else export DG_LIB_PATH=paper_conf_ipps_awadapo20_b200/variants_$v.so; fi
  timeout 600 python bench.py --steps 10 --warmup 3 --no-e2e --no-cpu-baseline --no-vdel --no-sorted-build ${BENCH_ARGS} > $D/$v.json 2>$D/$v.err
  python -c "
import json;d=json.loads(open('$D/$v.json').read().strip().splitlines()[-1])
print('$v', round(d['value']), {k:(round(v['M_edges_s']),round(v['kernel_ms_per_batch'],4)) for k,v in d['ops'].items()}, 'frac', round(d['roofline']['frac'],3))" || tail -3 $D/$v.err
done
unset DG_LIB_PATH
