# home layout A/B on cfg2: pre-home library (variants_prehome.so) vs current, ncu of the probe kernels
D=gpurun_out/homeab; mkdir -p $D
for v in prehome cur; do
  if [ $v = prehome ]; then export DG_LIB_PATH=paper_conf_ipps_awadapo20_b200/variants_prehome.so; else unset DG_LIB_PATH; fi
  timeout 600 python bench.py --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-sorted-build --no-vdel > $D/bench_$v.json 2>$D/bench_$v.err
  python -c "
import json;d=json.loads(open('$D/bench_$v.json').read().strip().splitlines()[-1])
print('$v', round(d['value']), {k:(round(v['M_edges_s']),round(v['kernel_ms_per_batch'],3)) for k,v in d['ops'].items()})" || tail -3 $D/bench_$v.err
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_edges" --launch-skip 1 -c 3 \
     -o $D/cfg2_$v -f python tools/prof_cfg.py --config cfg2 --no-sorted > $D/ncu_$v.log 2>&1; echo ncu $v rc=$?
  python tools/ncu_summary.py $D/cfg2_$v.ncu-rep > $D/summary_$v.txt 2>&1
done
unset DG_LIB_PATH
