D=gpurun_out/homeab3; mkdir -p $D
for c in cfg2 cfg3; do
timeout 600 python bench.py --config $c --steps 5 --warmup 3 --no-e2e --no-cpu-baseline --no-vdel > $D/bench_$c.json 2>$D/bench_$c.err
python -c "
import json;d=json.loads(open('$D/bench_$c.json').read().strip().splitlines()[-1])
print('$c', round(d['value']), {k:(round(v['M_edges_s']),round(v['kernel_ms_per_batch'],3)) for k,v in d['ops'].items()}, {k:round(v,2) for k,v in d['bulk_build'].items() if 'kernel_ms' in k})" || tail -3 $D/bench_$c.err
done
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_edges" --launch-skip 1 -c 3 \
   -o $D/cfg2_cur -f python tools/prof_cfg.py --config cfg2 --no-sorted > $D/ncu_cur.log 2>&1; echo ncu rc=$?
python tools/ncu_summary.py $D/cfg2_cur.ncu-rep > $D/summary_cur.txt 2>&1; grep -E "k_edges|time_dur|inst_exec|dram__bytes_read" $D/summary_cur.txt
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_multirank.py -q -x > $D/parity.log 2>&1; echo parity rc=$?; tail -3 $D/parity.log
