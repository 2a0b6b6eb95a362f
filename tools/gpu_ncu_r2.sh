# round 2 profiles: launch list of the default bench, ncu --set full of the probe
# kernels (cfg2, cfg3), the sorted bulk-build kernel and the cfg5 wedge kernel
D=gpurun_out/ncu_r2; mkdir -p $D
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $D/launches_bench_cfg2.csv \
   python bench.py --steps 3 --warmup 3 --no-e2e --no-cpu-baseline > $D/launches.log 2>&1; echo launches rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_edges|k_insert_sorted|k_order|k_validate" -c 24 \
   -o $D/cfg2 -f python tools/prof_cfg.py --config cfg2 > $D/cfg2.log 2>&1; echo cfg2 rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_edges" -c 8 \
   -o $D/cfg3 -f python tools/prof_cfg.py --config cfg3 --no-sorted > $D/cfg3.log 2>&1; echo cfg3 rc=$?
timeout 900 ncu --set full --clock-control none -k regex:"k_tc_wedges" -c 1 \
   -o $D/cfg5 -f python bench.py --config cfg5 --steps 1 --warmup 0 > $D/cfg5.log 2>&1; echo cfg5 rc=$?
for f in cfg2 cfg3 cfg5; do python tools/ncu_summary.py $D/$f.ncu-rep > $D/summary_$f.txt 2>&1; done
python tools/launch_share.py $D/launches_bench_cfg2.csv > $D/launches_summary.txt 2>&1
ls -la $D
timeout 1500 python bench.py --config cfg5 > $D/bench_cfg5.json 2> $D/bench_cfg5.err; echo cfg5 rc=$?
python -c "import json; d=json.loads(open('$D/bench_cfg5.json').read().strip().splitlines()[-1]); print('cfg5', d['value'], d['tc']['insert_ms_per_step'], d['tc']['tc_ms_per_step'], d['clocks'])"
