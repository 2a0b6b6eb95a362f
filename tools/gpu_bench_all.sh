# Round evidence: bench lines for every config, ncu launch list of the default bench
# command, ncu full capture of the cfg2 probe kernels.  Outputs in gpurun_out/$1/.
set -x
D=gpurun_out/${1:-rnext}; mkdir -p $D
python -c "import __graft_entry__ as g; g.build()" > $D/build.log 2>&1 || exit 1
timeout 900 python bench.py > $D/bench_cfg2.json 2> $D/bench_cfg2.err
for c in cfg3 cfg4 cfg5; do timeout 900 python bench.py --config $c > $D/bench_$c.json 2> $D/bench_$c.err; done
for b in 16 20 22; do timeout 600 python bench.py --batch-log2 $b --no-e2e --no-cpu-baseline --no-vdel > $D/bench_cfg2_b$b.json 2> $D/bench_cfg2_b$b.err; done
timeout 900 python bench.py --impl reference --steps 3 --warmup 3 > $D/bench_cfg2_reference_arm.json 2> $D/ref.err
timeout 1200 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $D/launches_bench_cfg2.csv \
   python bench.py --steps 3 --warmup 3 > $D/ncu_launches_bench.log 2>&1
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:k_edges --launch-skip 4 --launch-count 3 \
   -o $D/k_edges_cfg2 -f python bench.py --steps 1 --warmup 0 --no-e2e --no-vdel --no-cpu-baseline > $D/ncu_full.log 2>&1
tail -2 $D/*.err
