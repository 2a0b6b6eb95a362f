# bench lines only (after a measurement-method change): default cfg2, batch sweep, cfg3, cfg4, cfg5
D=gpurun_out/lines; mkdir -p $D
timeout 900 python bench.py > $D/bench_cfg2.json 2> $D/bench_cfg2.err; echo cfg2 rc=$?
for b in 16 20 22; do timeout 600 python bench.py --batch-log2 $b --steps 20 --warmup 5 --no-cpu-baseline --no-sorted-build > $D/bench_cfg2_b$b.json 2> $D/bench_cfg2_b$b.err; echo b$b rc=$?; done
for c in cfg3 cfg4 cfg5; do timeout 1500 python bench.py --config $c > $D/bench_$c.json 2> $D/bench_$c.err; echo $c rc=$?; done
