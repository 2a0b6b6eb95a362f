# round 2 final: full GPU suite + smoke, bench lines for every config, reference arm, batch sweep
D=gpurun_out/r2final; mkdir -p $D
(nvidia-smi; nproc; free -g) > $D/host.txt 2>&1
timeout 600 python -c "import __graft_entry__ as g; g.smoke()" > $D/smoke.log 2>&1; echo smoke rc=$?; tail -1 $D/smoke.log
timeout 3000 python -m pytest tests -m gpu -q --durations=15 > $D/pytest_gpu.log 2>&1; echo pytest rc=$?; tail -22 $D/pytest_gpu.log
timeout 900 python bench.py > $D/bench_cfg2.json 2> $D/bench_cfg2.err; echo bench cfg2 rc=$?; tail -c 400 $D/bench_cfg2.json
timeout 900 python bench.py --impl reference > $D/bench_reference.json 2> $D/bench_reference.err; echo ref rc=$?; tail -c 300 $D/bench_reference.json
for c in cfg3 cfg4 cfg5; do
timeout 1500 python bench.py --config $c > $D/bench_$c.json 2> $D/bench_$c.err; echo bench $c rc=$?; tail -c 300 $D/bench_$c.json; echo
done
for b in 16 20 22; do
timeout 600 python bench.py --batch-log2 $b --steps 20 --warmup 5 --no-cpu-baseline --no-sorted-build > $D/bench_cfg2_b$b.json 2> $D/bench_cfg2_b$b.err; echo b$b rc=$?
done
