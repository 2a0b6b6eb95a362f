# cfg2/cfg3 evidence (bench lines, sweep, reference arm, ncu) + query-prefetch A/B. Outputs in gpurun_out/$1/.
set -x
D=gpurun_out/${1:-rnext}; mkdir -p $D
python -c "import __graft_entry__ as g; g.build()" > $D/build.log 2>&1 || exit 1
timeout 1500 python -m pytest tests -m gpu -q > $D/pytest_gpu.log 2>&1; tail -3 $D/pytest_gpu.log

timeout 900 python bench.py > $D/bench_cfg2.json 2> $D/bench_cfg2.err
timeout 900 python bench.py --config cfg3 > $D/bench_cfg3.json 2> $D/bench_cfg3.err
for c in cfg2 cfg3; do timeout 900 python bench.py --config $c --bucket-bytes 0 --no-e2e --no-cpu-baseline > $D/bench_${c}_adaptive.json 2> $D/bench_${c}_adaptive.err; done
for b in 16 20 22; do timeout 600 python bench.py --batch-log2 $b --no-e2e --no-cpu-baseline --no-vdel --no-sorted-build > $D/bench_cfg2_b$b.json 2> $D/bench_cfg2_b$b.err; done
timeout 900 python bench.py --impl reference --steps 3 --warmup 3 > $D/bench_cfg2_reference_arm.json 2> $D/ref.err
timeout 1200 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $D/launches_bench_cfg2.csv \
   python bench.py --steps 3 --warmup 3 > $D/ncu_launches_bench.log 2>&1
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:k_edges --launch-skip 4 --launch-count 3 \
   -o $D/k_edges_cfg2 -f python bench.py --steps 1 --warmup 0 --no-e2e --no-vdel --no-cpu-baseline --no-sorted-build > $D/ncu_full.log 2>&1
for f in $D/*.err; do echo "== $f"; tail -n 2 $f; done
