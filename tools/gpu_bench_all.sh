# Round evidence: GPU test suite, bench lines for every config (+ adaptive layout), ncu
# launch list of the default bench command, ncu full capture of the cfg2 probe kernels
# and of the cfg4 insert.  Outputs in gpurun_out/$1/.
set -x
D=gpurun_out/${1:-rnext}; mkdir -p $D
python -c "import __graft_entry__ as g; g.build(); g.smoke()" > $D/build_smoke.log 2>&1 || exit 1
timeout 1500 python -m pytest tests -m gpu -q > $D/pytest_gpu.log 2>&1; tail -3 $D/pytest_gpu.log
timeout 900 python bench.py > $D/bench_cfg2.json 2> $D/bench_cfg2.err
for c in cfg3 cfg4 cfg5; do timeout 900 python bench.py --config $c > $D/bench_$c.json 2> $D/bench_$c.err; done
for c in cfg2 cfg3 cfg4; do timeout 900 python bench.py --config $c --bucket-bytes 0 --no-e2e --no-cpu-baseline > $D/bench_${c}_adaptive.json 2> $D/bench_${c}_adaptive.err; done
for b in 16 20 22; do timeout 600 python bench.py --batch-log2 $b --no-e2e --no-cpu-baseline --no-vdel > $D/bench_cfg2_b$b.json 2> $D/bench_cfg2_b$b.err; done
timeout 900 python bench.py --impl reference --steps 3 --warmup 3 > $D/bench_cfg2_reference_arm.json 2> $D/ref.err
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/gc tools/gather_ceiling.cu && /tmp/gc > $D/gather_ceiling.json
timeout 1200 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $D/launches_bench_cfg2.csv \
   python bench.py --steps 3 --warmup 3 > $D/ncu_launches_bench.log 2>&1
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:k_edges --launch-skip 4 --launch-count 3 \
   -o $D/k_edges_cfg2 -f python bench.py --steps 1 --warmup 0 --no-e2e --no-vdel --no-cpu-baseline --no-sorted-build > $D/ncu_full.log 2>&1
timeout 1200 ncu --set full --clock-control none --import-source on -k regex:k_edges --launch-skip 1 --launch-count 1 \
   -o $D/k_edges_cfg4_insert -f python bench.py --config cfg4 --steps 1 --warmup 3 --no-cpu-baseline --no-e2e > $D/ncu_full_cfg4.log 2>&1
for f in $D/*.err; do echo "== $f"; tail -n 2 $f; done
