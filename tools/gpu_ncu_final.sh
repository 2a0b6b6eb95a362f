D=gpurun_out/ncufinal; mkdir -p $D
python -c "import __graft_entry__ as g; g.build()" > $D/build.log 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file $D/launches_bench_cfg2.csv \
   python bench.py --steps 3 --warmup 3 > $D/ncu_launches_bench.log 2>&1; echo launches rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_edges --launch-skip 4 --launch-count 3 \
   -o $D/k_edges_cfg2 -f python bench.py --steps 1 --warmup 0 --no-e2e --no-vdel --no-cpu-baseline --no-sorted-build > $D/ncu_full.log 2>&1; echo full rc=$?
ls -la $D
