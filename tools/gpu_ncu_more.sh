# ncu --set full captures of the dominant kernels of cfg3 (delete probe), cfg4 (purge
# sweep) and cfg5 (TC wedges).  Outputs in gpurun_out/$1/.
D=gpurun_out/${1:-rnext}; mkdir -p $D
python -c "import __graft_entry__ as g; g.build()" > $D/build.log 2>&1 || exit 1
timeout 1500 ncu --set full --clock-control none --import-source on -k regex:k_edges --launch-skip 5 --launch-count 3 \
   -o $D/k_edges_cfg3 -f python bench.py --config cfg3 --steps 1 --warmup 0 --no-e2e --no-vdel --no-cpu-baseline --no-sorted-build > $D/ncu_cfg3.log 2>&1
timeout 1500 ncu --set full --clock-control none --import-source on -k regex:k_vdel --launch-skip 0 --launch-count 6 \
   -o $D/k_vdel_cfg4 -f python bench.py --config cfg4 --steps 1 --warmup 0 --no-cpu-baseline --no-e2e > $D/ncu_cfg4.log 2>&1
timeout 2400 ncu --set full --clock-control none --import-source on -k regex:k_tc_wedges --launch-skip 0 --launch-count 1 \
   -o $D/k_tc_cfg5 -f python bench.py --config cfg5 --steps 1 --warmup 0 --no-cpu-baseline --no-e2e > $D/ncu_cfg5.log 2>&1
for r in $D/*.ncu-rep; do python tools/ncu_summary.py $r > ${r%.ncu-rep}.txt; done
ls -la $D
