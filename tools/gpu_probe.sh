# scratch GPU session: bulk-build probe + ncu full capture of the cfg2 step kernels
set -x
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1
timeout 300 python tools/bulk_probe.py > gpurun_out/bulk_probe.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:k_edges --launch-skip 4 --launch-count 3 \
   -o gpurun_out/k_edges_cfg2 -f python bench.py --steps 1 --warmup 0 --no-e2e --no-vdel --no-cpu-baseline > gpurun_out/ncu.log 2>&1
tail -5 gpurun_out/ncu.log
