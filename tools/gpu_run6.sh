python -c "import __graft_entry__ as g; g.build()" > gpurun_out/build.log 2>&1 || exit 1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_export_fill|k_tc_" --launch-count 4 \
   -o gpurun_out/tc_set64 -f python tools/tc_probe.py 22 64 set 1 > gpurun_out/ncu_tc.log 2>&1
tail -3 gpurun_out/ncu_tc.log
