#!/bin/bash
# build libdg with extra nvcc flags into paper_conf_ipps_awadapo20_b200/variants_<name>.so
#   tools/build_variant.sh NAME -DFOO=1 ...   (load with DG_LIB_PATH=...)
set -e
name=$1; shift
cd "$(dirname "$0")/.."
inc=$(python -c "import sys; sys.path.insert(0,'paper_conf_ipps_awadapo20_b200'); import build; print(build._nccl_include())")
out=build/variant_$name; mkdir -p $out
for f in paper_conf_ipps_awadapo20_b200/csrc/*.cu; do
  /usr/local/cuda/bin/nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 --expt-relaxed-constexpr \
    -Xcompiler -fPIC -Xcompiler -fvisibility=hidden -Iinclude -I$inc "$@" -c $f -o $out/$(basename $f).o &
done
wait
/usr/local/cuda/bin/nvcc -gencode arch=compute_100a,code=sm_100a -shared -o paper_conf_ipps_awadapo20_b200/variants_$name.so $out/*.o -cudart static -ldl -lpthread -lrt
echo paper_conf_ipps_awadapo20_b200/variants_$name.so
