#!/bin/bash
# Build a kernel variant of libabft.so into variants/libabft_<name>.so
# with extra nvcc flags (e.g. -DABFT_LAST_ARRIVER=0), for tools/spmv_time.py.
set -e
NAME=$1; shift
ROOT=$(cd "$(dirname "$0")/.." && pwd)
NCCL=$(cd $ROOT && python -c "import paper_conf_cluster_pawelczakmpm17_b200.build as b; print(b._nccl_dir())")
D=/tmp/var_$NAME; mkdir -p $D $ROOT/variants
cd ${SRC:-$ROOT/paper_conf_cluster_pawelczakmpm17_b200/csrc}   # SRC=<dir>: build another csrc tree (e.g. a git-archive of HEAD)
for f in kernels capi spmv_es_none spmv_es_secded spmv_es_sed spmv_es_crc; do
  nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -std=c++17 --expt-relaxed-constexpr -Xcompiler -fPIC \
    -I $NCCL/include "$@" -c $f.cu -o $D/$f.o 2> $D/$f.log &
done
wait
grep -l "error" $D/*.log && { grep -h error $D/*.log | head; exit 1; }
nvcc -gencode arch=compute_100a,code=sm_100a -shared -o $ROOT/variants/libabft_$NAME.so $D/*.o \
  -L $NCCL/lib -l:libnccl.so.2 -Xlinker -rpath=$NCCL/lib
echo built variants/libabft_$NAME.so
