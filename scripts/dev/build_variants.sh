# usage: bash scripts/dev/build_variants.sh "name:-DFLAG=1 -DOTHER=0" ...
# Builds nt_kernels.cu and nt_event.cu with the given -D flags, links them with the other
# objects of the last full build (build/*.o), and writes lib/variants/libneutral_b200_<name>.so for A/B timing
# with NT_LIB_VARIANT=<name>.
set -e
ROOT=$(cd "$(dirname "$0")/../.." && pwd)
PKG=$ROOT/paper_conf_cluster_martineaum17_b200
NCCL=$(python -c "import nvidia.nccl as n, os; print(list(n.__path__)[0])")
mkdir -p $PKG/lib/variants $ROOT/build/variants
# the variants link against the other objects of a full build (build/ is not shipped to the
# GPU box: rebuild it there when missing)
ls $ROOT/build/nt_api.o > /dev/null 2>&1 || (cd $ROOT && python -m paper_conf_cluster_martineaum17_b200.build --force > /dev/null)
for spec in "$@"; do
  name=${spec%%:*}; flags=${spec#*:}
  for src in nt_kernels nt_event; do
    nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -fmad=false -std=c++17 -Xcompiler -fPIC \
         --expt-relaxed-constexpr -Xptxas -v -I$NCCL/include -I$ROOT/include $flags \
         -c $PKG/csrc/$src.cu -o $ROOT/build/variants/${src}_$name.o 2> $ROOT/build/variants/ptxas_${src}_$name.log &
  done
  wait
  cp $ROOT/build/variants/ptxas_nt_kernels_$name.log $ROOT/build/variants/ptxas_$name.log
  objs=$(ls $ROOT/build/*.o | grep -v "nt_kernels.o\|nt_event.o")
  nvcc -gencode arch=compute_100a,code=sm_100a -shared -o $PKG/lib/variants/libneutral_b200_$name.so \
       $objs $ROOT/build/variants/nt_kernels_$name.o $ROOT/build/variants/nt_event_$name.o \
       -L$NCCL/lib -l:libnccl.so.2 -Xlinker -rpath,$NCCL/lib
  echo "$name: $(grep -A2 'history_kernelILb0ELi2ELb1ELb1ELi6ELi0ELb0ELb0ELb0ELb0E' $ROOT/build/variants/ptxas_$name.log | sed -n 3p)"
done
