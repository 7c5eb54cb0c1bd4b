# usage: bash scripts/dev/build_rev.sh NAME GITREV -- builds the whole library of a git revision
# into lib/variants/libneutral_b200_<NAME>.so (A/B against the working tree)
set -e
ROOT=$(cd "$(dirname "$0")/../.." && pwd)
NAME=$1; REV=$2
TMP=$(mktemp -d)
git -C $ROOT archive $REV paper_conf_cluster_martineaum17_b200/csrc include | tar -x -C $TMP
NCCL=$(python -c "import nvidia.nccl as n; print(list(n.__path__)[0])")
objs=""
for f in $TMP/paper_conf_cluster_martineaum17_b200/csrc/*.cu; do
  o=$TMP/$(basename $f .cu).o
  nvcc -gencode arch=compute_100a,code=sm_100a -O3 -lineinfo -fmad=false -std=c++17 -Xcompiler -fPIC \
       --expt-relaxed-constexpr -I$NCCL/include -I$TMP/include -c $f -o $o &
  objs="$objs $o"
done
wait
mkdir -p $ROOT/paper_conf_cluster_martineaum17_b200/lib/variants
nvcc -gencode arch=compute_100a,code=sm_100a -shared -o $ROOT/paper_conf_cluster_martineaum17_b200/lib/variants/libneutral_b200_$NAME.so \
     $objs -L$NCCL/lib -l:libnccl.so.2 -Xlinker -rpath,$NCCL/lib
rm -rf $TMP
echo "built $NAME from $REV"
