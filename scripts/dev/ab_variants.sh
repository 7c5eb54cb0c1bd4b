# usage: bash scripts/dev/ab_variants.sh TAG "v0 v1 ..." "csp:history stream:event ..." [reps] -- GPU parity
# tests (without the full-scale file) and bench lines of each library variant (NT_LIB_VARIANT),
# interleaved per config
TAG=$1; VARS=$2; CFGS=${3:-csp:history stream:history split:history}; REPS=${4:-2}
OUT=gpurun_out/$TAG; mkdir -p $OUT
for v in $VARS; do
  NT_LIB_VARIANT=$v timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider --ignore=tests/test_gpu_fullscale.py > $OUT/pytest_$v.log 2>&1
  echo "$v pytest: $(tail -1 $OUT/pytest_$v.log)"
done
for rep in $(seq 1 $REPS); do
 for cm in $CFGS; do
  c=${cm%%:*}; m=${cm##*:}; [ "$m" = "$c" ] && m=history
  for v in $VARS; do
    NT_LIB_VARIANT=$v timeout 300 python bench.py --config $c --mode $m --no-cpu-baseline --no-e2e --no-extras --steps 5 --json-out $OUT/b_${c}_${m}_${v}_$rep.json > $OUT/b_${c}_${m}_${v}_$rep.log 2>&1
    python -c "import json; d=json.load(open('$OUT/b_${c}_${m}_${v}_$rep.json')); print('$rep $c $m $v', '%.2f ms' % d['roofline']['kernel_ms'], 'frac %.3f' % d['roofline']['frac'], d['clocks']['sm_mhz'])" 2>&1 | tail -1
  done
 done
done
