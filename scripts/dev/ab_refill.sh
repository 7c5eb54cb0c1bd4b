# usage: bash scripts/dev/ab_refill.sh TAG VARIANT "4 8 16" "csp split" -- refill_min sweep of one variant
TAG=$1; V=$2; RS=$3; CFGS=${4:-csp split}
OUT=gpurun_out/$TAG; mkdir -p $OUT
for c in $CFGS; do for r in $RS; do
  NT_LIB_VARIANT=$V timeout 300 python bench.py --config $c --refill-min $r --no-cpu-baseline --no-e2e --steps 5 --json-out $OUT/r_${c}_${V}_$r.json > $OUT/r_${c}_${V}_$r.log 2>&1
  python -c "import json; d=json.load(open('$OUT/r_${c}_${V}_$r.json')); print('$c $V refill $r', '%.2f ms' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
done; done
