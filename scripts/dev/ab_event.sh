# usage: bash scripts/dev/ab_event.sh TAG "v1 v2" "csp stream" -- event-mode parity tests + bench per variant
TAG=$1; VARS=$2; CFGS=${3:-csp stream split scatter}
OUT=gpurun_out/$TAG; mkdir -p $OUT
for v in $VARS; do
  NT_LIB_VARIANT=$v timeout 600 python -m pytest tests -m gpu -x -q -p no:cacheprovider -k "event or Event" > $OUT/pytest_$v.log 2>&1
  echo "$v pytest: $(tail -1 $OUT/pytest_$v.log)"
done
for rep in 1 2; do for c in $CFGS; do for v in $VARS; do
  NT_LIB_VARIANT=$v timeout 300 python bench.py --config $c --mode event --no-cpu-baseline --no-e2e --steps 3 --json-out $OUT/e_${c}_${v}_$rep.json > $OUT/e_${c}_${v}_$rep.log 2>&1
  python -c "import json; d=json.load(open('$OUT/e_${c}_${v}_$rep.json')); print('$rep $c $v', '%.2f ms' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
done; done; done
