# usage: bash scripts/dev/ab_opts.sh TAG "csp split" "label:--flag v ..." ... -- runtime-option sweep (default library)
TAG=$1; CFGS=$2; shift 2
OUT=gpurun_out/$TAG; mkdir -p $OUT
for rep in 1 2; do for c in $CFGS; do for spec in "$@"; do
  name=${spec%%:*}; flags=${spec#*:}
  timeout 300 python bench.py --config $c $flags --no-cpu-baseline --no-e2e --steps 5 --json-out $OUT/o_${c}_${name}_$rep.json > $OUT/o_${c}_${name}_$rep.log 2>&1
  python -c "import json; d=json.load(open('$OUT/o_${c}_${name}_$rep.json')); print('$rep $c $name', '%.2f ms' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
done; done; done
