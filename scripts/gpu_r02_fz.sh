# DEV A/B: fused phases with zero dedicated consumer CTAs (producers resume parked particles
# once their phase-1 range is exhausted) vs two launches vs fused 1.
TAG=${1:-r02_fz}
OUT=gpurun_out/$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
NT_FUSED_ZERO=1 timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x -k "fused" > $OUT/pytest.log 2>&1
echo "PYTEST(fused zero) $(tail -1 $OUT/pytest.log)"
for rep in 1 2; do
  for c in csp split scatter stream; do
    for v in "0 0" "1 1" "1 0"; do
      set -- $v
      if [ $2 = 1 ]; then export NT_FUSED_ZERO=1; else unset NT_FUSED_ZERO; fi
      python bench.py --config $c --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
        --fused-consumers $1 --json-out $OUT/b_${c}_f$1_z$2_r$rep.json > /dev/null 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_f$1_z$2_r$rep.json'))
print('$c fused=$1 zero=$2 rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
    done
  done
done
unset NT_FUSED_ZERO
