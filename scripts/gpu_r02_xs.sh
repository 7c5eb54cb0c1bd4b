# XS staging A/B (round 2): direct bucket rows (xs_search 3) and the L2 persisting window
# (xs_l2_persist 1) against the bucketed search, on scatter / scatter_src050 / csp, history
# and event; GPU parity of the XS paths first.
TAG=${1:-r02_xs}
OUT=gpurun_out/$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests -m gpu -q -p no:cacheprovider -x -k "xs or smoke or inject" > $OUT/pytest.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest.log)"; grep -E "^FAILED" $OUT/pytest.log | head
for rep in 1 2; do
  for cm in scatter:history scatter:event csp:history csp:event; do
    c=${cm%%:*}; m=${cm##*:}
    for v in "0 0" "3 0" "0 1" "3 1"; do
      set -- $v
      python bench.py --config $c --mode $m --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
        --xs-search $1 --xs-l2-persist $2 --json-out $OUT/b_${c}_${m}_xs$1_l2$2_r$rep.json > /dev/null 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_${m}_xs$1_l2$2_r$rep.json'))
print('$c $m xs=$1 l2=$2 rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'], 'ms %.3f' % d['ms_per_step'])" 2>&1 | tail -1
    done
  done
done
for v in "0 0" "3 0"; do
  set -- $v
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:history -c 2 -o $OUT/prof_scatter_xs$1 \
    python bench.py --config scatter --steps 1 --warmup 0 --no-cpu-baseline --no-e2e --no-extras --xs-search $1 > $OUT/ncu_xs$1.log 2>&1
  python scripts/ncu_summary.py $OUT/prof_scatter_xs$1.ncu-rep $OUT/ncu_scatter_xs$1.md > /dev/null 2>&1
  rm -f $OUT/prof_scatter_xs$1.ncu-rep
done
ls $OUT | head -50
