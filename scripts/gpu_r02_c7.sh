# runtime option sweep on the final tree: 7 CTAs/SM at 72 registers vs the default (6 x 80)
OUT=gpurun_out/r02_c7; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
for rep in 1 2; do
  for c in scatter csp split scatter_src050; do
    for v in 0 7; do
      python bench.py --config $c --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras --ctas-per-sm $v \
        --json-out $OUT/b_${c}_c${v}_r$rep.json > /dev/null 2>&1
      python -c "
import json; d=json.load(open('$OUT/b_${c}_c${v}_r$rep.json'))
print('$c ctas=$v rep=$rep', 'kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
    done
  done
done
