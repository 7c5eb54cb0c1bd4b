# init_mesh (chunked upload + hashed distinct values) and XS row cap: GPU tests touching the
# mesh / tables, the e2e breakdown per C-ABI call, the default bench line, the table sweep.
TAG=${1:-r02_mesh}
OUT=gpurun_out/$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 1500 python -m pytest tests -m gpu -q -p no:cacheprovider -x --ignore=tests/test_gpu_fullscale.py > $OUT/pytest.log 2>&1
echo "PYTEST $(tail -1 $OUT/pytest.log)"; grep -E "^FAILED|Error" $OUT/pytest.log | head -5
python scripts/dev/e2e_breakdown.py csp > $OUT/e2e_breakdown.json 2> $OUT/e2e_breakdown.err; tail -1 $OUT/e2e_breakdown.json
python bench.py --steps 5 --warmup 3 --no-cpu-baseline --no-extras --json-out $OUT/b_e2e.json > $OUT/b_e2e.log 2>&1
python -c "
import json; d=json.load(open('$OUT/b_e2e.json')); print('E2E', d['value'], d['ms_per_step'], d['e2e']['value'], d['e2e']['ms_per_step'])"
for n in 65536 1048576; do
  for x in 0 3; do
    python bench.py --config scatter --steps 5 --warmup 3 --no-cpu-baseline --no-e2e --no-extras --table-size $n \
      --xs-search $x --json-out $OUT/b_scatter_tab${n}_xs$x.json > /dev/null 2>&1
    python -c "
import json; d=json.load(open('$OUT/b_scatter_tab${n}_xs$x.json'))
print('TABLE $n xs=$x kernel_ms %.3f' % d['roofline']['kernel_ms'])" 2>&1 | tail -1
  done
done
