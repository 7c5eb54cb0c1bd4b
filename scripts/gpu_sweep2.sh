# usage: bash scripts/gpu_sweep2.sh "ARGS1" "ARGS2" ...   per-config bench for each argument set
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests -m gpu -x -q -p no:cacheprovider 2>&1 | tail -1 | sed "s/^/PYTEST: /"
for args in "$@"; do
  for c in ${CONFIGS:-csp stream scatter split}; do
    python bench.py --config $c $args --no-cpu-baseline --no-e2e --steps 3 > /tmp/d.json 2>/dev/null
    python -c "import json; d=json.load(open('/tmp/d.json')); print('[$args]', d['config']['workload'], '%.3e ev/s' % d['value'], '%.2f ms' % d['ms_per_step'])"
  done
done
