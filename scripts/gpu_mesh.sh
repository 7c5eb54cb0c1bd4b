python -c "import __graft_entry__ as g; g.build()"
for m in 1000 2000 2828 4000; do
  for dg in 0 1; do
    NT_DIAG=$dg python bench.py --config stream --mesh $m --no-cpu-baseline --no-e2e --steps 3 > /tmp/d.json 2>/dev/null
    python -c "import json; d=json.load(open('/tmp/d.json')); print('mesh', $m, 'diag', $dg, '%.3e ev/s' % d['value'], '%.2f ms' % d['ms_per_step'], d['event_mix']['facets'])"
  done
done
