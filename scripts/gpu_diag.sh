# Diagnostic experiments (NT_DIAG switches parts of the history kernel off; results WRONG).
python -c "import __graft_entry__ as g; g.build()"
for dg in ${DIAGS:-0 1 2 4 3 7}; do
  for c in ${CONFIGS:-stream csp}; do
    NT_DIAG=$dg python bench.py --config $c --no-cpu-baseline --no-e2e --steps 3 $EXTRA > /tmp/d.json 2>/dev/null
    python -c "import json; d=json.load(open('/tmp/d.json')); print('diag', $dg, d['config']['workload'], '%.3e' % d['value'], '%.2f ms' % d['ms_per_step'])"
  done
done
