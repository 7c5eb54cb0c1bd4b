# usage: bash scripts/gpu_variants.sh [reps]  -- A/B timing of prebuilt library variants
# build/variants/*.so (each copied over lib/libneutral_b200.so in turn; the tree's own build
# is restored at the end); CONFIGS (default "csp stream split scatter"), interleaved reps.
LIB=paper_conf_cluster_martineaum17_b200/lib/libneutral_b200.so
cp $LIB /tmp/own.so
REPS=${1:-2}
for rep in $(seq $REPS); do
  for v in build/variants/*.so; do
    cp $v $LIB
    for c in ${CONFIGS:-csp stream split scatter}; do
      python bench.py --config $c ${ARGS:-} --no-cpu-baseline --no-e2e --steps ${STEPS:-5} > /tmp/d.json 2>/dev/null
      python -c "import json; d=json.load(open('/tmp/d.json')); r=d['roofline']; print('$(basename $v .so)', d['config']['workload'], '%.3e ev/s' % d['value'], 'kernel %.2f ms' % r['kernel_ms'], 'clk', d['clocks']['sm_mhz'])" 2>&1 | tail -1
    done
  done
done
cp /tmp/own.so $LIB
