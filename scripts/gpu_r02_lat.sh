# lone-history facet latency: stream / csp with few particles (the GPU far from full)
OUT=gpurun_out/r02_lat; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
for c in stream csp; do
  for n in 148 1000 10000 100000 1000000; do
    python bench.py --config $c --particles $n --steps 3 --warmup 3 --no-cpu-baseline --no-e2e --no-extras \
      --json-out $OUT/b_${c}_n$n.json > /dev/null 2>&1
    python -c "
import json; d=json.load(open('$OUT/b_${c}_n$n.json'))
f=d['event_mix']['facets']; print('$c n=$n kernel_ms %.3f facets/particle %.0f ns_per_facet_per_particle %.1f' % (d['roofline']['kernel_ms'], f/$n, d['roofline']['kernel_ms']*1e6/(f/$n)))" 2>&1 | tail -1
  done
done
