# phase timeline (dev variant NT_TIMELINE=1) on csp, split, scatter, stream
TAG=${1:-r02_tl}
OUT=gpurun_out/$TAG; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
bash scripts/dev/build_variants.sh "tl:-DNT_TIMELINE=1" > $OUT/build.log 2>&1
for c in csp split scatter stream; do
  NT_LIB_VARIANT=tl python scripts/dev/phase_timeline.py $c $OUT/timeline_$c.json > $OUT/timeline_$c.log 2>&1
  python -c "
import json; d=json.load(open('$OUT/timeline_$c.json'))
for p in ('phase1','phase2'):
    x=d[p]; print('$c', p, 'span %.0f us, range out at %.0f us, tail %.0f us (%.2f), busy %.2f' % (x['span_us'], x['range_exhausted_at_us'], x['tail_us'], x['tail_frac'], x['warp_busy_frac']), 'end q50/q90 %.0f/%.0f' % (x['warp_end_quantiles_us'][50], x['warp_end_quantiles_us'][90]))
" 2>&1 | tail -2
done
