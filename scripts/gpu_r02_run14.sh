OUT=gpurun_out/r02_t14; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
bash scripts/dev/build_variants.sh "hbase:" > /dev/null 2>&1
bash scripts/dev/ab_variants.sh r02_ab12_hist_fsum_xsearly "hbase hfsum hxse hboth" "scatter:history csp:history split:history" 2 | grep -v pytest
bash scripts/dev/ab_variants.sh r02_ab13_ev_refill "ev_r8 ev_r8reg ev_r4reg" "csp:event stream:event split:event scatter:event" 2 | grep -v pytest
