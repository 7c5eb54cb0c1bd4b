OUT=gpurun_out/r02_t20; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
bash scripts/dev/build_variants.sh "ev_dw_lz:-DNT_EV_DOWHILE=1 -DNT_EV_LAZYREFILL=1" "ev_dw:-DNT_EV_DOWHILE=1 -DNT_EV_LAZYREFILL=0" "ev_base:-DNT_EV_DOWHILE=0 -DNT_EV_LAZYREFILL=0" > /dev/null 2>&1
bash scripts/dev/ab_variants.sh r02_ab17_ev_loop "ev_dw_lz ev_dw ev_base" "csp:event stream:event split:event scatter:event" 2 | grep -v "pytest: 2"
