OUT=gpurun_out/r02_t19; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 900 python -m pytest tests/test_gpu_parity.py -m gpu -q -p no:cacheprovider -k "parity_deterministic or production_atomic" > $OUT/pytest.log 2>&1; echo "PYTEST $(tail -1 $OUT/pytest.log)"
bash scripts/dev/build_variants.sh "evffs:-DNT_EV_FFS=1" "evnoffs:-DNT_EV_FFS=0" > /dev/null 2>&1
bash scripts/dev/ab_variants.sh r02_ab16_ev_ffs "evffs evnoffs" "csp:event stream:event split:event scatter:event" 2 | grep -v pytest
