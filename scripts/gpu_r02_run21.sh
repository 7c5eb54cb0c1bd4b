OUT=gpurun_out/r02_t21; mkdir -p $OUT
python -c "import __graft_entry__ as g; g.build()"
timeout 1800 python -m pytest tests -m gpu -q -p no:cacheprovider -x -k "event or mode" --ignore=tests/test_gpu_fullscale.py > $OUT/pytest.log 2>&1; echo "PYTEST $(tail -1 $OUT/pytest.log)"; grep -E "^FAILED" $OUT/pytest.log | head
bash scripts/dev/ab_variants.sh r02_ab18_ev_pairs "evnew evold" "csp:event stream:event split:event scatter:event" 2 | grep -v "pytest: 2"
