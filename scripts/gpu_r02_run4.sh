bash scripts/gpu_r02_prof.sh r02_t4 "csp:event stream:event" tests
bash scripts/dev/ab_variants.sh r02_ab_xs "xsbase xshint" "scatter:history csp:history scatter:event" 2
