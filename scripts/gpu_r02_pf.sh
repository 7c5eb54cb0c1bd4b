# A/B: L1 prefetch of the XS row at the new energy (pf) vs the same sources without it (base)
bash scripts/dev/ab_variants.sh r02_pf "base pf" "scatter:history scatter:event csp:history split:history csp:event" 2
