# A/B: phase 1 at 5 CTAs/SM (90 registers), phase 2 at 6 (80) vs both at 6
bash scripts/dev/ab_variants.sh r02_p15 "base p15" "csp:history stream:history split:history scatter:history" 2
