"""B200-native neutral particle-history tracker (Martineau & McIntosh-Smith, CLUSTER 2017).

The product is the C-ABI library ``lib/libneutral_b200.so`` (header ``include/neutral_b200.h``)
built from ``csrc/`` for sm_100a; ``binding`` is its thin ctypes binding.  ``workloads``
holds the seeded synthetic input generators.
"""
