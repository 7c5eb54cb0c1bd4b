"""Pins P1/P2 for the oracle's counter-based RNG (§IV-F).

P1: Threefry-2x64-20 against the published zero vector, and against an independent
round-parameterised, word-size-parameterised Threefry written here and validated on
four further published vectors (2x64-13, three 2x32-20) from tests/golden/threefry_kat.txt.
P2: the u01 lattice map (reading R13).
"""
from pathlib import Path

import numpy as np
import pytest

GOLD = Path(__file__).parent / "golden" / "threefry_kat.txt"


def _kats():
    out = []
    for line in GOLD.read_text().splitlines():
        if not line.strip() or line.startswith("#"):
            continue
        f = line.split()
        out.append((f[0], int(f[1]), [int(v, 16) for v in f[2:6]], [int(v, 16) for v in f[6:8]]))
    return out


def _threefry_template(bits, rounds, ctr, key):
    """Threefry-2xW (Salmon et al. SC'11): W-bit words, given round count."""
    mask = (1 << bits) - 1
    if bits == 64:
        R, C = [16, 42, 12, 31, 16, 32, 24, 21], 0x1BD11BDAA9FC1A22
    else:
        R, C = [13, 15, 26, 6, 17, 29, 16, 24], 0x1BD11BDA
    ks = [key[0], key[1], C ^ key[0] ^ key[1]]
    x0 = (ctr[0] + ks[0]) & mask
    x1 = (ctr[1] + ks[1]) & mask
    for r in range(rounds):
        x0 = (x0 + x1) & mask
        rr = R[r % 8]
        x1 = ((x1 << rr) | (x1 >> (bits - rr))) & mask
        x1 ^= x0
        if r % 4 == 3:
            s = (r + 1) // 4
            x0 = (x0 + ks[s % 3]) & mask
            x1 = (x1 + ks[(s + 1) % 3] + s) & mask
    return x0, x1


@pytest.mark.parametrize("kat", _kats(), ids=lambda k: f"{k[0]}-{k[1]}-{k[2][0]:x}")
def test_template_reproduces_published_vectors(kat):
    name, rounds, inp, out = kat
    bits = 64 if name == "threefry2x64" else 32
    assert _threefry_template(bits, rounds, inp[:2], inp[2:]) == tuple(out)


def test_oracle_threefry_zero_kat(orc):
    assert orc.threefry2x64_20(0, 0, 0, 0) == (0xC2B6E3A8C2C69865, 0x6F81ED42F350084D)


def test_oracle_threefry_matches_validated_template(orc):
    rng = np.random.default_rng(123)
    for _ in range(300):
        c0, c1, k0, k1 = (int(v) for v in rng.integers(0, 2**64, 4, dtype=np.uint64))
        assert orc.threefry2x64_20(c0, c1, k0, k1) == _threefry_template(64, 20, (c0, c1), (k0, k1))


def test_u01_lattice(orc):
    assert orc.u01(0) == 2.0**-53
    assert orc.u01(2**64 - 1) == 1.0 - 2.0**-53
    rng = np.random.default_rng(7)
    for x in rng.integers(0, 2**64, 2000, dtype=np.uint64):
        u = orc.u01(int(x))
        assert 0.0 < u < 1.0
        m = u * 2.0**53
        assert m == int(m) and int(m) % 2 == 1          # odd multiple of 2^-53
        assert int(m) == ((int(x) >> 11) | 1)
