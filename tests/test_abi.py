"""The C-ABI library loads and exports every symbol include/*.h declares (no GPU needed).

Also checks that the product package does not import the oracle (the
oracle is test infrastructure only) and that the library has no CPU fallback.
"""
import ast
import ctypes as C
import re
from pathlib import Path

import pytest

ROOT = Path(__file__).resolve().parent.parent
PKG = ROOT / "paper_conf_cluster_martineaum17_b200"


def _declared():
    names = set()
    for h in (ROOT / "include").glob("*.h"):
        txt = re.sub(r"/\*.*?\*/", "", h.read_text(), flags=re.S)
        names |= set(re.findall(r"\b(nt_[a-z_0-9]+)\s*\(", txt))
    return names


@pytest.fixture(scope="module")
def L():
    from paper_conf_cluster_martineaum17_b200 import build, binding
    build.build()
    return binding.lib()


def test_exports_every_declared_symbol(L):
    from paper_conf_cluster_martineaum17_b200 import binding
    declared = _declared()
    assert declared, "no declarations found"
    assert declared == set(binding.EXPORTS)
    for name in declared:
        assert hasattr(L, name), name


def test_identity_calls(L):
    from paper_conf_cluster_martineaum17_b200 import binding
    assert L.nt_abi_version() == 5
    assert b"sm_100a" in L.nt_build_info()
    assert b"-fmad=false" in L.nt_build_info()
    for k, v in binding.STATUS.items():
        assert L.nt_status_string(k).decode() == v
    o = binding.Options()
    assert L.nt_options_default(C.byref(o)) == 0
    assert o.nranks == 1 and o.A == 1.0 and o.e_min == 1.0 and o.w_min == 1e-3
    assert o.max_events_per_history == 10**9 and o.det_batch == 65536 and o.refill_min == 4
    assert o.defer_below == 8 and o.resume_prefetch == 0 and o.xs_search == 0


def test_struct_layouts_match_header():
    """ctypes structs mirror the header's field lists (names and order)."""
    from paper_conf_cluster_martineaum17_b200 import binding
    txt = (ROOT / "include" / "neutral_b200.h").read_text()

    def fields(struct_name):
        body = re.search(r"typedef struct \{([^{}]*)\}\s*" + struct_name + ";", txt).group(1)
        body = re.sub(r"/\*.*?\*/", "", body, flags=re.S)
        out = []
        for decl in body.split(";"):
            decl = decl.strip()
            if not decl:
                continue
            names = decl.split(None, 1)[1] if not decl.startswith("const") else decl.split(None, 2)[2]
            for n in names.split(","):
                out.append(n.strip().lstrip("*").strip())
        return out

    assert fields("nt_options") == [f for f, _ in binding.Options._fields_]
    assert fields("nt_step_stats") == [f for f, _ in binding.StepStats._fields_]
    assert fields("nt_particles") == [f for f, _ in binding.ParticlesView._fields_]


def test_product_never_imports_oracle():
    for py in PKG.rglob("*.py"):
        tree = ast.parse(py.read_text())
        for node in ast.walk(tree):
            if isinstance(node, ast.Import):
                assert all(not a.name.startswith("oracle") for a in node.names), py
            if isinstance(node, ast.ImportFrom):
                assert not (node.module or "").startswith("oracle"), py
    for src in (PKG / "csrc").glob("*"):
        for inc in re.findall(r'#include\s*[<"]([^>"]+)[>"]', src.read_text()):
            assert "oracle" not in inc, (src, inc)


def test_missing_library_fails_loudly(tmp_path, monkeypatch):
    from paper_conf_cluster_martineaum17_b200 import binding
    monkeypatch.setattr(binding, "_lib", None)
    monkeypatch.setattr(binding, "LIB_PATH", tmp_path / "nope.so")
    with pytest.raises(ImportError):
        binding.lib()


def test_bench_roofline_inputs():
    """bench.py's two roofline denominators load from committed, driver- or B200-measured files
    (MEASURED_PEAKS.json; profiles/r01_v16_red_microbench.json), and its byte and
    RED counts follow SURVEY §8(d) (24 B per facet, 16 B per flush, 138 B per particle)."""
    import bench
    assert bench.measured_peaks()["hbm_gbs"] > 1000.0
    peak = bench.l2_red_peak()
    assert peak is not None and 1e10 < peak < 1e12
    s = {"n_facets": 10, "n_census": 2, "n_killed": 1, "n_alive_start": 3}
    assert bench.algorithmic_bytes(s) == 24 * 10 + 16 * 3 + 138 * 3


def test_bench_issue_roofline():
    """The ALU (instruction-issue) roofline of a collision-dominated config: committed ncu
    instruction counts over the kernel time against SMs x 4 schedulers x clock."""
    import bench
    r = bench.issue_roofline("scatter", "history", 7.4, 1965.0, 148)
    assert r is not None and r["bound"] == "alu"
    assert r["peak"] == 148 * 4 * 1965e6
    assert 0.3 < r["frac"] < 1.0
    assert bench.issue_roofline("no_such_config", "history", 7.4, 1965.0, 148) is None
