#!/usr/bin/env python
"""Mutation check of the oracle's pins: apply one plausible mistake at a time to
oracle/neutral_oracle.c, rebuild, run the CPU pin suite (-m "not gpu").  Works on a copy
of the repository under /tmp, so the tree itself is never mutated.

Every mutation must turn at least one pin red.  Output: one line per mutation with the
failing test count (profiles/r02_oracle_mutations.txt holds the committed run).

    python scripts/dev/oracle_mutations.py [--out profiles/r02_oracle_mutations.txt]
"""
import argparse
import shutil
import subprocess
import sys
import tempfile
from pathlib import Path

REPO = Path(__file__).resolve().parents[2]

MUTATIONS = {
    "census timer not converted at a collision (drop dcen = tcen * v)":
        ("            dcen = tcen * v;\n", ""),
    "census timer converted with the pre-collision speed":
        ("            v = or_speed(e);\n            dcen = tcen * v;", "            dcen = tcen * v;\n            v = or_speed(e);"),
    "census does not carry n_mfp (drop the census n_mfp update)":
        ("            double nm = mfp - ds * sig;\n            mfp = nm > 0.0 ? nm : 0.0;\n            or_flush",
         "            or_flush"),
    "facet does not update n_mfp":
        ("            double nm = mfp - df * sig;\n            mfp = nm > 0.0 ? nm : 0.0;\n            dcen = dcen - df;",
         "            dcen = dcen - df;"),
    "wrong heating constant f = (A^2+A+1)/(A+1)^2":
        ("double f = (A * A + 1.0) / ((A + 1.0) * (A + 1.0));", "double f = (A * A + A + 1.0) / ((A + 1.0) * (A + 1.0));"),
    "squared capture probability":
        ("w = w * (1.0 - m.pa);", "w = w * (1.0 - m.pa * m.pa);"),
    "transposed rotation":
        ("double nox = ox * ct - oy * stt;", "double nox = ox * ct + oy * stt;"),
    "Sigma_t from sigma_s only":
        ("    double t = ss + sa;\n    double A", "    double t = ss + 0.0 * sa;\n    double A"),
    "mu from word b":
        ("double mu = 1.0 - 2.0 * or_u01(r[0]);", "double mu = 1.0 - 2.0 * or_u01(r[1]);"),
    "new n_mfp from word a":
        ("double mfp_u = or_u01(r[1]);           /* the draw for the new n_mfp  */",
         "double mfp_u = or_u01(r[0]);           /* the draw for the new n_mfp  */"),
    "density not reloaded at a facet":
        ("            nd = pb->density[(int64_t)cy * nx + cx] * cn;   /* load new density */\n", ""),
    "Threefry rotation constant":
        ("{16, 42, 12, 31, 16, 32, 24, 21}", "{16, 42, 12, 31, 16, 32, 24, 22}"),
    "census deposit uses the facet distance":
        ("            acc += ((w * ds) * sig) * m.H;", "            acc += ((w * dcen * 0.5) * sig) * m.H;"),
    "collision does not advance the census timer":
        ("            dcen = dcen - dc;\n", ""),
    "X-facet deposit flushed into the entered cell":
        ("                or_flush(tally, nx, cx, cy, &acc, &dep, st);\n"
         "                int at_boundary = ox > 0.0 ? cx == nx - 1 : cx == 0;\n"
         "                if (at_boundary && pb->boundary) { escaped = 1; }\n"
         "                else if (ox > 0.0) {\n"
         "                    if (cx == nx - 1) { ox = -ox; iox = -iox; } else { cx += 1; }\n"
         "                } else {\n"
         "                    if (cx == 0) { ox = -ox; iox = -iox; } else { cx -= 1; }\n"
         "                }\n",
         "                int at_boundary = ox > 0.0 ? cx == nx - 1 : cx == 0;\n"
         "                if (at_boundary && pb->boundary) { escaped = 1; }\n"
         "                else if (ox > 0.0) {\n"
         "                    if (cx == nx - 1) { ox = -ox; iox = -iox; } else { cx += 1; }\n"
         "                } else {\n"
         "                    if (cx == 0) { ox = -ox; iox = -iox; } else { cx -= 1; }\n"
         "                }\n"
         "                or_flush(tally, nx, cx, cy, &acc, &dep, st);\n"),
    "tie rule: facet axis tie -> X":
        ("        int axis_x = tx < ty;", "        int axis_x = tx <= ty;"),
}


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--out", default=None)
    a = ap.parse_args()
    tmp = Path(tempfile.mkdtemp(prefix="oracle_mut_"))
    ROOT = tmp / "repo"
    shutil.copytree(REPO, ROOT, ignore=shutil.ignore_patterns(".git", "gpurun_out", "build",
                                                              "__pycache__"))
    SRC = ROOT / "oracle" / "neutral_oracle.c"
    LIB = ROOT / "oracle" / "liboracle.so"
    orig = SRC.read_text()
    lines = []
    try:
        for name, (old, new) in MUTATIONS.items():
            assert orig.count(old) == 1, f"mutation anchor not unique/found: {name}"
            SRC.write_text(orig.replace(old, new))
            LIB.unlink(missing_ok=True)
            r = subprocess.run([sys.executable, "-m", "pytest", "tests", "-q", "-m", "not gpu", "-p", "no:cacheprovider"],
                               cwd=ROOT, capture_output=True, text=True)
            tail = r.stdout.strip().splitlines()[-1] if r.stdout.strip() else r.stderr[-200:]
            failed = [l.split(" ")[1] for l in r.stdout.splitlines() if l.startswith("FAILED ")]
            files = sorted({f.split("::")[0] for f in failed})
            line = f"{'RED  ' if r.returncode else 'GREEN'} {name}: {tail} :: {', '.join(files)}"
            print(line, flush=True)
            lines.append(line)
    finally:
        shutil.rmtree(tmp, ignore_errors=True)
    if a.out:
        Path(a.out).write_text("\n".join(lines) + "\n")
    return 0 if all(l.startswith("RED") for l in lines) else 1


if __name__ == "__main__":
    sys.exit(main())
