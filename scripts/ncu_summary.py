#!/usr/bin/env python
"""Summarise an ncu --set full capture (run here, on the CPU box, with ncu -i).

    python scripts/ncu_summary.py gpurun_out/r01/prof.ncu-rep profiles/r01_csp_history_ncu.md \
        [--traffic-key csp/history]

Writes the key metrics (time, DRAM bytes, hit rates, REDs, occupancy, divergence, FP64 pipe,
stall reasons) and the top stall-sampled SASS lines; with --traffic-key also records
dram read+write bytes per launch into profiles/ncu_traffic.json (bench.py's roofline.traffic).
"""
from __future__ import annotations

import argparse
import csv
import io
import json
import re
import subprocess
from pathlib import Path

KEYS = [
    "gpu__time_duration.sum", "dram__bytes_read.sum", "dram__bytes_write.sum",
    "dram__throughput.avg.pct_of_peak_sustained_elapsed", "lts__t_sector_hit_rate.pct",
    "l1tex__t_sector_hit_rate.pct", "lts__t_requests_srcunit_tex_op_red.sum",
    "smsp__inst_executed_op_global_red.sum", "lts__throughput.avg.pct_of_peak_sustained_elapsed",
    "l1tex__throughput.avg.pct_of_peak_sustained_elapsed", "sm__warps_active.avg.pct_of_peak_sustained_active",
    "launch__registers_per_thread", "launch__occupancy_limit_registers", "launch__grid_size",
    "launch__block_size", "smsp__thread_inst_executed_per_inst_executed.ratio",
    "sm__pipe_fp64_cycles_active.avg.pct_of_peak_sustained_active", "smsp__inst_executed.sum",
    "smsp__issue_active.avg.pct_of_peak_sustained_active", "sm__throughput.avg.pct_of_peak_sustained_elapsed",
    # shared memory (the event variant's slot state)
    "smsp__inst_executed_op_shared_ld.sum", "smsp__inst_executed_op_shared_st.sum",
    "l1tex__data_pipe_lsu_wavefronts_mem_shared_op_ld.sum", "l1tex__data_pipe_lsu_wavefronts_mem_shared_op_st.sum",
    "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum", "l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum",
]
STALL = re.compile(r"^smsp__pcsamp_warps_issue_stalled_([a-z_]+)$")


def ncu(args):
    return subprocess.run(["ncu", *args], capture_output=True, text=True, check=True).stdout


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("rep")
    ap.add_argument("out")
    ap.add_argument("--traffic-key", default=None)
    ap.add_argument("--top", type=int, default=25)
    a = ap.parse_args()
    raw = list(csv.reader(io.StringIO(ncu(["-i", a.rep, "--page", "raw", "--csv"]))))
    hdr, units, rows = raw[0], raw[1], raw[2:]
    lines = [f"# ncu summary: {Path(a.rep).name}", ""]
    traffic = 0.0      # summed over the captured launches (history phases 1 + 2 of one step)
    inst = 0.0         # warp instructions issued, summed the same way (bench.py's issue roofline)
    for r in rows:
        d = dict(zip(hdr, r))
        u = dict(zip(hdr, units))
        lines.append(f"## kernel `{d.get('Kernel Name', '?')}`")
        lines.append("")
        lines.append("| metric | value | unit |")
        lines.append("|---|---|---|")
        for k in KEYS:
            if k in d:
                lines.append(f"| {k} | {d[k]} | {u[k]} |")
        stalls = {}
        for k, v in d.items():
            m = STALL.match(k)
            if m and v not in ("", "0"):
                try:
                    stalls[m.group(1)] = float(v.replace(",", ""))
                except ValueError:
                    pass
        tot = sum(stalls.values()) or 1.0
        lines.append("")
        lines.append("| stall reason (pc sampling) | share |")
        lines.append("|---|---|")
        for k, v in sorted(stalls.items(), key=lambda kv: -kv[1])[:12]:
            lines.append(f"| {k} | {100 * v / tot:.1f}% |")
        def num(k, scale):
            s = d.get(k, "").replace(",", "")
            f = float(s) if s else 0.0
            un = u.get(k, "")
            mult = {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9, "Tbyte": 1e12}.get(un, 1)
            return f * mult
        tr = num("dram__bytes_read.sum", 1) + num("dram__bytes_write.sum", 1)
        traffic += tr
        inst += num("smsp__inst_executed.sum", 1)
        lines.append("")
        lines.append(f"DRAM traffic of this launch (read + write): {tr:.4g} B")
        lines.append("")
    lines.append(f"DRAM traffic of all captured launches: {traffic:.4g} B")
    # source page: top stall-sampled SASS lines, per captured kernel (the page repeats a
    # "Kernel Name" row and a header row for every launch)
    try:
        src = list(csv.reader(io.StringIO(ncu(["-i", a.rep, "--page", "source", "--csv",
                                                "--print-source", "sass"]))))
        blocks, cur = [], None
        for row in src:
            if row and row[0] == "Kernel Name":
                cur = {"name": row[1] if len(row) > 1 else "", "rows": []}
                blocks.append(cur)
            elif cur is not None and row and row[0] == "Address":
                cur["h"] = row
            elif cur is not None and row:
                cur["rows"].append(row)
        seen, uniq = set(), []
        for b in blocks:                        # the page can repeat a launch; keep one copy
            key = (b["name"], len(b["rows"]), tuple(b["rows"][0]) if b["rows"] else ())
            if b["rows"] and "h" in b and key not in seen:
                seen.add(key)
                uniq.append(b)
        for nb, b in enumerate(uniq):
            h, body = b["h"], b["rows"]
            iS, iW = h.index("Source"), h.index("Warp Stall Sampling (All Samples)")
            iE, iT = h.index("Instructions Executed"), h.index("Avg. Threads Executed")
            num_ = lambda v: int(v) if v.strip().lstrip("-").isdigit() else 0  # noqa: E731
            tot = sum(num_(x[iW]) for x in body) or 1
            ex_tot = sum(num_(x[iE]) for x in body)
            lines += ["", f"### launch {nb}: top {a.top} stall-sampled SASS instructions "
                      f"({ex_tot:.4g} warp instructions executed)", "",
                      "| # | share | executed | avg threads | SASS |", "|---|---|---|---|---|"]
            for k, x in sorted(enumerate(body), key=lambda kx: -num_(kx[1][iW]))[:a.top]:
                lines.append(f"| {k} | {100 * num_(x[iW]) / tot:.1f}% | {x[iE]} | {x[iT]} | `{x[iS].strip()}` |")
            # executed-instruction mix by opcode (what the issue slots go to)
            mix: dict[str, int] = {}
            for x in body:
                op = x[iS].strip().split()
                if not op:
                    continue
                o = op[1] if op[0].startswith("@") and len(op) > 1 else op[0]
                mix[o.split(".")[0]] = mix.get(o.split(".")[0], 0) + num_(x[iE])
            lines += ["", f"opcode mix of launch {nb} (share of executed warp instructions): " +
                      ", ".join(f"{o} {100 * v / max(ex_tot, 1):.1f}%" for o, v in
                                sorted(mix.items(), key=lambda kv: -kv[1])[:24])]
    except Exception as e:  # noqa: BLE001
        lines.append(f"(source page unavailable: {e})")
    # CUDA source lines (needs -lineinfo and --import-source on): stall samples and executed
    # instructions of the SASS under each line of our .cu/.cuh files ("cuda,sass" listing:
    # a "File Path" row per file, a "Function Name" row per kernel, then each source line
    # followed by its SASS rows)
    try:
        src = list(csv.reader(io.StringIO(ncu(["-i", a.rep, "--page", "source", "--csv",
                                                "--print-source", "cuda,sass"]))))
        agg: dict[str, dict] = {}
        fname, func, line, h = "", "", None, None
        seen_pairs: dict = {}
        for row in src:
            if not row:
                continue
            if row[0] == "File Path":
                fname = Path(row[1]).name if len(row) > 1 else ""
            elif row[0] == "Function Name":
                # a (file, function) block repeats for every captured launch of the kernel
                fn = row[1] if len(row) > 1 else ""
                n_seen = seen_pairs.get((fname, fn), 0)
                seen_pairs[(fname, fn)] = n_seen + 1
                func = f"launch {n_seen}: {fn}"
                line = None
            elif row[0] == "Line No":
                h = row
            elif h is not None:
                if row[0]:
                    line = (row[0], row[1].strip())
                    continue
                if line is None:
                    continue
                iW = h.index("Warp Stall Sampling (All Samples)")
                iE = h.index("Instructions Executed")
                iT = h.index("Thread Instructions Executed")
                f = lambda v: float(v) if v.replace(".", "", 1).isdigit() else 0.0  # noqa: E731
                k = agg.setdefault(func, {}).setdefault((fname, line[0]), {"src": line[1], "w": 0.0, "e": 0.0, "t": 0.0})
                k["w"] += f(row[iW])
                k["e"] += f(row[iE])
                k["t"] += f(row[iT])
        for nb, (func, d) in enumerate(agg.items()):
            tot = sum(v["w"] for v in d.values()) or 1.0
            lines += ["", f"### {func[:70]}...: top {a.top} stall-sampled CUDA source lines", "",
                      "| file:line | stall share | warp instr executed | avg threads | source |", "|---|---|---|---|---|"]
            for (fn, ln), v in sorted(d.items(), key=lambda kv: -kv[1]["w"])[:a.top]:
                thr = v["t"] / v["e"] if v["e"] else 0.0
                lines.append(f"| {fn}:{ln} | {100 * v['w'] / tot:.1f}% | {v['e']:.4g} | {thr:.1f} | `{v['src'][:80]}` |")
    except Exception as e:  # noqa: BLE001
        lines.append(f"(CUDA source page unavailable: {e})")
    Path(a.out).write_text("\n".join(lines) + "\n")
    if a.traffic_key and traffic:
        p = Path(a.out).parent / "ncu_traffic.json"
        d = json.loads(p.read_text()) if p.exists() else {}
        d[a.traffic_key] = traffic
        p.write_text(json.dumps(d, indent=1, sort_keys=True) + "\n")
        p = Path(a.out).parent / "ncu_inst.json"
        d = json.loads(p.read_text()) if p.exists() else {}
        d[a.traffic_key] = inst
        p.write_text(json.dumps(d, indent=1, sort_keys=True) + "\n")
    print(f"wrote {a.out}")


if __name__ == "__main__":
    main()
