"""Summarise an ncu report: per kernel launch the time, DRAM bytes, issue activity,
stall breakdown and the hottest SASS lines (needs -lineinfo + --import-source)."""
import csv
import io
import subprocess
import sys


def ncu_csv(rep, *args):
    out = subprocess.run(["ncu", "-i", rep, *args, "--csv"], capture_output=True, text=True).stdout
    return list(csv.reader(io.StringIO(out)))


def main(rep, kernel_regex=None, top=12):
    rows = ncu_csv(rep, "--page", "raw")
    hdr, units = rows[0], rows[1]
    for row in rows[2:]:
        d = {h: (f"{v} {u}".strip() if u and h.startswith("dram__bytes") else v) for h, v, u in zip(hdr, row, units)}
        name = d["Kernel Name"]
        if kernel_regex and kernel_regex not in name:
            continue
        f = lambda k: d.get(k, "?")
        print(f"== {name[:60]}  id={f('ID')}")
        print(f"   time {f('gpu__time_duration.sum')} us  dram rd {f('dram__bytes_read.sum')}  wr {f('dram__bytes_write.sum')}"
              f"  dram% {f('gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed')}  issue% {f('smsp__issue_active.avg.pct_of_peak_sustained_active')}"
              f"  warps% {f('sm__warps_active.avg.pct_of_peak_sustained_active')}  inst {f('smsp__inst_executed.sum')}  grid {f('launch__grid_size')}"
              f"  regs {f('launch__registers_per_thread')}")
        st = []
        for h, v in d.items():
            if h.startswith("smsp__pcsamp_warps_issue_stalled") and not h.endswith("not_issued"):
                try:
                    st.append((float(v), h.replace("smsp__pcsamp_warps_issue_stalled_", "")))
                except ValueError:
                    pass
        tot = sum(v for v, _ in st) or 1
        print("   stalls: " + ", ".join(f"{h} {v / tot * 100:.0f}%" for v, h in sorted(st, reverse=True)[:7]))


if __name__ == "__main__":
    main(sys.argv[1], sys.argv[2] if len(sys.argv) > 2 else None)


def hot_lines(rep, kernel_regex, top=25, by="Warp Stall Sampling (All Samples)"):
    rows = ncu_csv(rep, "--page", "source", "-k", f"regex:{kernel_regex}", "--launch-count", "1",
                   "--print-source", "sass")
    hi = [i for i, x in enumerate(rows) if by in x][0]
    hdr = rows[hi]
    body = [x for x in rows[hi + 1:] if len(x) == len(hdr)]
    i_s, i_src, i_ex = hdr.index(by), hdr.index("Source"), hdr.index("Instructions Executed")

    def num(v):
        try:
            return float(v)
        except ValueError:
            return 0.0
    tot = sum(num(x[i_s]) for x in body)
    print(f"   total {by}: {tot:.0f}; instructions executed: {sum(num(x[i_ex]) for x in body):.0f}")
    for x in sorted(body, key=lambda x: -num(x[i_s]))[:top]:
        print(f"   {num(x[i_s]):8.0f} {num(x[i_ex]):10.0f}  {x[0][-5:]}  {x[i_src].strip()[:90]}")


def hot_blocks(rep, kernel_regex, top=14, key="inst"):
    """Group SASS into runs of equal execution count (≈ basic blocks); rank by instructions or stalls."""
    rows = ncu_csv(rep, "--page", "source", "-k", f"regex:{kernel_regex}", "--launch-count", "1",
                   "--print-source", "sass")
    hi = [i for i, x in enumerate(rows) if "Instructions Executed" in x][0]
    hdr = rows[hi]
    body = []
    for x in rows[hi + 1:]:
        if "Instructions Executed" in x:
            break                      # next launch's table
        if len(x) == len(hdr):
            body.append(x)
    ie, src = hdr.index("Instructions Executed"), hdr.index("Source")
    ws = hdr.index("Warp Stall Sampling (All Samples)")
    blocks = []
    for x in body:
        c, s = float(x[ie] or 0), float(x[ws] or 0)
        if blocks and blocks[-1][0] == c:
            blocks[-1][1] += 1
            blocks[-1][3] += s
            blocks[-1][4].append(x[src].strip())
        else:
            blocks.append([c, 1, x[0][-5:], s, [x[src].strip()]])
    tot = sum(b[0] * b[1] for b in blocks) or 1
    tws = sum(b[3] for b in blocks) or 1
    print(f"   instructions {tot:.0f}, stall samples {tws:.0f}")
    k = (lambda b: -b[0] * b[1]) if key == "inst" else (lambda b: -b[3])
    for b in sorted(blocks, key=k)[:top]:
        print(f"   {b[0]:9.0f} x{b[1]:4d} = {b[0] * b[1] / tot * 100:5.1f}% inst {b[3] / tws * 100:5.1f}% stall"
              f" @{b[2]}: {' | '.join(b[4][:7])[:170]}")


def hot_src(rep, kernel_regex, top=30):
    """Per CUDA source line (all files): instructions executed and stall samples (-lineinfo + --import-source)."""
    rows = ncu_csv(rep, "--page", "source", "-k", f"regex:{kernel_regex}", "--launch-count", "1",
                   "--print-source", "cuda,sass")
    fname, hdr, lines = "?", None, []
    for x in rows:
        if len(x) == 2 and x[0] == "File Path":
            fname = x[1].rsplit("/", 1)[-1]
        elif "Instructions Executed" in x:
            hdr = x
        elif hdr and len(x) == len(hdr) and x[0] not in ("", "-"):
            lines.append((fname, x[0], x[1], float(x[hdr.index("Instructions Executed")] or 0),
                          float(x[hdr.index("Warp Stall Sampling (All Samples)")] or 0)))
    tot = sum(l[3] for l in lines) or 1
    tws = sum(l[4] for l in lines) or 1
    print(f"   instructions {tot:.0f}, stall samples {tws:.0f}")
    for f, ln, src, ie, ws in sorted(lines, key=lambda l: -l[3])[:top]:
        print(f"   {ie / tot * 100:5.1f}% inst {ws / tws * 100:5.1f}% stall  {f}:{ln:<5} {src.strip()[:100]}")
