"""GPU parity of the staged path against the CPU oracle: the one-kernel ordered
select (select_rr_kernel: round-robin look-back, entries written once at their
final offsets; a3) and, in a subprocess with AR_SEL_RR=0, the
tile kernel + compaction; then refine + SUM on the candidates
(refine_sum_sliced_kernel; Alg. 2, SUM over exact values
812-841).  Sizes from one row to several look-back rounds per CTA (24 M rows =
2930 tiles over at most 1024 CTAs), selectivities from none to all rows (tiles
past the 512-entry staging buffer take the dense path), ragged tails, with and
without the approximation tuple, K = 4 / 8 residual planes, every SUM-factor
mode."""
import os
import subprocess
import sys

import numpy as np
import pytest

import datagen
import oracle

pytestmark = pytest.mark.gpu
torch = pytest.importorskip("torch")
ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
Q6 = [datagen.Q6_SHIPDATE, datagen.Q6_DISCOUNT, datagen.Q6_QUANTITY]


@pytest.fixture(scope="module")
def cu():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_icde_pirkmk14_b200 import column
    return column


def staged(cu, n, seed, k, aggs, ep_bits=None, bounds=None, carry=True, check_select=True):
    """Q6-shaped columns (l_shipdate with k residual planes): ar_approx_select -> ar_refine_sum."""
    from paper_conf_icde_pirkmk14_b200 import _ar
    c = datagen.q6_columns(seed, 1.0, n=n)
    if ep_bits:   # another aggregate domain: packed values straddle 32-bit words
        c["extprice"] = datagen.uniform_u32(seed + 5, n, 0, (1 << ep_bits) - 1)
    bounds = bounds or Q6
    los, his = [b[0] for b in bounds], [b[1] for b in bounds]
    ks = [k, 0, 0]
    cols = {"shipdate": cu.BWDColumn(c["shipdate"], 32 - k), "discount": cu.BWDColumn(c["discount"], 32),
            "quantity": cu.BWDColumn(c["quantity"], 32),
            "extprice": cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)}
    pcols = [cols["shipdate"], cols["discount"], cols["quantity"]]
    preds = list(zip(pcols, los, his))
    cands = cu.CandidateList(n)
    ws = cu.Workspace(_ar.ar_select_ws_bytes(n))
    cu.approx_select(preds, cands, ws, carry=carry)
    torch.cuda.synchronize()
    sel_kernel = _ar.ar_last_scan_kernel()
    values = [c["shipdate"], c["discount"], c["quantity"]]
    if check_select:
        ref_pos, ref_def = oracle.approx_select(values, ks, los, his)
        assert cands.count() == ref_pos.size
        assert np.array_equal(cands.positions(), ref_pos)
        assert np.array_equal(cands.definite(), ref_def)
        if carry and ref_pos.size:
            aux = cands.aux_words().astype(np.uint64)
            shift = 0
            for v, kk, col in zip(values, ks, pcols):
                major, _, w = oracle.decompose(v, kk)
                got = (aux >> np.uint64(shift)) & np.uint64((1 << w) - 1)
                assert np.array_equal(got, major[ref_pos].astype(np.uint64))
                shift += w
    if not carry:
        return sel_kernel, None, cands.count(), None
    s = torch.zeros(1, dtype=torch.int64, device="cuda")
    cnt = torch.zeros(1, dtype=torch.int64, device="cuda")
    cu.refine_sum(cands, preds, [cols[a] for a in aggs], s, cnt)
    torch.cuda.synchronize()
    ref_kernel = _ar.ar_last_scan_kernel()
    _, ref_cnt, ref_sum = oracle.select_sum(values, los, his, [c[a] for a in aggs], positions=False)
    assert int(cnt.item()) == ref_cnt
    assert int(s.item()) == (ref_sum if aggs else 0)
    return sel_kernel, ref_kernel, cands.count(), ref_cnt


@pytest.mark.parametrize("n", [1, 100, 8191, 8193, 5_001_003, 24_000_011])
@pytest.mark.parametrize("k", [8, 4])
def test_staged_q6_sizes(cu, n, k):
    sel, ref, ncand, _ = staged(cu, n, 60 + n % 11, k, ["extprice", "discount"])
    assert sel == "select_rr_kernel" or (ncand == 0 and sel == "")   # "": a relaxed range is empty
    if ncand:
        assert ref == "refine_sum_sliced_kernel"


@pytest.mark.parametrize("bounds", [
    [(3, 2523), (0, 10), (1, 50)],        # nearly every row: every tile dense, both edges undecided
    [(0, 2600), (0, 10), (0, 5)],         # ~10-12 % of rows: a mix of staged and dense tiles
    [(1000, 1000), (0, 10), (0, 60)],     # one day: every candidate undecided
    [(768, 1023), (5, 7), (0, 23)],       # aligned: every candidate definite
    [(5000, 6000), (0, 10), (0, 60)],     # no row qualifies
])
def test_staged_bound_placements(cu, bounds):
    # default kernel choice: dense placements go to the tile kernel + compaction
    sel, ref, ncand, res = staged(cu, 6_000_001, 90, 8, ["extprice", "discount"], bounds=bounds)
    assert sel in ("select_rr_kernel", "select_tile_kernel") or (ncand == 0 and sel == "")
    assert ncand >= res


BOUNDS = [[(3, 2523), (0, 10), (1, 50)], [(0, 2600), (0, 10), (0, 5)], [(1000, 1000), (0, 10), (0, 60)],
          [(768, 1023), (5, 7), (0, 23)], [(5000, 6000), (0, 10), (0, 60)]]


@pytest.mark.parametrize("grid", ["0", "3"])
def test_rr_dense_paths_in_subprocess(grid):
    """AR_SEL_RR=2: the one-kernel select on every bound placement -- tiles staged in shared memory,
    through workspace slices (513-2048 candidates) and resolved at once (> 2048) -- with the whole
    grid and with 3 CTAs (many look-back rounds)."""
    code = (
        "import sys; sys.path.insert(0, %r); sys.path.insert(0, %r)\n"
        "import test_gpu_staged as t\n"
        "from paper_conf_icde_pirkmk14_b200 import column as cu\n"
        "for b in t.BOUNDS:\n"
        "    sel, _, ncand, res = t.staged(cu, 6_000_001, 90, 8, ['extprice', 'discount'], bounds=b)\n"
        "    assert sel == 'select_rr_kernel' or (ncand == 0 and sel == ''), sel\n"
        "print('ok')\n" % (ROOT, os.path.join(ROOT, "tests")))
    env = {**os.environ, "AR_SEL_RR": "2"}
    if grid != "0":
        env["AR_SEL_RR_GRID"] = grid
    r = subprocess.run([sys.executable, "-c", code], cwd=ROOT, capture_output=True, text=True, timeout=900,
                       env=env)
    assert r.returncode == 0 and "ok" in r.stdout, r.stderr[-3000:]


@pytest.mark.parametrize("aggs", [(), ("discount",), ("discount", "quantity"), ("extprice",),
                                  ("extprice", "quantity")])
def test_staged_factor_modes(cu, aggs):
    staged(cu, 2_000_003, 71, 8, list(aggs))


@pytest.mark.parametrize("ep_bits", [1, 7, 17, 24, 31, 32])
def test_staged_gathered_widths(cu, ep_bits):
    staged(cu, 1_000_033, 80 + ep_bits, 8, ["extprice", "discount"], ep_bits=ep_bits)


@pytest.mark.parametrize("n", [8193, 6_000_001])
def test_staged_select_without_tuple(cu, n):
    sel, _, _, _ = staged(cu, n, 33, 8, [], carry=False)
    assert sel == "select_rr_kernel"


@pytest.mark.parametrize("env", [{"AR_SEL_RR_CTAS": "1", "AR_SEL_RR_BUFS": "2"}, {"AR_SEL_RR_GRID": "3"},
                                 {"AR_SEL_RR_GRID": "1"}])
def test_staged_rr_grids_in_subprocess(env):
    """Fewer CTAs (one per SM, 3, 1): many look-back rounds per CTA, same results."""
    code = (
        "import sys; sys.path.insert(0, %r); sys.path.insert(0, %r)\n"
        "import test_gpu_staged as t\n"
        "from paper_conf_icde_pirkmk14_b200 import column as cu\n"
        "for n in (100, 5_001_003, 24_000_011):\n"
        "    sel, _, _, _ = t.staged(cu, n, 60 + n %% 11, 8, ['extprice', 'discount'])\n"
        "    assert sel == 'select_rr_kernel', sel\n"
        "sel, _, _, _ = t.staged(cu, 6_000_001, 90, 8, ['extprice'], bounds=[(0, 2600), (0, 10), (0, 5)])\n"
        "print('ok')\n" % (ROOT, os.path.join(ROOT, "tests")))
    r = subprocess.run([sys.executable, "-c", code], cwd=ROOT, capture_output=True, text=True, timeout=900,
                       env={**os.environ, "AR_SEL_RR": "2", **env})
    assert r.returncode == 0 and "ok" in r.stdout, r.stderr[-3000:]


def test_tile_kernel_and_compaction_in_subprocess():
    """AR_SEL_RR=0: the tile kernel + compaction (the choice is read once per process)."""
    code = (
        "import sys; sys.path.insert(0, %r); sys.path.insert(0, %r)\n"
        "import test_gpu_staged as t\n"
        "from paper_conf_icde_pirkmk14_b200 import column as cu\n"
        "for n in (100, 5_001_003, 24_000_011):\n"
        "    sel, _, _, _ = t.staged(cu, n, 60 + n %% 11, 8, ['extprice', 'discount'])\n"
        "    assert sel == 'select_tile_kernel', sel\n"
        "sel, _, _, _ = t.staged(cu, 6_000_001, 90, 8, ['extprice'], bounds=[(0, 2600), (0, 10), (0, 5)])\n"
        "assert sel == 'select_tile_kernel', sel\n"
        "print('ok')\n" % (ROOT, os.path.join(ROOT, "tests")))
    r = subprocess.run([sys.executable, "-c", code], cwd=ROOT, capture_output=True, text=True, timeout=900,
                       env={**os.environ, "AR_SEL_RR": "0"})
    assert r.returncode == 0 and "ok" in r.stdout, r.stderr[-3000:]


def test_rr_forced_on_narrow_planes_in_subprocess():
    """AR_SEL_RR=2: the one-kernel select also on shapes the default leaves to the tile kernel
    (fewer than 12 major planes), compared with the oracle by test_gpu_parity's checker."""
    code = (
        "import sys; sys.path.insert(0, %r); sys.path.insert(0, %r)\n"
        "import numpy as np, datagen, torch\n"
        "import test_gpu_parity as tp\n"
        "from paper_conf_icde_pirkmk14_b200 import column as cu, _ar\n"
        "for n, k, lo, hi in ((100_003, 24, 1 << 29, 3 << 29), (3_000_017, 24, 5 << 24, 5 << 24),\n"
        "                     (3_000_017, 28, 0, 1 << 31), (70_001, 16, 12345, 2 ** 32 - 7)):\n"
        "    v = datagen.uniform_u32(n + k, n)\n"
        "    tp.check_select(cu, [v], [k], [lo], [hi])\n"
        "    assert _ar.ar_last_scan_kernel() == 'select_rr_kernel', _ar.ar_last_scan_kernel()\n"
        "print('ok')\n" % (ROOT, os.path.join(ROOT, "tests")))
    r = subprocess.run([sys.executable, "-c", code], cwd=ROOT, capture_output=True, text=True, timeout=900,
                       env={**os.environ, "AR_SEL_RR": "2"})
    assert r.returncode == 0 and "ok" in r.stdout, r.stderr[-3000:]


@pytest.mark.parametrize("bounds", [None, [(3, 2523), (0, 10), (1, 50)], [(0, 2600), (0, 10), (0, 5)],
                                    [(1000, 1000), (0, 10), (0, 60)]])
def test_ordered_refine_positions(cu, bounds):
    """ar_refine (a5, positions out; refine_kernel: warp 0 resolves a tile's offset by look-back a
    round later while the CTA refines the next one): ascending exact positions equal to the oracle's,
    up to ~3000 tiles of 2048 candidates (several rounds of the ~600-CTA grid)."""
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 6_000_001
    c = datagen.q6_columns(95, 1.0, n=n)
    b = bounds or Q6
    los, his = [x[0] for x in b], [x[1] for x in b]
    cols = [cu.BWDColumn(c["shipdate"], 24), cu.BWDColumn(c["discount"], 32), cu.BWDColumn(c["quantity"], 32)]
    preds = list(zip(cols, los, his))
    cands = cu.CandidateList(n)
    cu.approx_select(preds, cands, cu.Workspace(_ar.ar_select_ws_bytes(n)), carry=True)
    out = cu.PositionList(n)
    cu.refine(cands, preds, out, cu.Workspace(_ar.ar_refine_ws_bytes(n)))
    torch.cuda.synchronize()
    assert _ar.ar_last_scan_kernel() == "refine_kernel"
    ref_pos, ref_cnt, _ = oracle.select_sum([c["shipdate"], c["discount"], c["quantity"]], los, his)
    assert out.count() == ref_cnt
    assert np.array_equal(out.positions(), ref_pos)
