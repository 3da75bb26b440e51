"""GPU parity of the one-pass result-ring kernels (fused.cu, ar_select_refine_sum:
fused_rg_kernel with the residual sectors of non-definite candidates gathered
and refined one tile later, fused_rl_kernel with the exact predicate on
streamed residual planes) against the CPU oracle:
ragged tails, every SUM-factor mode (COUNT only, predicate-column factors,
one gathered column with and without a second factor), ring overflow at high
selectivity, and every (warps, blocks-per-thread) configuration plus the
general kernel in subprocesses (the kernel choice is read from the
environment once per process)."""
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


@pytest.fixture(scope="module")
def cu():
    if not torch.cuda.is_available():
        pytest.skip("no CUDA device")
    from paper_conf_icde_pirkmk14_b200 import column
    return column


def q6(cu, seed, n, bounds=None):
    from paper_conf_icde_pirkmk14_b200 import _ar
    c = datagen.q6_columns(seed, 1.0, n=n)
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    if bounds:
        los, his = [b[0] for b in bounds], [b[1] for b in bounds]
    cols = {"shipdate": cu.BWDColumn(c["shipdate"], 24), "discount": cu.BWDColumn(c["discount"], 32),
            "quantity": cu.BWDColumn(c["quantity"], 32),
            "extprice": cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)}
    return c, cols, los, his


def run(cu, c, cols, los, his, aggs):
    from paper_conf_icde_pirkmk14_b200 import _ar
    preds = [(cols["shipdate"], los[0], his[0]), (cols["discount"], los[1], his[1]),
             (cols["quantity"], los[2], his[2])]
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [cols[a] for a in aggs], o4)
    torch.cuda.synchronize()
    kernel = _ar.ar_last_scan_kernel()
    values = [c["shipdate"], c["discount"], c["quantity"]]
    _, ref_cnt, ref_sum = oracle.select_sum(values, los, his, [c[a] for a in aggs], positions=False)
    cpos, cdef = oracle.approx_select(values, [8, 0, 0], los, his)
    assert o4.cpu().tolist() == [ref_sum if aggs else 0, ref_cnt, cpos.size, int(cdef.sum())]
    return kernel, ref_cnt


@pytest.mark.parametrize("n", [1, 31, 8191, 8192, 8193, 3 * 8192 + 127, 300_001])
@pytest.mark.parametrize("aggs", [("extprice", "discount"), ("extprice",), (), ("discount",),
                                  ("discount", "quantity")])
def test_rl_q6_modes_and_tails(cu, n, aggs):
    c, cols, los, his = q6(cu, 40 + n % 97, n)
    kernel, _ = run(cu, c, cols, los, his, list(aggs))
    if n >= 8192:
        assert kernel == "fused_rl_kernel"


@pytest.mark.parametrize("aggs", [("extprice", "discount"), ("extprice", "quantity")])
def test_rl_ring_overflow(cu, aggs):
    # unaligned shipdate bounds keep both boundary buckets (12.5 % of the 16 majors) non-definite,
    # so the residual planes stream; nearly every row qualifies, so each warp's share of a tile
    # overflows the 256-entry result ring many times over
    c, cols, los, his = q6(cu, 7, 200_000, bounds=[(3, 2523), (0, 10), (1, 50)])
    kernel, cnt = run(cu, c, cols, los, his, list(aggs))
    assert kernel == "fused_rl_kernel" and cnt > 190_000


def test_rl_single_column_c1(cu):
    v = datagen.uniform_u32(1, datagen.C1_N)
    col = cu.BWDColumn(v, 24)
    # a 25 %-wide range: the two boundary buckets are non-definite, residual planes stream (AR_RES_STREAM
    # heuristics: forced on by the subprocess sweep below for the narrow C1 range)
    lo, hi = 0x12345678, 0x12345678 + (1 << 30)
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum([(col, lo, hi)], [col], o4)
    torch.cuda.synchronize()
    _, cnt, s = oracle.select_sum([v], [lo], [hi], [v], positions=False)
    cpos, cdef = oracle.approx_select([v], [8], [lo], [hi])
    assert o4.cpu().tolist() == [s, cnt, cpos.size, int(cdef.sum())]


SWEEP = r"""
import sys, numpy as np, torch
sys.path.insert(0, {root!r})
import datagen, oracle
from paper_conf_icde_pirkmk14_b200 import _ar, column as cu
want, want_c1 = sys.argv[1], sys.argv[2]
for seed, n, bounds in [(3, 100_003, None), (4, 70_001, [(3, 2523), (0, 10), (1, 50)])]:
    c = datagen.q6_columns(seed, 1.0, n=n)
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    if bounds:
        los, his = [b[0] for b in bounds], [b[1] for b in bounds]
    sd, dc, qt = cu.BWDColumn(c["shipdate"], 24), cu.BWDColumn(c["discount"], 32), cu.BWDColumn(c["quantity"], 32)
    ep = cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)
    preds = [(sd, los[0], his[0]), (dc, los[1], his[1]), (qt, los[2], his[2])]
    vals = [c["shipdate"], c["discount"], c["quantity"]]
    cpos, cdef = oracle.approx_select(vals, [8, 0, 0], los, his)
    for aggs in ([ep, dc], [ep], []):
        o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
        cu.select_refine_sum(preds, aggs, o4)
        torch.cuda.synchronize()
        assert _ar.ar_last_scan_kernel() == want, (_ar.ar_last_scan_kernel(), want)
        av = [c["extprice"], c["discount"]][:len(aggs)]
        _, cnt, s = oracle.select_sum(vals, los, his, av, positions=False)
        assert o4.cpu().tolist() == [s if aggs else 0, cnt, cpos.size, int(cdef.sum())], (o4.tolist(), s, cnt)
# C1: narrow range, residual streaming forced on
v = datagen.uniform_u32(1, datagen.C1_N)
col = cu.BWDColumn(v, 24)
o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
cu.select_refine_sum([(col, datagen.C1_LO, datagen.C1_HI)], [col], o4)
torch.cuda.synchronize()
assert _ar.ar_last_scan_kernel() == want_c1, (_ar.ar_last_scan_kernel(), want_c1)
o1 = torch.zeros(4, dtype=torch.int64, device="cuda")
cu.select_refine_sum([(col, datagen.C1_LO, datagen.C1_HI)], [], o1)   # COUNT: the gathered kernel applies too
torch.cuda.synchronize()
_, cnt, s = oracle.select_sum([v], [datagen.C1_LO], [datagen.C1_HI], [v], positions=False)
cpos, cdef = oracle.approx_select([v], [8], [datagen.C1_LO], [datagen.C1_HI])
assert o4.cpu().tolist() == [s, cnt, cpos.size, int(cdef.sum())]
assert o1.cpu().tolist() == [0, cnt, cpos.size, int(cdef.sum())]
print("ok")
"""


@pytest.mark.parametrize("env,want,want_c1", [
    ({"AR_RL_CFG": "0", "AR_RL_RESMODE": "1"}, "fused_rl_kernel", "fused_rl_kernel"),
    ({"AR_RL_CFG": "1", "AR_RL_RESMODE": "1"}, "fused_rl_kernel", "fused_rl_kernel"),
    ({"AR_RL_CFG": "2", "AR_RL_RESMODE": "1"}, "fused_rl_kernel", "fused_rl_kernel"),
    ({"AR_RL_CFG": "0", "AR_RL_RESMODE": "2"}, "fused_rg_kernel", "fused_kernel"),
    ({"AR_RL_CFG": "1", "AR_RL_RESMODE": "2"}, "fused_rg_kernel", "fused_kernel"),
    ({"AR_RL_CFG": "3", "AR_RL_RESMODE": "2"}, "fused_rg_kernel", "fused_kernel"),
    ({"AR_RL_CFG": "4", "AR_RL_RESMODE": "2"}, "fused_rg_kernel", "fused_kernel"),
    ({"AR_RL_CFG": "0"}, "fused_rl_kernel", "fused_rl_kernel"),
    ({"AR_FUSED_LEGACY": "1"}, "fused_kernel", "fused_kernel")])
def test_rl_config_sweep_subprocess(cu, env, want, want_c1):
    e = dict(os.environ, AR_RES_STREAM="1", **env)
    r = subprocess.run([sys.executable, "-c", SWEEP.format(root=ROOT), want, want_c1], env=e, capture_output=True,
                       text=True, timeout=600)
    assert r.returncode == 0 and "ok" in r.stdout, r.stdout + r.stderr


@pytest.mark.parametrize("flags", [0, 1, 2])
def test_rl_workspace_and_pdl_back_to_back(cu, flags):
    # ar_select_refine_sum_ws: one launch per query, out4 written (not accumulated), ticket re-armed;
    # alternate two different queries on the same workspace and output, 6 calls without a sync
    from paper_conf_icde_pirkmk14_b200 import _ar
    c, cols, los, his = q6(cu, 91, 250_001)
    _, _, los2, his2 = q6(cu, 91, 8, bounds=[(3, 2523), (0, 10), (1, 50)])
    values = [c["shipdate"], c["discount"], c["quantity"]]
    ws = cu.SrsWorkspace()
    outs = [torch.full((4,), -7, dtype=torch.int64, device="cuda") for _ in range(6)]
    shared = torch.full((4,), -7, dtype=torch.int64, device="cuda")
    aggs = [cols["extprice"], cols["discount"]]
    for i in range(6):
        lo, hi = (los, his) if i % 2 == 0 else (los2, his2)
        preds = [(cols["shipdate"], lo[0], hi[0]), (cols["discount"], lo[1], hi[1]),
                 (cols["quantity"], lo[2], hi[2])]
        cu.select_refine_sum(preds, aggs, shared, ws=ws, flags=flags)
        outs[i].copy_(shared)
        assert _ar.ar_last_scan_kernel() == "fused_rl_kernel"
    torch.cuda.synchronize()
    for i in range(6):
        lo, hi = (los, his) if i % 2 == 0 else (los2, his2)
        _, cnt, s = oracle.select_sum(values, lo, hi, [c["extprice"], c["discount"]], positions=False)
        cpos, cdef = oracle.approx_select(values, [8, 0, 0], lo, hi)
        assert outs[i].cpu().tolist() == [s, cnt, cpos.size, int(cdef.sum())]
    assert int(ws.t[:4].view(torch.int32).item()) == 0        # ticket left zero


def test_rl_workspace_runtime_shape_and_empty(cu):
    # the workspace call on a shape without a compiled result-ring shape (the runtime-shape kernel) and
    # on an empty predicate still writes out4 (the output is not accumulated)
    from paper_conf_icde_pirkmk14_b200 import _ar
    v = datagen.uniform_u32(5, 100_000, 0, (1 << 11) - 1)      # w_major = 3: no compiled shape
    col = cu.BWDColumn(v, 24)
    ws = cu.SrsWorkspace()
    o4 = torch.full((4,), -7, dtype=torch.int64, device="cuda")
    cu.select_refine_sum([(col, 300, 1500)], [col], o4, ws=ws)
    torch.cuda.synchronize()
    assert _ar.ar_last_scan_kernel() == "fused_rl_kernel"
    _, cnt, s = oracle.select_sum([v], [300], [1500], [v], positions=False)
    cpos, cdef = oracle.approx_select([v], [8], [300], [1500])
    assert o4.cpu().tolist() == [s, cnt, cpos.size, int(cdef.sum())]
    o4.fill_(-7)
    cu.select_refine_sum([(col, 1500, 300)], [col], o4, ws=ws, flags=_ar.AR_SRS_PDL)
    torch.cuda.synchronize()
    assert o4.cpu().tolist() == [0, 0, 0, 0]


@pytest.mark.parametrize("n", [8193, 1_000_003])
@pytest.mark.parametrize("aggs", [("extprice", "discount"), ()])
def test_rg_host_resident_residual(cu, n, aggs):
    # the C5 mechanism: the l_shipdate residual in pinned host memory, gathered over the host link by the
    # two-phase kernel for the blocks that hold a non-definite candidate
    from paper_conf_icde_pirkmk14_b200 import _ar
    c, cols, los, his = q6(cu, 77, n)
    cols["shipdate"] = cu.BWDColumn(c["shipdate"], 24, residual_loc=_ar.AR_LOC_HOST_PINNED)
    kernel, _ = run(cu, c, cols, los, his, list(aggs))
    assert kernel == "fused_rg_kernel"


def test_rg_spatial_two_decomposed_predicates(cu):
    # two decomposed signed predicates (24/8, FOR base): both residuals gathered, COUNT
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 500_009
    s = datagen.spatial_columns(23, n)
    lon, lat = np.asarray(s["lon"], dtype=np.int32), np.asarray(s["lat"], dtype=np.int32)
    cl = [cu.BWDColumn(lon, 24, signed=True, base="min"), cu.BWDColumn(lat, 24, signed=True, base="min")]
    for los, his in (([datagen.SPATIAL_LON[0], datagen.SPATIAL_LAT[0]], [datagen.SPATIAL_LON[1], datagen.SPATIAL_LAT[1]]),
                     ([-900_000, 4_000_000], [600_000, 6_000_000])):
        preds = [(cl[0], los[0] & 0xFFFFFFFF, his[0] & 0xFFFFFFFF), (cl[1], los[1] & 0xFFFFFFFF, his[1] & 0xFFFFFFFF)]
        o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
        cu.select_refine_sum(preds, [], o4)
        torch.cuda.synchronize()
        kernel = _ar.ar_last_scan_kernel()
        _, cnt, _ = oracle.select_sum([lon, lat], los, his, signed=[True, True], positions=False)
        cpos, cdef = oracle.approx_select([lon, lat], [8, 8], los, his, base=[int(c.desc.base) for c in cl],
                                          signed=[True, True])
        assert o4.cpu().tolist() == [0, cnt, cpos.size, int(cdef.sum())]
        if cl[0].w_major == 24 and cl[1].w_major == 24:
            assert kernel == "fused_rg_kernel"


@pytest.mark.parametrize("ship_bits", [30, 28, 26, 25, 23])
@pytest.mark.parametrize("aggs", [("extprice", "discount"), (), ("discount",)])
def test_rl_runtime_shape_q6_splits(cu, ship_bits, aggs):
    # other bwdecompose(l_shipdate, M) splits (k = 2..9 residual bits): the runtime-shape result-ring
    # kernel where the residual planes stream (k <= 8), the general kernel otherwise; identical results
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 300_007
    c = datagen.q6_columns(57, 1.0, n=n)
    cols = {"shipdate": cu.BWDColumn(c["shipdate"], ship_bits), "discount": cu.BWDColumn(c["discount"], 32),
            "quantity": cu.BWDColumn(c["quantity"], 32),
            "extprice": cu.BWDColumn(c["extprice"], 32, layout=_ar.AR_LAYOUT_PACKED)}
    los = [datagen.Q6_SHIPDATE[0], datagen.Q6_DISCOUNT[0], datagen.Q6_QUANTITY[0]]
    his = [datagen.Q6_SHIPDATE[1], datagen.Q6_DISCOUNT[1], datagen.Q6_QUANTITY[1]]
    preds = [(cols["shipdate"], los[0], his[0]), (cols["discount"], los[1], his[1]),
             (cols["quantity"], los[2], his[2])]
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [cols[a] for a in aggs], o4)
    torch.cuda.synchronize()
    values = [c["shipdate"], c["discount"], c["quantity"]]
    _, cnt, sm = oracle.select_sum(values, los, his, [c[a] for a in aggs], positions=False)
    cpos, cdef = oracle.approx_select(values, [32 - ship_bits, 0, 0], los, his)
    assert o4.cpu().tolist() == [sm if aggs else 0, cnt, cpos.size, int(cdef.sum())]


def test_rl_runtime_shape_spatial_for_base(cu):
    # two signed 24/8 predicates with a frame-of-reference base (w_major < 24): runtime shape, COUNT
    from paper_conf_icde_pirkmk14_b200 import _ar
    n = 400_021
    s = datagen.spatial_columns(29, n)
    lon, lat = np.asarray(s["lon"], dtype=np.int32), np.asarray(s["lat"], dtype=np.int32)
    cl = [cu.BWDColumn(lon, 24, signed=True, base="min"), cu.BWDColumn(lat, 24, signed=True, base="min")]
    los, his = [-900_000, 4_000_000], [600_000, 6_000_000]
    preds = [(cl[0], los[0] & 0xFFFFFFFF, his[0] & 0xFFFFFFFF), (cl[1], los[1] & 0xFFFFFFFF, his[1] & 0xFFFFFFFF)]
    o4 = torch.zeros(4, dtype=torch.int64, device="cuda")
    cu.select_refine_sum(preds, [], o4)
    torch.cuda.synchronize()
    _, cnt, _ = oracle.select_sum([lon, lat], los, his, signed=[True, True], positions=False)
    cpos, cdef = oracle.approx_select([lon, lat], [8, 8], los, his, base=[int(c.desc.base) for c in cl],
                                      signed=[True, True])
    assert o4.cpu().tolist() == [0, cnt, cpos.size, int(cdef.sum())]
