"""tools/ncu_flag_stall.py (the stall-on-flag evidence in profiles/r01_stall_*.txt): region
attribution of SASS stall samples on a hand-made `--page source --print-source cuda,sass` export."""
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

HDR = '"Line No","Source","Address","Source","Warp Stall Sampling (All Samples)","Warp Stall Sampling (Not-issued Samples)","stall_wait","stall_sleep"\n'


def _csv(tmp_path):
    nw = "/x/paper_conf_ppopp_mohantyc14_b200/csrc/wf_nw.cuh"
    helper = "/x/paper_conf_ppopp_mohantyc14_b200/csrc/wf_internal.h"
    rows = [
        f'"File Path","{nw}"\n', '"Function Name","nw_kernel"\n', HDR,
        '"320","seen = lds_vol_i(ctr);","-","-","0","0","0","0"\n',          # wait_ctr (compute wait)
        '"","","0x100","LDS R1, [R2]","30","30","30","0"\n',
        '"260","cells","-","-","0","0","0","0"\n',                            # compute cells
        '"","","0x300","VIADDMNMX R3","50","10","10","0"\n',
        '"700","io loop","-","-","0","0","0","0"\n',                          # I/O warp
        '"","","0x500","LDG.E.STRONG.SYS R4","10","10","10","0"\n',
        f'"File Path","{helper}"\n', '"Function Name","nw_kernel"\n', HDR,
        '"5","__nanosleep","-","-","0","0","0","0"\n',                        # inlined helper inside wait_ctr
        '"","","0x110","NANOSLEEP 0x14","10","10","0","10"\n',
    ]
    p = tmp_path / "src.csv"
    p.write_text("".join(rows))
    return str(p)


def test_regions_and_fractions(tmp_path):
    out = subprocess.run([sys.executable, os.path.join(ROOT, "tools", "ncu_flag_stall.py"), _csv(tmp_path), "nw"],
                         capture_output=True, text=True, check=True).stdout
    # 100 samples: wait_ctr 30 + the inlined NANOSLEEP 10 (inherits the wait region), cells 50, I/O 10
    assert "100 samples" in out
    assert "stall_on_flag_fraction (all warps: samples in flag / counter polling) = 0.500" in out
    assert "compute_warps_wait_fraction (compute-warp samples in dependency waits) = 0.444" in out
