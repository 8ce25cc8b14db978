"""Host-side logic of the library that needs no GPU (-m "not gpu"): the magic-number division
the Dslash uses for its site coordinates (internal.h make_fastdiv; the device applies
q = umulhi(n, m) >> sh), compiled from the library's own header with the host compiler and
checked against exact integer division over every divisor a lattice extent can take."""
import os
import subprocess
import textwrap

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))

SRC = textwrap.dedent("""
    #include <cstdio>
    #include <cstdint>
    #include "internal.h"
    static int fdiv_host(int n, const qx::FastDiv &f) {  // the device formula, __umulhi spelled out
        if (!f.m) return n;
        const unsigned hi = (unsigned)(((unsigned long long)(unsigned)n * f.m) >> 32);
        return (int)(hi >> f.sh);
    }
    int main() {
        long bad = 0, checked = 0;
        unsigned long long s = 12345;
        for (int d = 1; d <= 4096; ++d) {
            const qx::FastDiv f = qx::make_fastdiv(d);
            const int edge[] = {0, 1, d - 1, d, d + 1, 2 * d - 1, 0x7fffffff, 0x7fffffff - d, 1 << 30};
            for (int n : edge) { if (n < 0) continue; ++checked; if (fdiv_host(n, f) != n / d) ++bad; }
            for (int k = 0; k < 2000; ++k) {
                s = s * 6364136223846793005ULL + 1442695040888963407ULL;
                const int n = (int)((s >> 33) & 0x7fffffff);
                ++checked;
                if (fdiv_host(n, f) != n / d) ++bad;
            }
        }
        std::printf("%ld %ld\\n", checked, bad);
        return bad != 0;
    }
""")


def test_fastdiv_matches_integer_division(tmp_path):
    cuda_inc = "/usr/local/cuda/include"
    if not os.path.exists(os.path.join(cuda_inc, "cuda_runtime.h")):
        pytest.skip("CUDA headers not available")
    src = tmp_path / "fd.cpp"
    src.write_text(SRC)
    exe = tmp_path / "fd"
    inc = [os.path.join(ROOT, "include"), os.path.join(ROOT, "paper_1011_0024_b200", "csrc"), cuda_inc]
    subprocess.run(["g++", "-O2", "-std=c++17", *[f"-I{i}" for i in inc], str(src), "-o", str(exe)], check=True)
    out = subprocess.run([str(exe)], capture_output=True, text=True)
    checked, bad = map(int, out.stdout.split())
    assert checked > 8_000_000 and bad == 0, out.stdout
