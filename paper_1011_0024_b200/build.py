"""Build libqudax.so in-tree: nvcc, sm_100a only (-gencode arch=compute_100a,code=sm_100a),
-lineinfo for ncu source correlation.  NCCL is the same 2.28 wheel PyTorch loads.

    python -m paper_1011_0024_b200.build [--force] [-v]
"""
import concurrent.futures as cf
import glob
import os
import subprocess
import sys

HERE = os.path.dirname(os.path.abspath(__file__))
ROOT = os.path.dirname(HERE)
CSRC = os.path.join(HERE, "csrc")
OUT_DIR = os.path.join(HERE, "lib")
LIB = os.path.join(OUT_DIR, "libqudax.so")
NVCC = os.environ.get("NVCC", "/usr/local/cuda/bin/nvcc")
ARCH = ["-gencode", "arch=compute_100a,code=sm_100a"]


def nccl_dirs():
    import importlib.util
    spec = importlib.util.find_spec("nvidia")
    for base in list(spec.submodule_search_locations or []):
        inc = os.path.join(base, "nccl", "include")
        lib = os.path.join(base, "nccl", "lib")
        if os.path.exists(os.path.join(inc, "nccl.h")) and os.path.exists(os.path.join(lib, "libnccl.so.2")):
            return inc, lib
    raise RuntimeError("NCCL wheel (nvidia/nccl) not found")


def _needs(obj, deps):
    if not os.path.exists(obj):
        return True
    t = os.path.getmtime(obj)
    return any(os.path.getmtime(d) > t for d in deps)


def build(force=False, verbose=False, out_dir=None, defines=()):
    """Compile and link libqudax.so.  out_dir/defines build experiment variants elsewhere
    (e.g. -DQX_DSLASH_MINB=6); the product library is the default one in lib/."""
    global OUT_DIR, LIB
    if out_dir is not None:
        OUT_DIR, LIB = out_dir, os.path.join(out_dir, "libqudax.so")
    inc, lib = nccl_dirs()
    os.makedirs(os.path.join(OUT_DIR, "obj"), exist_ok=True)
    headers = glob.glob(os.path.join(CSRC, "*.h")) + glob.glob(os.path.join(CSRC, "*.cuh")) + \
        [os.path.join(ROOT, "include", "qudax.h")]
    srcs = sorted(glob.glob(os.path.join(CSRC, "*.cu")) + glob.glob(os.path.join(CSRC, "*.cpp")))
    common = ["-O3", "-std=c++17", "-Xcompiler", "-fPIC", "-I", os.path.join(ROOT, "include"), "-I", CSRC, "-I", inc]
    common += [f"-D{d}" for d in defines]
    jobs = []
    objs = []
    for s in srcs:
        o = os.path.join(OUT_DIR, "obj", os.path.basename(s) + ".o")
        objs.append(o)
        if force or _needs(o, [s] + headers):
            cmd = [NVCC] + ARCH + common + ["-lineinfo", "-Xptxas", "-v" if verbose else "-O3", "-c", s, "-o", o]
            if s.endswith(".cpp"):
                cmd = [NVCC] + common + ["-x", "c++", "-c", s, "-o", o]
            jobs.append((s, cmd))
    errors = []
    with cf.ThreadPoolExecutor(max_workers=os.cpu_count() or 4) as ex:
        futs = {ex.submit(subprocess.run, cmd, capture_output=True, text=True): s for s, cmd in jobs}
        for f in cf.as_completed(futs):
            r = f.result()
            if r.returncode != 0:
                errors.append(f"== {futs[f]}\n{r.stdout}\n{r.stderr}")
            elif verbose:
                sys.stderr.write(f"== {futs[f]}\n{r.stderr}")
    if errors:
        raise RuntimeError("nvcc failed:\n" + "\n".join(errors))
    if force or jobs or not os.path.exists(LIB):
        link = [NVCC] + ARCH + ["-shared", "-cudart", "static", "-o", LIB] + objs + \
            ["-L", lib, "-l:libnccl.so.2", "-Xlinker", f"-rpath={lib}"]
        r = subprocess.run(link, capture_output=True, text=True)
        if r.returncode != 0:
            raise RuntimeError("link failed:\n" + r.stdout + r.stderr)
    return LIB


if __name__ == "__main__":
    defs = [a[2:] for a in sys.argv[1:] if a.startswith("-D")]
    od = next((a.split("=", 1)[1] for a in sys.argv[1:] if a.startswith("--out=")), None)
    print(build(force="--force" in sys.argv, verbose="-v" in sys.argv, out_dir=od, defines=defs))
