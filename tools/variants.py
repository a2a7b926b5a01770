"""Build a patched copy of the package under /tmp (tuning aid; the library in
the repo is not changed): variant(tag, [(csrc file, old, new), ...]) -> dir,
whose liblift.so is built from the patched sources.  Run timing code with
cwd = that dir so `import paper_conf_cgo_steuwerrd17_b200` loads the copy."""
import os
import shutil
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
PKG = "paper_conf_cgo_steuwerrd17_b200"


def variant(tag: str, patches) -> str:
    d = f"/tmp/variant_{tag}"
    shutil.rmtree(d, ignore_errors=True)
    os.makedirs(d)
    for sub in (PKG, "include", "synth", "tools"):
        shutil.copytree(os.path.join(ROOT, sub), os.path.join(d, sub),
                        ignore=shutil.ignore_patterns("_build", "*.so", "__pycache__"))
    for fname, old, new in patches:
        f = os.path.join(d, PKG, "csrc", fname)
        s = open(f).read()
        assert old in s, (fname, old)
        open(f, "w").write(s.replace(old, new))
    subprocess.run([sys.executable, "-c", f"import sys; sys.path.insert(0, '{d}'); from {PKG} import build; "
                    "build.build(force=True)"], check=True, cwd=d)
    return d


def run(d: str, code: str, **env) -> None:
    subprocess.run([sys.executable, "-c", code], cwd=d, check=True, env=dict(os.environ, **env))
